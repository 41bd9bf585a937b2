// kernels.cu -- instantiates accel_persistent<T> / accel_native<T> for every
// built-in tenant, the table behind accel_builtin_kernel(), and the Virtual
// NDRange initialisation kernel (§5: "constructs a
// Virtual Kernel Execution Range which is copied to the accelerator memory").
#include <climits>
#include <cstring>

#include "device/dispatch.cuh"
#include "host/internal.h"
#include "tenants/histo.cuh"
#include "tenants/mop.cuh"
#include "tenants/stencil.cuh"

namespace accel {

static_assert(sizeof(Desc) == kDescBytes, "descriptor size");

__global__ void desc_init_kernel(const InitParams p, uint32_t n_desc) {
  const uint32_t i = blockIdx.x * blockDim.x + threadIdx.x;
  if (i == 0 && p.live_quota != nullptr) *p.live_quota = p.live_init;
  if (i >= n_desc) return;
  uint32_t s = 0;
  while (s + 1 < p.n_steps && i >= p.steps[s + 1].first) ++s;
  const InitStep& st = p.steps[s];
  const uint32_t r = i - st.first;
  Desc* d = p.d + i;
  d->total = st.total;
  d->gx = st.gx;
  d->gy = st.gy;
  d->gz = st.gz;
  d->chunk = st.chunk;
  d->launch_idx = r;
  d->flags = p.flags;
  d->total_seen = 0xffffffffu;
  d->live_quota = p.live_quota;
  d->coverage = p.coverage ? p.coverage + st.cov_offset + (size_t)r * st.total : nullptr;
  d->t_first = ULLONG_MAX;
  d->t_last = 0;
  d->ctas_started = 0;
  d->alive = 0;
  d->max_alive = 0;
  d->next = 0;
}

cudaError_t launch_desc_init(const InitParams& p, uint32_t n_desc, cudaStream_t s) {
  const uint32_t threads = 128;
  const uint32_t blocks = (n_desc + threads - 1) / threads;
  desc_init_kernel<<<blocks ? blocks : 1, threads, 0, s>>>(p, n_desc);
  return cudaGetLastError();
}

template <class T>
accel_kernel_desc make_desc(const char* name) {
  accel_kernel_desc d;
  d.name = name;
  d.persistent_fn = reinterpret_cast<const void*>(&accel_persistent<T>);
  d.native_fn = reinterpret_cast<const void*>(&accel_native<T>);
  d.block = accel_dim3{(uint32_t)T::kThreads, 1u, 1u};
  d.dyn_smem = T::kDynSmem;
  d.regs = 0;
  d.chunk = T::kChunk;
  d.args_size = sizeof(typename T::Args);
  return d;
}

namespace {
struct Builtin {
  const char* name;
  accel_kernel_desc (*make)(const char*);
};
const Builtin kBuiltins[] = {
    {"mop", &make_desc<Mop>},
    {"stencil", &make_desc<Stencil>},
    {"histo", &make_desc<Histo>},
};
constexpr int kNumBuiltins = sizeof(kBuiltins) / sizeof(kBuiltins[0]);
}  // namespace

}  // namespace accel

extern "C" int accel_builtin_kernel(const char* name, accel_kernel_desc* out) {
  if (!name || !out) return ACCEL_EINVAL;
  for (int i = 0; i < accel::kNumBuiltins; ++i)
    if (std::strcmp(accel::kBuiltins[i].name, name) == 0) {
      *out = accel::kBuiltins[i].make(accel::kBuiltins[i].name);
      return ACCEL_OK;
    }
  return ACCEL_EINVAL;
}

extern "C" int accel_builtin_count(void) { return accel::kNumBuiltins; }

extern "C" const char* accel_builtin_name(int i) {
  return (i >= 0 && i < accel::kNumBuiltins) ? accel::kBuiltins[i].name : nullptr;
}
