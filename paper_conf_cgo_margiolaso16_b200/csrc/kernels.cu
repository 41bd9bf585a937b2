// kernels.cu -- instantiates accel_persistent<T> / accel_native<T> for every
// built-in tenant, the table behind accel_builtin_kernel(), and the Virtual
// NDRange initialisation kernel (§5: "constructs a
// Virtual Kernel Execution Range which is copied to the accelerator memory").
#include <climits>
#include <cstring>

#include "device/dispatch.cuh"
#include "host/internal.h"
#include "tenants/bfs.cuh"
#include "tenants/cutcp.cuh"
#include "tenants/histo.cuh"
#include "tenants/mop.cuh"
#include "tenants/mriq.cuh"
#include "tenants/sad.cuh"
#include "tenants/lbm.cuh"
#include "tenants/gridding.cuh"
#include "tenants/sgemm.cuh"
#include "tenants/sgemm_tc.cuh"
#include "tenants/spmv.cuh"
#include "tenants/stencil.cuh"
#include "tenants/stencil_tma.cuh"
#include "tenants/tpacf.cuh"

namespace accel {

static_assert(sizeof(Desc) == kDescBytes, "descriptor size");
static_assert(sizeof(Ctl) == kCtlBytes, "control block size");

__global__ void desc_init_kernel(const InitParams p, uint32_t n_desc) {
  const uint32_t i = blockIdx.x * blockDim.x + threadIdx.x;
  if (i == 0 && p.ctl != nullptr) {
    p.ctl->live = p.live_init;
    p.ctl->grown = 0;
    p.ctl->lost = 0;
    p.ctl->cur = 0;
  }
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
  d->total_seen = kTerminate;
  d->ctl = p.ctl;
  d->coverage = p.coverage ? p.coverage + st.cov_offset + (size_t)r * st.total : nullptr;
  d->trace = p.trace ? p.trace + st.cov_offset + (size_t)r * st.total : nullptr;
  d->governed = s == p.main_step ? 1u : 0u;
  d->order = st.order;
  d->t_first = ULLONG_MAX;
  d->t_last = 0;
  d->ctas_started = 0;
  d->max_alive = 0;
  d->admit_fail = 0;
  d->evicted = 0;
  d->draining = 0;
  d->tu_alive = 0;
  d->last_live = 0;
  d->topped = 0;
  d->req_idx = i;
  d->has_prev = i > 0 ? 1u : 0u;
  d->qa = st.qa0;
  d->vg_base = 0;
  d->slice = 0;
  if (st.slices > 1) {
    // slice r of a single launch (R-disp-9): VGs [r * slice_vgs, ...) of the
    // same grid; one logical launch (launch_idx 0), one coverage region
    d->slice = r;
    d->vg_base = r * st.slice_vgs;
    d->total = min(st.slice_vgs, st.total - d->vg_base);
    d->launch_idx = 0;
    d->coverage = p.coverage ? p.coverage + st.cov_offset : nullptr;
    d->trace = p.trace ? p.trace + st.cov_offset : nullptr;
  }
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
  d.persistent_fn = reinterpret_cast<const void*>(&accel_persistent<T, false>);
  d.persistent_resolve_fn = reinterpret_cast<const void*>(&accel_persistent<T, true>);
  d.native_fn = reinterpret_cast<const void*>(&accel_native<T>);
  d.topup_fn = reinterpret_cast<const void*>(&accel_topup<T>);
  d.block = accel_dim3{(uint32_t)T::kThreads, 1u, 1u};
  d.dyn_smem = T::kDynSmem;
  d.regs = 0;
  d.chunk = T::kChunk;
  d.args_size = sizeof(typename T::Args);
  d.max_ctas_per_sm = max_ctas_per_sm<T>::value;
  d.slices = slices_of<T>::value;
  if constexpr (has_vg_cost<T>::value)
    d.order_fn = reinterpret_cast<const void*>(&accel_lpt_order<T>);
  else
    d.order_fn = nullptr;
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
    {"stencil_x", &make_desc<StencilX>},
    {"stencil_deep", &make_desc<StencilDeep>},
    {"stencil_z16", &make_desc<StencilZ16>},
    {"stencil2", &make_desc<Stencil2>},
    {"stencil_tma", &make_desc<StencilTma>},
    {"stencil_bulk", &make_desc<StencilBulk>},
    {"histo", &make_desc<Histo>},
    {"histo_wide", &make_desc<HistoWide>},
    {"histo_prescan", &make_desc<HistoPrescan>},
    {"histo_intermediates", &make_desc<HistoIntermediates>},
    {"bfs", &make_desc<Bfs>},
    {"cutcp", &make_desc<Cutcp>},
    {"tpacf", &make_desc<Tpacf>},
    {"spmv", &make_desc<Spmv>},
    {"spmv_v4", &make_desc<SpmvV4>},
    {"sgemm", &make_desc<Sgemm>},
    {"sgemm_split", &make_desc<SgemmSplit>},
    {"sgemm_tc", &make_desc<SgemmTc>},
    {"sgemm_tc1", &make_desc<SgemmTc1>},
    {"lbm", &make_desc<Lbm>},
    {"gridding_binning", &make_desc<GridBinning>},
    {"gridding_scan_l1", &make_desc<GridScanL1>},
    {"gridding_scan_inter", &make_desc<GridScanInter>},
    {"gridding_scan_add", &make_desc<GridScanAdd>},
    {"gridding_reorder", &make_desc<GridReorder>},
    {"gridding_grid", &make_desc<GridGrid>},
    {"sad_4x4", &make_desc<Sad4>},
    {"sad_8x8", &make_desc<Sad8>},
    {"sad_16x16", &make_desc<Sad16>},
    {"mriq_phimag", &make_desc<MriqPhiMag>},
    {"mriq_q", &make_desc<MriqQ>},
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
