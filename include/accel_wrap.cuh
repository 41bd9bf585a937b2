/*
 * accel_wrap.cuh -- transparent accelOS sharing for an application's own
 * kernels (§4 lines 558-563 and §5:
 * the paper's ProxyCL intercepts an unmodified application's kernel launches
 * and its JIT rewrites the kernel into the scheduling form).
 *
 * B200 design: no JIT.  The application writes its kernel body once, as a
 * tenant struct (the contract of csrc/device/dispatch.cuh: Args, kThreads,
 * kChunk, kDynSmem, body(const Args&, const VirtualBlock&, char* smem)), and
 * declares its ORIGINAL kernel with
 *
 *     ACCEL_WRAP_KERNEL(my_kernel, MyTenant)
 *
 * which defines  __global__ void my_kernel(MyTenant::Args)  -- the plain
 * kernel over the original grid, what the application launches with
 * my_kernel<<<grid, MyTenant::kThreads, MyTenant::kDynSmem, stream>>>(args) --
 * and, compiled into the same binary, the persistent (scheduling) forms of the
 * same body.  A static initialiser offers the pair to
 * accel_intercept_register(), a WEAK symbol: without the interception shim it
 * is absent and the application runs natively; with
 *
 *     LD_PRELOAD=.../libaccel_intercept.so ./app
 *
 * the shim's cudaLaunchKernel redirects every launch of a registered kernel to
 * a SHARED-mode accelOS request (persistent CTAs, fair quotas, ordered with the
 * application's stream) and passes every other launch through unchanged.
 * The application must link the CUDA runtime dynamically (nvcc -cudart shared)
 * so that the shim can interpose it.
 */
#ifndef ACCEL_WRAP_CUH_
#define ACCEL_WRAP_CUH_

#include "accel.h"
#include "../paper_conf_cgo_margiolaso16_b200/csrc/device/dispatch.cuh"

extern "C" {
/* Provided by libaccel_intercept.so (weak here: absent = run natively).
 * original_fn: host stub of the application's kernel; d: its scheduling forms. */
int accel_intercept_register(const void *original_fn, const accel_kernel_desc *d) __attribute__((weak));
}

namespace accel {

// The original kernel's body: one CTA per VG over the hardware grid.
template <class T>
__device__ __forceinline__ void original_body(const typename T::Args& a) {
  extern __shared__ __align__(128) char smem[];
  VirtualBlock vb;
  vb.x = blockIdx.x; vb.y = blockIdx.y; vb.z = blockIdx.z;
  vb.gx = gridDim.x; vb.gy = gridDim.y; vb.gz = gridDim.z;
  vb.linear = blockIdx.x + gridDim.x * (blockIdx.y + gridDim.y * blockIdx.z);
  vb.launch_idx = 0;
  T::body(a, vb, smem);
}

template <class T>
inline int wrap_register(const void* original_fn, const char* name) {
  if (accel_intercept_register == nullptr) return 0;   // no shim: native
  accel_kernel_desc d{};
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
  if constexpr (has_vg_cost<T>::value)
    d.order_fn = reinterpret_cast<const void*>(&accel_lpt_order<T>);
  else
    d.order_fn = nullptr;
  return accel_intercept_register(original_fn, &d);
}

}  // namespace accel

#define ACCEL_WRAP_KERNEL(name, T)                                                                  \
  __global__ void __launch_bounds__(T::kThreads, ::accel::min_blocks<T>::value)                   \
      name(const __grid_constant__ typename T::Args a) {                                          \
    ::accel::original_body<T>(a);                                                                   \
  }                                                                                                 \
  static const int name##_accel_registered =                                                        \
      ::accel::wrap_register<T>(reinterpret_cast<const void*>(&name), #name);

#endif /* ACCEL_WRAP_CUH_ */
