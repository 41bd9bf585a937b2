// spmv -- y = A x with A in CSR, fp32 (Parboil "spmv").
//
// One VG = 64 consecutive rows; 256 threads = 4 threads per row.  The 4 lanes
// of a row read consecutive non-zeros (coalesced col/val stream, the dominant
// traffic: 8 B per non-zero), gather x through L1/L2, and combine with two
// shuffles in a fixed order, so the result is deterministic and identical in
// both modes.  HBM-bound in principle; at the default size (31 MB per SpMV)
// the matrix stays L2-resident across the repeated launches.
#pragma once
#include "../device/dispatch.cuh"
#include "accel_tenants.h"

namespace accel {

struct Spmv {
  using Args = accel_spmv_args;
  static constexpr int kThreads = 256;
  static constexpr int kRows = 64;
  static constexpr int kLanesPerRow = kThreads / kRows;  // 4
  static constexpr uint32_t kChunk = 1;
  static constexpr int kMinBlocks = 6;
  static constexpr uint32_t kMaxCtasPerSm = 4;   // in a mix: 1.21 ms at 4 CTAs/SM vs 1.26 at 6 (occ_scaling.py)
  static constexpr uint32_t kDynSmem = 0;

  static __device__ __forceinline__ void body(const Args& a, const VirtualBlock& vb, char*) {
    const int t = threadIdx.x;
    const int row = (int)vb.linear * kRows + t / kLanesPerRow;
    const int sub = t % kLanesPerRow;
    float s = 0.f;
    if (row < (int)a.n) {
      const int k0 = __ldg(a.row_ptr + row), k1 = __ldg(a.row_ptr + row + 1);
      for (int k = k0 + sub; k < k1; k += kLanesPerRow)
        s = fmaf(__ldg(a.val + k), __ldg(a.x + __ldg(a.col + k)), s);
    }
    s += __shfl_xor_sync(0xffffffffu, s, 1);
    s += __shfl_xor_sync(0xffffffffu, s, 2);
    if (row < (int)a.n && sub == 0) a.y[row] = s;
  }
};

// spmv_v4 -- the same product with 128-bit col/val loads (north star: "128-bit
// HBM access").  The non-zeros are read in aligned 4-element chunks: the 4
// lanes of a row take the chunks floor(k0/4) .. floor((k1-1)/4) round-robin,
// one LDG.128 of val and one of col each, and add the chunk's in-row
// elements in k order.  col/val must be 16-B aligned and readable up to a
// multiple of 4 elements (SpmvJob pads them).  Fixed lane/chunk assignment
// and reduction order: deterministic, identical in both modes (the order
// differs from "spmv", so the two kernels agree to rounding, not bitwise).
struct SpmvV4 {
  using Args = accel_spmv_args;
  static constexpr int kThreads = 256;
  static constexpr int kRows = 64;                       // (128 rows / 2 lanes: native 1.94 ms)
  static constexpr int kLanesPerRow = kThreads / kRows;  // 4
  static constexpr uint32_t kChunk = 1;
  static constexpr int kMinBlocks = 6;
  static constexpr uint32_t kMaxCtasPerSm = 4;
  static constexpr uint32_t kDynSmem = 0;

  static __device__ __forceinline__ void body(const Args& a, const VirtualBlock& vb, char*) {
    const int t = threadIdx.x;
    const int row = (int)vb.linear * kRows + t / kLanesPerRow;
    const int sub = t % kLanesPerRow;
    float s = 0.f;
    if (row < (int)a.n) {
      const int k0 = __ldg(a.row_ptr + row), k1 = __ldg(a.row_ptr + row + 1);
      const float4* __restrict__ v4 = reinterpret_cast<const float4*>(a.val);
      const int4* __restrict__ c4 = reinterpret_cast<const int4*>(a.col);
      const int cend = (k1 + 3) >> 2;
      for (int c = (k0 >> 2) + sub; c < cend; c += kLanesPerRow) {
        const float4 v = __ldg(v4 + c);
        const int4 cc = __ldg(c4 + c);
        const int kb = c << 2;
        if (kb + 0 >= k0 && kb + 0 < k1) s = fmaf(v.x, __ldg(a.x + cc.x), s);
        if (kb + 1 >= k0 && kb + 1 < k1) s = fmaf(v.y, __ldg(a.x + cc.y), s);
        if (kb + 2 >= k0 && kb + 2 < k1) s = fmaf(v.z, __ldg(a.x + cc.z), s);
        if (kb + 3 >= k0 && kb + 3 < k1) s = fmaf(v.w, __ldg(a.x + cc.w), s);
      }
    }
#pragma unroll
    for (int o = 1; o < kLanesPerRow; o <<= 1) s += __shfl_xor_sync(0xffffffffu, s, o);
    if (row < (int)a.n && sub == 0) a.y[row] = s;
  }
};

}  // namespace accel
