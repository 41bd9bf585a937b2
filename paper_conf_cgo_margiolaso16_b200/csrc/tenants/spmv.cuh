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

}  // namespace accel
