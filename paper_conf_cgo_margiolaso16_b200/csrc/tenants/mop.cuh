// mop -- the example kernel of PAPER.md Fig. 8a (lines 735-746): each work-item
// adds or subtracts two buffers depending on its GROUP id, so any error in the
// virtual-id substitution (Fig. 8b lines 5-6: rt_global_id / rt_group_id)
// changes the output.
#pragma once
#include "../device/dispatch.cuh"
#include "accel_tenants.h"

namespace accel {

struct Mop {
  using Args = accel_mop_args;
  static constexpr int kThreads = 256;
  static constexpr uint32_t kChunk = 8;   // tiny body: 8 VGs per dequeue (§6.4, < 10 instrs)
  static constexpr int kMinBlocks = 8;    // full occupancy (<= 32 regs) in both modes
  static constexpr uint32_t kDynSmem = 0;
  static __device__ __forceinline__ void body(const Args& a, const VirtualBlock& vb, char*) {
    const uint32_t grid = vb.x;                               // get_group_id(0)
    const uint32_t gid = vb.x * kThreads + threadIdx.x;       // get_global_id(0)
    if (gid >= a.n) return;
    const float x = a.ina[gid], y = a.inb[gid];
    a.out[gid] = grid < a.nconst ? x + y : x - y;
  }
};

}  // namespace accel
