// bfs -- level-synchronous top-down breadth-first search (Parboil "bfs",
// PAPER.md lines 290-298, 978, 1131-1133) on a directed CSR graph.
//
// Launch l expands frontier level l: VG v owns frontier entries
// [256 v, 256 v + 256); a thread claims each unvisited neighbour with
// atomicCAS(level, -1, l+1) (the winner is unique, so level[] is the same
// whatever the interleaving) and appends it to a per-CTA shared-memory queue;
// the queue is published with ONE global atomicAdd per VG and a coalesced copy
// into the next frontier.  The frontier size lives on the device (count[l]):
// native CTAs past it return at once, persistent CTAs read it as their
// dynamic total -- no host round trip between levels.
#pragma once
#include "../device/dispatch.cuh"
#include "accel_tenants.h"

namespace accel {

struct Bfs {
  using Args = accel_bfs_args;
  static constexpr int kThreads = 256;
  static constexpr uint32_t kChunk = 1;
  static constexpr int kMinBlocks = 6;
  // useful occupancy in a mix (R-solver-10): 0.374 ms at 2 CTAs/SM, 0.373 at
  // 3, 0.42 at 6 (more CTAs only add queue-append contention on the small
  // levels; scripts/occ_scaling.py)
  static constexpr uint32_t kMaxCtasPerSm = 2;
  static constexpr uint32_t kQueueCap = 4096;  // local queue entries (16 KB)
  static constexpr uint32_t kDynSmem = kQueueCap * sizeof(int32_t);
  static constexpr bool kDynamicTotal = true;

  static __device__ __forceinline__ uint32_t frontier_size(const Args& a, uint32_t l) {
    return l == 0 ? 1u : ld_volatile(a.count + l);
  }
  static __device__ __forceinline__ uint32_t dynamic_total(const Args& a, uint32_t l) {
    return (frontier_size(a, l) + kThreads - 1) / kThreads;
  }

  static __device__ __forceinline__ void body(const Args& a, const VirtualBlock& vb, char* smem) {
    __shared__ uint32_t s_n, s_base;
    int32_t* q = reinterpret_cast<int32_t*>(smem);
    const uint32_t l = vb.launch_idx;
    const uint32_t nv = a.nv;
    const int32_t* fin = a.frontier + (size_t)(l & 1u) * nv;
    int32_t* fout = a.frontier + (size_t)((l + 1u) & 1u) * nv;
    uint32_t* next_count = a.count + l + 1;
    if (threadIdx.x == 0) s_n = 0;
    __syncthreads();
    const uint32_t f = frontier_size(a, l);
    const uint32_t i = vb.linear * kThreads + threadIdx.x;
    if (i < f) {
      int32_t u;
      if (l == 0) {
        u = (int32_t)a.src;
        a.level[u] = 0;
      } else {
        u = __ldcg(fin + i);
      }
      const uint32_t e0 = __ldg(a.row_ptr + u), e1 = __ldg(a.row_ptr + u + 1);
      const int32_t nl = (int32_t)l + 1;
      for (uint32_t e = e0; e < e1; ++e) {
        const int32_t w = __ldg(a.col + e);
        if (__ldcg(a.level + w) == -1 && atomicCAS(a.level + w, -1, nl) == -1) {
          const uint32_t p = atomicAdd(&s_n, 1u);
          if (p < kQueueCap) {
            q[p] = w;
          } else {  // overflow: publish directly
            fout[atomicAdd(next_count, 1u)] = w;
          }
        }
      }
    }
    __syncthreads();
    const uint32_t n = min(s_n, kQueueCap);
    if (threadIdx.x == 0 && n) s_base = atomicAdd(next_count, n);
    __syncthreads();
    for (uint32_t j = threadIdx.x; j < n; j += kThreads) fout[s_base + j] = q[j];
  }
};

}  // namespace accel
