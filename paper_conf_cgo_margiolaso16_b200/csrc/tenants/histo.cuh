// histo -- saturating histogram (Parboil "histo" main + final fused; PAPER.md
// names "histo final" / "hist inter" at line 979).
//
// One VG = `per_vg` samples read with 16-B vector loads (coalesced, HBM-bound),
// counted into a shared-memory private histogram with shared atomics, then
// flushed (non-zero bins only) with global atomics into hist[r&1].  The VG that
// completes launch r (done[r] counter, threadfence reduction) runs the "final"
// step: sat[b] = min(hist, 255), and zeroes the other half of hist for the
// next launch.  No cross-CTA waiting: the last finisher does the tail work.
//
// Two instantiations (up to 16,384 bins at the B200 default):
//   histo       u32 private counters, <= 4,096 bins, 16 KB smem
//   histo_wide  16-bit private counters packed two per word (bin b in the
//               half b & 1 of word b >> 1: a shared-memory add of 1 << 16
//               never carries into the other half while a VG counts fewer
//               than 65,536 samples), <= 16,384 bins in 32 KB smem, u32
//               samples only.
#pragma once
#include "../device/dispatch.cuh"
#include "accel_tenants.h"

namespace accel {

template <bool kPacked>
struct HistoT {
  using Args = accel_histo_args;
  static constexpr int kThreads = 256;
  static constexpr uint32_t kChunk = 1;
  static constexpr int kMinBlocks = 6;    // <= 40 regs in both modes
  static constexpr uint32_t kMaxBins = kPacked ? 16384 : 4096;
  static constexpr uint32_t kWords = kPacked ? kMaxBins / 2 : kMaxBins;
  static constexpr uint32_t kDynSmem = kWords * sizeof(uint32_t);  // 16 / 32 KB

  static __device__ __forceinline__ void count4(uint32_t* h, uint32_t w, uint32_t sb) {
    if constexpr (kPacked) {
      atomicAdd(&h[w >> 1], 1u << ((w & 1u) << 4));
    } else if (sb == 1) {
#pragma unroll
      for (int k = 0; k < 4; ++k) atomicAdd(&h[(w >> (8 * k)) & 0xffu], 1u);
    } else {
      atomicAdd(&h[w], 1u);
    }
  }

  static __device__ __forceinline__ void body(const Args& a, const VirtualBlock& vb, char* smem) {
    uint32_t* h = reinterpret_cast<uint32_t*>(smem);
    __shared__ bool s_last;
    const uint32_t bins = a.bins;
    const uint32_t words = kPacked ? (bins + 1u) >> 1 : bins;
    const uint32_t r = vb.launch_idx;
    for (uint32_t b = threadIdx.x; b < words; b += kThreads) h[b] = 0u;
    __syncthreads();

    const uint32_t sb = a.sample_bytes;
    const uint64_t lo = (uint64_t)vb.linear * a.per_vg;
    const uint64_t hi = (lo + a.per_vg < (uint64_t)a.n) ? lo + a.per_vg : (uint64_t)a.n;
    const char* base = reinterpret_cast<const char*>(a.samples);
    // 16-B vectors fully inside [lo, hi): per_vg is a multiple of 4096 so lo
    // is 16-B aligned for both sample sizes.
    const uint64_t per_vec = 16 / sb;
    const uint64_t nvec = (hi - lo) / per_vec;
    const uint4* v = reinterpret_cast<const uint4*>(base + lo * sb);
    // four independent 16-B loads in flight per thread before counting
    uint64_t i = threadIdx.x;
    for (; i + 3 * kThreads < nvec; i += 4 * kThreads) {
      uint4 w[4];
#pragma unroll
      for (int u = 0; u < 4; ++u) w[u] = __ldcs(v + i + u * kThreads);  // streamed once
#pragma unroll
      for (int u = 0; u < 4; ++u) {
        count4(h, w[u].x, sb);
        count4(h, w[u].y, sb);
        count4(h, w[u].z, sb);
        count4(h, w[u].w, sb);
      }
    }
    for (; i < nvec; i += kThreads) {
      const uint4 w = __ldcs(v + i);
      count4(h, w.x, sb);
      count4(h, w.y, sb);
      count4(h, w.z, sb);
      count4(h, w.w, sb);
    }
    for (uint64_t i = lo + nvec * per_vec + threadIdx.x; i < hi; i += kThreads) {
      const uint32_t s = sb == 1 ? (uint32_t)reinterpret_cast<const uint8_t*>(base)[i]
                                 : reinterpret_cast<const uint32_t*>(base)[i];
      if constexpr (kPacked)
        atomicAdd(&h[s >> 1], 1u << ((s & 1u) << 4));
      else
        atomicAdd(&h[s], 1u);
    }
    __syncthreads();
    uint32_t* gh = a.hist + (r & 1u) * bins;
    for (uint32_t b = threadIdx.x; b < words; b += kThreads) {
      const uint32_t c = h[b];
      if constexpr (kPacked) {
        if (c & 0xffffu) atomicAdd(&gh[2 * b], c & 0xffffu);
        if (c >> 16) atomicAdd(&gh[2 * b + 1], c >> 16);   // bin 2b+1 < bins whenever counted
      } else {
        if (c) atomicAdd(&gh[b], c);
      }
    }
    // final step by the VG that completes launch r
    __threadfence();
    __syncthreads();
    if (threadIdx.x == 0) {
      const uint32_t nvg = vb.gx * vb.gy * vb.gz;
      s_last = atomicAdd(&a.done[r], 1u) == nvg - 1;
    }
    __syncthreads();
    if (s_last) {
      __threadfence();
      uint32_t* other = a.hist + ((r + 1u) & 1u) * bins;
      for (uint32_t b = threadIdx.x; b < bins; b += kThreads) {
        const uint32_t c = __ldcg(gh + b);
        a.sat[b] = (uint8_t)(c > 255u ? 255u : c);
        other[b] = 0u;
      }
    }
  }
};

using Histo = HistoT<false>;
using HistoWide = HistoT<true>;

}  // namespace accel
