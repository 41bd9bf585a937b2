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
    // packed, even bin count: bins 2b and 2b+1 are one 8-B-aligned pair of
    // global counters, flushed with ONE 64-bit atomic (half the L2 atomics:
    // the flush is what an L2-bound co-runner competes with).  A count never
    // reaches 2^32 (n < 2^32), so the low half cannot carry into the high one.
    const bool pair64 = kPacked && (bins & 1u) == 0u;
    for (uint32_t b = threadIdx.x; b < words; b += kThreads) {
      const uint32_t c = h[b];
      if constexpr (kPacked) {
        if (pair64) {
          if (c)
            atomicAdd(reinterpret_cast<unsigned long long*>(gh + 2 * b),
                      ((unsigned long long)(c >> 16) << 32) | (c & 0xffffu));
        } else {
          if (c & 0xffffu) atomicAdd(&gh[2 * b], c & 0xffffu);
          if (c >> 16) atomicAdd(&gh[2 * b + 1], c >> 16);   // bin 2b+1 < bins whenever counted
        }
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

// Parboil histo's first two kernels: the input range and
// the bin-index stream.  Both stream the raw samples with 16-B loads (HBM).
struct HistoPrescan {
  using Args = accel_histo_pre_args;
  static constexpr int kThreads = 256;
  static constexpr uint32_t kChunk = 1;
  static constexpr int kMinBlocks = 6;
  static constexpr uint32_t kDynSmem = 0;
  static __device__ __forceinline__ void body(const Args& a, const VirtualBlock& vb, char*) {
    __shared__ uint32_t s_lo[kThreads / 32], s_hi[kThreads / 32];
    const uint64_t lo0 = (uint64_t)vb.linear * a.per_vg;
    const uint64_t hi0 = lo0 + a.per_vg < a.n ? lo0 + a.per_vg : a.n;
    uint32_t mn = 0xffffffffu, mx = 0u;
    const uint64_t nvec = (hi0 - lo0) / 4;
    const uint4* v = reinterpret_cast<const uint4*>(a.raw + lo0);
    for (uint64_t i = threadIdx.x; i < nvec; i += kThreads) {
      const uint4 w = __ldcs(v + i);
      mn = min(min(mn, w.x), min(w.y, min(w.z, w.w)));
      mx = max(max(mx, w.x), max(w.y, max(w.z, w.w)));
    }
    for (uint64_t i = lo0 + nvec * 4 + threadIdx.x; i < hi0; i += kThreads) {
      mn = min(mn, a.raw[i]);
      mx = max(mx, a.raw[i]);
    }
    mn = __reduce_min_sync(0xffffffffu, mn);
    mx = __reduce_max_sync(0xffffffffu, mx);
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    if (lane == 0) {
      s_lo[warp] = mn;
      s_hi[warp] = mx;
    }
    __syncthreads();
    if (threadIdx.x < 32) {
      mn = lane < kThreads / 32 ? s_lo[lane] : 0xffffffffu;
      mx = lane < kThreads / 32 ? s_hi[lane] : 0u;
      mn = __reduce_min_sync(0xffffffffu, mn);
      mx = __reduce_max_sync(0xffffffffu, mx);
      if (lane == 0) {
        atomicMin(a.lo, mn);
        atomicMax(a.hi, mx);
      }
    }
    __syncthreads();   // s_lo / s_hi are reused by the CTA's next VG
  }
};

struct HistoIntermediates {
  using Args = accel_histo_pre_args;
  static constexpr int kThreads = 256;
  static constexpr uint32_t kChunk = 1;
  static constexpr int kMinBlocks = 6;
  static constexpr uint32_t kDynSmem = 0;
  static __device__ __forceinline__ uint32_t bin(uint32_t x, uint32_t lo, uint64_t span, uint32_t bins) {
    return (uint32_t)(((uint64_t)(x - lo) * bins) / span);
  }
  static __device__ __forceinline__ void body(const Args& a, const VirtualBlock& vb, char*) {
    const uint32_t lo = __ldcg(a.lo), hi = __ldcg(a.hi), bins = a.bins;
    const uint64_t span = (uint64_t)(hi - lo) + 1u;
    const uint64_t lo0 = (uint64_t)vb.linear * a.per_vg;
    const uint64_t hi0 = lo0 + a.per_vg < a.n ? lo0 + a.per_vg : a.n;
    const uint64_t nvec = (hi0 - lo0) / 4;
    const uint4* v = reinterpret_cast<const uint4*>(a.raw + lo0);
    uint4* o = reinterpret_cast<uint4*>(a.bins_out + lo0);
    for (uint64_t i = threadIdx.x; i < nvec; i += kThreads) {
      const uint4 w = __ldcs(v + i);
      o[i] = make_uint4(bin(w.x, lo, span, bins), bin(w.y, lo, span, bins), bin(w.z, lo, span, bins),
                        bin(w.w, lo, span, bins));
    }
    for (uint64_t i = lo0 + nvec * 4 + threadIdx.x; i < hi0; i += kThreads) a.bins_out[i] = bin(a.raw[i], lo, span, bins);
  }
};

using Histo = HistoT<false>;
using HistoWide = HistoT<true>;

}  // namespace accel
