// tpacf -- two-point angular correlation histograms (Parboil "tpacf",
// PAPER.md lines 290-298, 1132).
//
// VG (x, y): 256 points i of block x from set P against every point j of set
// Q; y = 0 -> DD (P = Q = data, pairs i < j), y = 1..S -> RR of random set
// y-1 (i < j), y = S+1..2S -> DR (data x random set y-S-1, all pairs).  Q is
// staged through shared memory in tiles of 256 points (broadcast reads).  The
// angular bin of a pair is decided on the fp32 dot product
// (x*x' + y*y') + z*z' (round-to-nearest, no FMA, DESIGN.md R-fp-1) by a
// binary search over the descending bin edges; each lane counts into its own
// shared-memory sub-histogram column (bank = lane, conflict-free) with one
// shared-memory RED.ADD per pair (TPACF_REDS=0: load + add + store); the VG
// ends with one 64-bit global atomic per bin.  Integer result: bit-exact.
#pragma once
#include "../device/dispatch.cuh"
#include "accel_tenants.h"

#ifndef TPACF_REDS
#define TPACF_REDS 1
#endif
#ifndef TPACF_UNROLL2
#define TPACF_UNROLL2 1
#endif
#ifndef TPACF_LUT
#define TPACF_LUT 1
#endif

namespace accel {

struct Tpacf {
  using Args = accel_tpacf_args;
  static constexpr int kThreads = 256;
  static constexpr uint32_t kChunk = 1;
  static constexpr bool kSpread = true;     // VG cost varies in space (dispatch.cuh)
  static constexpr int kMinBlocks = 6;   // <= 40 regs: smem allows 6 CTAs/SM
  static constexpr uint32_t kMaxCtasPerSm = 3;   // in a mix: 1.414 ms at 3 CTAs/SM vs 1.40 at 6 (occ_scaling.py)
  static constexpr int kWarps = kThreads / 32;
  static constexpr int kMaxBins = 32;      // nedges + 1 <= 32
  static constexpr int kTile = 256;
  // [warp][bin][lane] u32 counters + Q tile (256 float4: x, y, z, pad; one
  // LDS.128 per pair) + edges (32)
  // + the exponent table (30 float4, below; 6 CTAs/SM still fit)
  static constexpr int kLut = 30;
  static constexpr uint32_t kDynSmem = kWarps * kMaxBins * 32 * sizeof(uint32_t) + kTile * sizeof(float4) +
                                       32 * sizeof(float) + kLut * sizeof(float4);

  // Dequeue-order cost model (dispatch.cuh accel_lpt_order): Q tiles the VG
  // walks -- DD / RR blocks (y <= S) start at their diagonal tile, DR blocks
  // (y > S) walk all of them.
  // Q tiles [t0, t1) of VG vb: part vb.z of the run that starts at the
  // diagonal tile (DD / RR: pairs i < j) or at tile 0 (DR)
  static __device__ __forceinline__ void tile_range(const Args& a, const VirtualBlock& vb, uint32_t& t0,
                                                    uint32_t& t1) {
    const uint32_t ntiles = (a.npts + kTile - 1) / kTile;
    const uint32_t first = vb.y <= a.nsets ? vb.x : 0u;
    const uint32_t len = ntiles - first, parts = vb.gz;
    t0 = first + (uint32_t)(((uint64_t)len * vb.z) / parts);
    t1 = first + (uint32_t)(((uint64_t)len * (vb.z + 1)) / parts);
  }

  static __device__ float vg_cost(const Args& a, const VirtualBlock& vb) {
    uint32_t t0, t1;
    tile_range(a, vb, t0, t1);
    // the diagonal tile holds half its pairs
    return (float)(t1 - t0) - ((vb.y <= a.nsets && t0 == vb.x && t1 > t0) ? 0.5f : 0.f);
  }

  static __device__ __forceinline__ void body(const Args& a, const VirtualBlock& vb, char* smem) {
    uint32_t* hist = reinterpret_cast<uint32_t*>(smem);
    float4* qt = reinterpret_cast<float4*>(hist + kWarps * kMaxBins * 32);   // 16-B aligned (32 KB of counters)
    float* edges = reinterpret_cast<float*>(qt + kTile);
    const int t = threadIdx.x, lane = t & 31, warp = t >> 5;
    const uint32_t n = a.npts, S = a.nsets, ne = a.nedges;
    const uint32_t s = vb.y;
    const float* P;
    const float* Q;
    unsigned long long* out;
    bool upper;
    if (s == 0) {
      P = Q = a.data;
      out = a.dd;
      upper = true;
    } else if (s <= S) {
      P = Q = a.rand + (size_t)(s - 1) * 3 * n;
      out = a.rr;
      upper = true;
    } else {
      P = a.data;
      Q = a.rand + (size_t)(s - S - 1) * 3 * n;
      out = a.dr;
      upper = false;
    }
    for (int b = t; b < kWarps * kMaxBins * 32; b += kThreads) hist[b] = 0u;
    if (t < 32) edges[t] = t < (int)ne ? __ldg(a.binb + t) : -3.0f;  // pad: never > d
    const uint32_t i = vb.x * kTile + t;
    const bool have = i < n;
    const float ix = have ? __ldg(P + i) : 0.f, iy = have ? __ldg(P + n + i) : 0.f,
                iz = have ? __ldg(P + 2 * n + i) : 0.f;
    uint32_t* myh = hist + warp * kMaxBins * 32 + lane;
    __syncthreads();   // edges staged
    // Exponent table (exact): u = 1 - d in fp32 is monotone in d, so the
    // (clamped) exponent field of u orders d against every edge whose
    // u-exponent cell differs; only the (at most two) edges sharing d's cell
    // need a compare.  Cell c in 0..28 = exponent field min(max(e, 102), 130)
    // - 102 (u = 0, i.e. d = 1, and u < 2^-24 fall in cell 0; fp32 d has no
    // value strictly between), cell 29 = u < 0 (d > 1).  Entry c = (edges in
    // lower cells -- all greater than d --, candidate 1, candidate 2).  The
    // bins are log-spaced in angle, so consecutive edges are more than an
    // octave apart in u; an input with three edges in one cell falls back to
    // the binary search.
    float4* lut = reinterpret_cast<float4*>(edges + 32);
    auto cell_of = [](uint32_t ub) {
      return (ub >> 31) ? kLut - 1 : min(max((int)(ub >> 23), 102), 130) - 102;
    };
    bool crowded = false;
    if (TPACF_LUT && t < kLut) {
      int base = 0, nc = 0;
      float c1 = -3.0f, c2 = -3.0f;
      for (uint32_t k = 0; k < ne; ++k) {
        const float e = edges[k];
        const int ce = cell_of(__float_as_uint(__fsub_rn(1.0f, e)));
        // an edge above 1 (cell 29) exceeds every d <= 1
        const bool lower = t < kLut - 1 && (ce < t || ce == kLut - 1);
        if (lower) ++base;
        if (ce == t) {
          if (nc == 0) c1 = e; else c2 = e;
          ++nc;
        }
      }
      crowded = nc > 2;
      lut[t] = make_float4(__int_as_float(base), c1, c2, 0.f);
    }
    const bool use_lut = TPACF_LUT && !__syncthreads_or(crowded);
    const float e7 = edges[7], e15 = edges[15], e23 = edges[23];
    uint32_t tile0, tile1;
    tile_range(a, vb, tile0, tile1);
    for (uint32_t jt = tile0 * kTile; jt < tile1 * kTile; jt += kTile) {
      __syncthreads();
      const uint32_t jj = jt + t;
      if (jj < n) qt[t] = make_float4(__ldg(Q + jj), __ldg(Q + n + jj), __ldg(Q + 2 * n + jj), 0.f);
      __syncthreads();
      if (!have) continue;
      const uint32_t cnt = min((uint32_t)kTile, n - jt);
      // pairs i < j on the diagonal tile start after i
      const uint32_t q0 = (upper && jt == vb.x * kTile) ? (uint32_t)t + 1 : 0u;
      // bin = #{k : d < edges[k]}: the exponent table, else a binary search
      // over the descending edges, its first two levels from registers
      // (edges[15], then edges[7] / [23])
      auto bin_lut = [&](float d) {
        const float4 L = lut[cell_of(__float_as_uint(__fsub_rn(1.0f, d)))];
        return __float_as_int(L.x) + (d < L.y ? 1 : 0) + (d < L.z ? 1 : 0);
      };
      auto bin_search = [&](float d) {
        int m = (e15 > d) ? 16 : 0;
        if (((m != 0) ? e23 : e7) > d) m += 8;
#pragma unroll
        for (int step = 4; step >= 1; step >>= 1)
          if (edges[m + step - 1] > d) m += step;
        return m;
      };
      auto dot = [&](const float4& qv) {
        return __fadd_rn(__fadd_rn(__fmul_rn(ix, qv.x), __fmul_rn(iy, qv.y)), __fmul_rn(iz, qv.z));
      };
      auto count = [&](int m) {
#if TPACF_REDS
        // lane-private counter (bank = lane): one RED.ADD on shared memory
        // instead of load + add + store
        atomicAdd(myh + m * 32, 1u);
#else
        myh[m * 32] += 1u;
#endif
      };
      uint32_t q = q0;
      if (use_lut) {
        for (; q + 1 < cnt; q += 2) {
          const int m0 = bin_lut(dot(qt[q])), m1 = bin_lut(dot(qt[q + 1]));
          count(m0);
          count(m1);
        }
        for (; q < cnt; ++q) count(bin_lut(dot(qt[q])));
      } else {
#if TPACF_UNROLL2
        // two independent search chains in flight (their shared-memory edge
        // loads overlap)
        for (; q + 1 < cnt; q += 2) {
          const int m0 = bin_search(dot(qt[q])), m1 = bin_search(dot(qt[q + 1]));
          count(m0);
          count(m1);
        }
#endif
        for (; q < cnt; ++q) count(bin_search(dot(qt[q])));
      }
    }
    __syncthreads();
    if (t < (int)ne + 1) {
      unsigned long long tot = 0;
      for (int w = 0; w < kWarps; ++w)
        for (int l = 0; l < 32; ++l) tot += hist[(w * kMaxBins + t) * 32 + l];
      if (tot) atomicAdd(out + t, tot);
    }
  }
};

}  // namespace accel
