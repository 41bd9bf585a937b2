// mri-gridding -- Parboil "mri-gridding" (§7.2
// lines 853-860 names the Parboil suite): non-Cartesian MRI samples convolved
// onto a G^3 grid with a separable Kaiser-Bessel kernel (definition:
// oracle/tenants.c).  Parboil bins the samples (binning + a radix sort) and
// then grids per output tile; here the same pipeline as six kernels, the six
// steps of one request (R-solver-8, main step = the gridding):
//   binning     cell of every sample, rank by atomicAdd on the cell count
//   scan_l1 / scan_inter / scan_add   exclusive scan of the counts
//   reorder     samples scattered into cell order (SoA)
//   grid        VG = 8x8x8 grid points: the samples of every cell within hw of
//               the tile staged through shared memory (256 at a time), each
//               thread tests them against its 2 points; contributions are
//               the oracle's fp32 op sequence, accumulated in 64-bit fixed
//               point so the result does not depend on the (atomic, hence
//               run-dependent) order of the samples inside a cell.
#pragma once
#include "../device/dispatch.cuh"
#include "accel_tenants.h"

namespace accel {

struct GridBase {
  using Args = accel_gridding_args;
  static constexpr int kThreads = 256;
  static constexpr uint32_t kChunk = 1;
  static constexpr int kMinBlocks = 4;
  static constexpr uint32_t kDynSmem = 0;
  static constexpr uint32_t kPerVG = 1024;
  static __device__ __forceinline__ uint32_t cell_of(const Args& a, float v) {
    const int c = (int)(v / a.cell);
    return (uint32_t)min(max(c, 0), (int)a.cells - 1);
  }
};

struct GridBinning : GridBase {
  static __device__ __forceinline__ void body(const Args& a, const VirtualBlock& vb, char*) {
    const uint32_t nc = a.cells;
    for (uint32_t k = threadIdx.x; k < kPerVG; k += kThreads) {
      const uint32_t i = vb.linear * kPerVG + k;
      if (i >= a.n) break;
      const uint32_t b = (cell_of(a, a.z[i]) * nc + cell_of(a, a.y[i])) * nc + cell_of(a, a.x[i]);
      a.bin[i] = b;
      a.rank[i] = atomicAdd(a.count + b, 1u);
    }
  }
};

// exclusive scan of 1024 values by 256 threads (4 each), returns the total
__device__ __forceinline__ uint32_t block_scan_1024(uint32_t v[4], uint32_t* s_warp) {
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  const uint32_t t0 = v[0], t1 = t0 + v[1], t2 = t1 + v[2], tot = t2 + v[3];
  uint32_t incl = tot;
#pragma unroll
  for (int o = 1; o < 32; o <<= 1) {
    const uint32_t u = __shfl_up_sync(0xffffffffu, incl, o);
    if (lane >= o) incl += u;
  }
  if (lane == 31) s_warp[warp] = incl;
  __syncthreads();
  if (warp == 0) {
    uint32_t w = lane < 8 ? s_warp[lane] : 0u;
#pragma unroll
    for (int o = 1; o < 8; o <<= 1) {
      const uint32_t u = __shfl_up_sync(0xffffffffu, w, o);
      if (lane >= o) w += u;
    }
    if (lane < 8) s_warp[lane] = w;   // inclusive warp totals
  }
  __syncthreads();
  const uint32_t base = (warp ? s_warp[warp - 1] : 0u) + incl - tot;
  const uint32_t total = s_warp[7];
  v[0] = base;
  v[1] = base + t0;
  v[2] = base + t1;
  v[3] = base + t2;
  __syncthreads();   // s_warp reused by the CTA's next VG
  return total;
}

struct GridScanL1 : GridBase {
  static __device__ __forceinline__ void body(const Args& a, const VirtualBlock& vb, char*) {
    __shared__ uint32_t s_warp[8];
    const uint32_t B = a.cells * a.cells * a.cells;
    const uint32_t b0 = vb.linear * kPerVG + 4 * threadIdx.x;
    uint32_t v[4];
#pragma unroll
    for (int k = 0; k < 4; ++k) v[k] = b0 + k < B ? a.count[b0 + k] : 0u;
    const uint32_t total = block_scan_1024(v, s_warp);
#pragma unroll
    for (int k = 0; k < 4; ++k)
      if (b0 + k < B) a.start[b0 + k] = v[k];
    if (threadIdx.x == 0) a.block_sum[vb.linear] = total;
  }
};

struct GridScanInter : GridBase {
  static __device__ __forceinline__ void body(const Args& a, const VirtualBlock&, char*) {
    __shared__ uint32_t s_warp[8];
    const uint32_t B = a.cells * a.cells * a.cells;
    const uint32_t nb = (B + kPerVG - 1) / kPerVG;   // <= 1024
    uint32_t v[4];
#pragma unroll
    for (int k = 0; k < 4; ++k) v[k] = 4 * threadIdx.x + k < nb ? a.block_sum[4 * threadIdx.x + k] : 0u;
    const uint32_t total = block_scan_1024(v, s_warp);
#pragma unroll
    for (int k = 0; k < 4; ++k)
      if (4 * threadIdx.x + k < nb) a.block_sum[4 * threadIdx.x + k] = v[k];
    if (threadIdx.x == 0) a.start[B] = total;
  }
};

struct GridScanAdd : GridBase {
  static __device__ __forceinline__ void body(const Args& a, const VirtualBlock& vb, char*) {
    const uint32_t B = a.cells * a.cells * a.cells;
    const uint32_t off = a.block_sum[vb.linear];
    for (uint32_t k = threadIdx.x; k < kPerVG; k += kThreads) {
      const uint32_t b = vb.linear * kPerVG + k;
      if (b < B) a.start[b] += off;
    }
  }
};

struct GridReorder : GridBase {
  static __device__ __forceinline__ void body(const Args& a, const VirtualBlock& vb, char*) {
    for (uint32_t k = threadIdx.x; k < kPerVG; k += kThreads) {
      const uint32_t i = vb.linear * kPerVG + k;
      if (i >= a.n) break;
      const uint32_t p = a.start[a.bin[i]] + a.rank[i];
      a.sx[p] = a.x[i];
      a.sy[p] = a.y[i];
      a.sz[p] = a.z[i];
      a.sre[p] = a.re[i];
      a.sim[p] = a.im[i];
    }
  }
};

struct GridGrid : GridBase {
  static constexpr int kStage = 256;        // samples staged per round
  static constexpr int kMaxLut = 1024;
  // staged samples (x, y, z, re, im as two float4 rows would waste: SoA) + LUT
  static constexpr uint32_t kDynSmem = 5 * kStage * 4 + kMaxLut * 4;
  static __device__ __forceinline__ long long fx(float v) {   // 2^-30 fixed point
    return __float2ll_rn(v * 1073741824.0f);
  }
  static __device__ __forceinline__ void body(const Args& a, const VirtualBlock& vb, char* smem) {
    float* s_x = reinterpret_cast<float*>(smem);
    float* s_y = s_x + kStage;
    float* s_z = s_y + kStage;
    float* s_re = s_z + kStage;
    float* s_im = s_re + kStage;
    float* s_lut = s_im + kStage;
    const int t = threadIdx.x;
    const uint32_t L = a.L, G = a.G, nc = a.cells;
    for (uint32_t k = t; k < L; k += kThreads) s_lut[k] = a.lut[k];
    const float hw = a.hw, ks = (float)(L - 1) / hw;
    const int gx0 = 8 * (int)vb.x, gy0 = 8 * (int)vb.y, gz0 = 8 * (int)vb.z;
    const float px = (float)(gx0 + (t & 7)), py = (float)(gy0 + ((t >> 3) & 7));
    const float pz0 = (float)(gz0 + (t >> 6)), pz1 = pz0 + 4.0f;
    long long ar0 = 0, ai0 = 0, ar1 = 0, ai1 = 0;
    // cells within hw of the tile [g0, g0 + 7]
    auto crange = [&](int g0, int& c0, int& c1) {
      c0 = max(0, (int)floorf(((float)g0 - hw) / a.cell));
      c1 = min((int)nc - 1, (int)floorf(((float)(g0 + 7) + hw) / a.cell));
    };
    int cx0, cx1, cy0, cy1, cz0, cz1;
    crange(gx0, cx0, cx1);
    crange(gy0, cy0, cy1);
    crange(gz0, cz0, cz1);
    __syncthreads();   // LUT staged
    for (int cz = cz0; cz <= cz1; ++cz)
      for (int cy = cy0; cy <= cy1; ++cy) {
        // the cells (cx0..cx1, cy, cz) are one contiguous run of samples
        const uint32_t row = (uint32_t)(cz * (int)nc + cy) * nc;
        const uint32_t s0 = a.start[row + cx0], s1 = a.start[row + cx1 + 1];
        for (uint32_t base = s0; base < s1; base += kStage) {
          const uint32_t cnt = min((uint32_t)kStage, s1 - base);
          __syncthreads();
          if ((uint32_t)t < cnt) {
            s_x[t] = a.sx[base + t];
            s_y[t] = a.sy[base + t];
            s_z[t] = a.sz[base + t];
            s_re[t] = a.sre[base + t];
            s_im[t] = a.sim[base + t];
          }
          __syncthreads();
          for (uint32_t q = 0; q < cnt; ++q) {
            const float dx = fabsf(px - s_x[q]), dy = fabsf(py - s_y[q]);
            if (dx < hw && dy < hw) {
              const float wxy = __fmul_rn(s_lut[(int)__fmul_rn(dx, ks)], s_lut[(int)__fmul_rn(dy, ks)]);
              const float sz = s_z[q], re = s_re[q], im = s_im[q];
              const float dz0 = fabsf(pz0 - sz), dz1 = fabsf(pz1 - sz);
              if (dz0 < hw) {
                const float w = __fmul_rn(wxy, s_lut[(int)__fmul_rn(dz0, ks)]);
                ar0 += fx(__fmul_rn(w, re));
                ai0 += fx(__fmul_rn(w, im));
              }
              if (dz1 < hw) {
                const float w = __fmul_rn(wxy, s_lut[(int)__fmul_rn(dz1, ks)]);
                ar1 += fx(__fmul_rn(w, re));
                ai1 += fx(__fmul_rn(w, im));
              }
            }
          }
        }
      }
    const int ix = gx0 + (t & 7), iy = gy0 + ((t >> 3) & 7), iz0 = gz0 + (t >> 6);
    if (ix < (int)G && iy < (int)G) {
      const double sc = 1.0 / 1073741824.0;
      if (iz0 < (int)G) {
        const size_t p = ((size_t)iz0 * G + iy) * G + ix;
        reinterpret_cast<float2*>(a.grid)[p] = make_float2((float)(ar0 * sc), (float)(ai0 * sc));
      }
      if (iz0 + 4 < (int)G) {
        const size_t p = ((size_t)(iz0 + 4) * G + iy) * G + ix;
        reinterpret_cast<float2*>(a.grid)[p] = make_float2((float)(ar1 * sc), (float)(ai1 * sc));
      }
    }
  }
};

}  // namespace accel
