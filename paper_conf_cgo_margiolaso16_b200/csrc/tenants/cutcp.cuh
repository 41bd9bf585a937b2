// cutcp -- cutoff Coulombic potential on a 3-D lattice (Parboil "cutcp",
// PAPER.md lines 290-291, 978).
//
// One VG = 8 x 8 x 8 lattice points; 128 threads, thread t owns the column
// (i, j) = (t % 8, (t / 8) % 8) and 4 consecutive k.  Atoms arrive binned in
// cells (x fastest); a row of cells along x is one contiguous atom range, so
// the VG walks the (y, z) cell rows whose distance to the VG box is < cutoff,
// trims each row's x-range to the sphere, stages the atoms in shared memory
// (128 float4 per tile) and every thread tests them against its 4 points.
// The rows' ranges are found 128 at a time in parallel and the tile is
// gathered one atom per thread (CUTCP_GATHER), so small cells cost no
// per-row latency (1-A cells: 25 % faster alone).
// Membership r^2 < c^2 and the exclusion r^2 < e^2 are decided on the fp32
// value ((dx*dx + dy*dy) + dz*dz, round-to-nearest, no FMA) exactly like the
// oracle (DESIGN.md R-fp-1); the term q/r (1 - r^2/c^2)^2 is fp32.
// FP32-ALU bound (+ MUFU rsqrt for in-range pairs).
#pragma once
#include "../device/dispatch.cuh"
#include "accel_tenants.h"

namespace accel {

struct Cutcp {
  using Args = accel_cutcp_args;
  static constexpr int kThreads = 128;
  static constexpr uint32_t kChunk = 1;
// 9 resident CTAs/SM caps the body at 56 registers (no spills; 62
// uncapped).  Registers are cutcp's dominant resource, so its equal share
// holds 21 % more CTAs.  Measured with the branchy loop before the ftz/min
// change: C2 unfairness 2.03-2.09 -> 1.86-1.94 at 1.07x native throughput,
// isolated dispatch overhead 9.5 -> 7.6 %; at 10/SM (48 registers) U 1.70-1.81
// but the isolated persistent run lost 18 % to its tail (DESIGN.md section 6,
// profiles/round1_cutcp_regcap.log).
#ifndef CUTCP_MINB
#define CUTCP_MINB 9
#endif
  // in a mix (R-solver-10): 1.195 ms at 4 CTAs/SM = 98 % of the 1.17 ms at 6
  static constexpr uint32_t kMaxCtasPerSm = 4;
  static constexpr int kMinBlocks = CUTCP_MINB;
  static constexpr int kTile = 128;  // atoms staged per round
  static constexpr int kPts = 4;     // points per thread along z
#ifndef CUTCP_GATHER
#define CUTCP_GATHER 1
#endif
  // tile + (CUTCP_GATHER) per-batch row starts, prefix sums and warp totals
  static constexpr uint32_t kDynSmem =
      kTile * sizeof(float4) + (CUTCP_GATHER ? (2 * kThreads + 1 + kThreads / 32) * sizeof(int) : 0);

  // MUFU.RSQ without the denormal rescaling rsqrtf() wraps around it (4
  // instructions per in-range pair): r^2 < 2^-126 only occurs for excluded
  // points (r^2 < e^2), whose output is 0 whatever the sum.
  static __device__ __forceinline__ float rsqrt_ftz(float x) {
    float y;
    asm("rsqrt.approx.ftz.f32 %0, %1;" : "=f"(y) : "f"(x));
    return y;
  }

  static __device__ __forceinline__ float gap(float lo, float hi, float clo, float chi) {
    // distance between intervals [lo, hi] and [clo, chi]
    return fmaxf(0.f, fmaxf(clo - hi, lo - chi));
  }

  // Dequeue-order cost model (dispatch.cuh accel_lpt_order): the atoms the
  // body streams for this VG -- the same cell rows and trimmed x-ranges, in
  // the same fp32 arithmetic.
  static __device__ float vg_cost(const Args& a, const VirtualBlock& vb) {
    const float h = a.h, cs = a.cell, cm = a.cutoff + 0.05f;
    const int nc = (int)a.ncell;
    const float bx0 = h * (float)(vb.x * 8), bx1 = h * (float)(vb.x * 8 + 7);
    const float by0 = h * (float)(vb.y * 8), by1 = h * (float)(vb.y * 8 + 7);
    const float bz0 = h * (float)(vb.z * 8), bz1 = h * (float)(vb.z * 8 + 7);
    auto clampc = [&](int v) { return v < 0 ? 0 : (v >= nc ? nc - 1 : v); };
    const int cy0 = clampc((int)floorf((by0 - cm) / cs)), cy1 = clampc((int)floorf((by1 + cm) / cs));
    const int cz0 = clampc((int)floorf((bz0 - cm) / cs)), cz1 = clampc((int)floorf((bz1 + cm) / cs));
    float atoms = 0.f;
    for (int cz = cz0; cz <= cz1; ++cz) {
      const float gz = gap(bz0, bz1, cz * cs, (cz + 1) * cs);
      for (int cy = cy0; cy <= cy1; ++cy) {
        const float gy = gap(by0, by1, cy * cs, (cy + 1) * cs);
        const float d2 = gy * gy + gz * gz;
        if (d2 >= cm * cm) continue;
        const float rx = sqrtf(cm * cm - d2);
        const int cx0 = clampc((int)floorf((bx0 - rx) / cs)), cx1 = clampc((int)floorf((bx1 + rx) / cs));
        const int row = (cz * nc + cy) * nc;
        atoms += (float)(a.cell_start[row + cx1 + 1] - a.cell_start[row + cx0]);
      }
    }
    return atoms;
  }

  static __device__ __forceinline__ void body(const Args& a, const VirtualBlock& vb, char* smem) {
    float4* tile = reinterpret_cast<float4*>(smem);
    const int t = threadIdx.x;
    const int i = vb.x * 8 + (t & 7);
    const int j = vb.y * 8 + ((t >> 3) & 7);
    const int k0 = vb.z * 8 + (t >> 6) * kPts;
    const float h = a.h;
    const float px = h * (float)i, py = h * (float)j;
    float pz[kPts];
#pragma unroll
    for (int p = 0; p < kPts; ++p) pz[p] = h * (float)(k0 + p);
    const float c = a.cutoff;
    const float c2 = c * c, e2 = a.excl * a.excl, inv_c2 = 1.0f / c2;
    // excl[p] = "some r^2 < e^2" is kept as the running minimum of r^2 (one
    // FMNMX per pair instead of a compare, select and byte merge)
    float sum[kPts], r2min[kPts];
#pragma unroll
    for (int p = 0; p < kPts; ++p) {
      sum[p] = 0.f;
      r2min[p] = __int_as_float(0x7f800000);   // +inf
    }
    // VG bounding box in Angstrom
    const float bx0 = h * (float)(vb.x * 8), bx1 = h * (float)(vb.x * 8 + 7);
    const float by0 = h * (float)(vb.y * 8), by1 = h * (float)(vb.y * 8 + 7);
    const float bz0 = h * (float)(vb.z * 8), bz1 = h * (float)(vb.z * 8 + 7);
    const float cs = a.cell;
    const int nc = (int)a.ncell;
    const float cm = c + 0.05f;  // conservative margin for the cell filter
    auto clampc = [&](int v) { return v < 0 ? 0 : (v >= nc ? nc - 1 : v); };
    const int cy0 = clampc((int)floorf((by0 - cm) / cs)), cy1 = clampc((int)floorf((by1 + cm) / cs));
    const int cz0 = clampc((int)floorf((bz0 - cm) / cs)), cz1 = clampc((int)floorf((bz1 + cm) / cs));
    // the cell rows' trimmed atom ranges are packed back to back into the
    // shared tile (a row of 2-A cells holds a few atoms), which is evaluated
    // whenever it is full: two barriers per 128 atoms instead of per row
    auto evaluate = [&](int n) {
#pragma unroll 2
      for (int q = 0; q < n; ++q) {
        const float4 at = tile[q];
        const float dx = __fsub_rn(px, at.x), dy = __fsub_rn(py, at.y);
        const float dxy = __fadd_rn(__fmul_rn(dx, dx), __fmul_rn(dy, dy));
#pragma unroll
        for (int p = 0; p < kPts; ++p) {
          const float dz = __fsub_rn(pz[p], at.z);
          const float r2 = __fadd_rn(dxy, __fmul_rn(dz, dz));
          r2min[p] = fminf(r2min[p], r2);
          if (r2 < c2) {
            // explicit FMAs: the same op sequence in every instantiation
            // (native and persistent must agree bit for bit)
            const float s = __fmaf_rn(-r2, inv_c2, 1.0f);
            const float qs = __fmul_rn(__fmul_rn(at.w, rsqrt_ftz(r2)), s);
            sum[p] = __fmaf_rn(qs, s, sum[p]);
          }
        }
      }
    };
    int fill = 0;   // atoms staged in the tile (uniform)
#if CUTCP_GATHER
    // The cell rows' atom ranges are found in parallel, one row per thread
    // per batch of kThreads rows (same (cz, cy) order and fp32 arithmetic as
    // the row loop below), prefix-summed, and the tile is then gathered one
    // atom per thread, each locating its row by binary search.  One dependent
    // global round trip per tile instead of two per row: the tile holds the
    // same atoms in the same order, so the sums are bit-identical.
    int* row_a0 = reinterpret_cast<int*>(smem + kTile * sizeof(float4));
    int* row_pre = row_a0 + kThreads;              // kThreads + 1 entries
    int* wsum = row_pre + kThreads + 1;            // kThreads / 32 entries
    const int nyc = cy1 - cy0 + 1, nrows = (cz1 - cz0 + 1) * nyc;
    for (int rb = 0; rb < nrows; rb += kThreads) {
      int a0 = 0, len = 0;
      const int rr = rb + t;
      if (rr < nrows) {
        const int cz = cz0 + rr / nyc, cy = cy0 + rr % nyc;
        const float gz = gap(bz0, bz1, cz * cs, (cz + 1) * cs);
        const float gy = gap(by0, by1, cy * cs, (cy + 1) * cs);
        const float d2 = gy * gy + gz * gz;
        if (d2 < cm * cm) {
          const float rx = sqrtf(cm * cm - d2);
          const int cx0 = clampc((int)floorf((bx0 - rx) / cs)), cx1 = clampc((int)floorf((bx1 + rx) / cs));
          const int row = (cz * nc + cy) * nc;
          a0 = __ldg(a.cell_start + row + cx0);
          len = __ldg(a.cell_start + row + cx1 + 1) - a0;
        }
      }
      // block exclusive scan of len
      int inc = len;
#pragma unroll
      for (int o = 1; o < 32; o <<= 1) {
        const int v = __shfl_up_sync(0xffffffffu, inc, o);
        if ((t & 31) >= o) inc += v;
      }
      __syncthreads();   // the previous batch's gather is done with row_a0 / row_pre
      if ((t & 31) == 31) wsum[t >> 5] = inc;
      __syncthreads();
      int base = 0, tot = 0;
#pragma unroll
      for (int w = 0; w < kThreads / 32; ++w) {
        const int s = wsum[w];
        base += w < (t >> 5) ? s : 0;
        tot += s;
      }
      row_a0[t] = a0;
      row_pre[t] = base + inc - len;
      if (t == 0) row_pre[kThreads] = tot;
      __syncthreads();
      for (int done = 0; done < tot;) {
        const int take = min(kTile - fill, tot - done);
        if (t < take) {
          const int pos = done + t;
          // the last row r with row_pre[r] <= pos: never an empty row (its
          // successor starts at the same position); row_pre[kThreads] = tot > pos
          int lo = 0, hi = kThreads;
          while (hi - lo > 1) {
            const int mid = (lo + hi) >> 1;
            if (row_pre[mid] <= pos) lo = mid; else hi = mid;
          }
          tile[fill + t] = __ldg(reinterpret_cast<const float4*>(a.atoms) + row_a0[lo] + (pos - row_pre[lo]));
        }
        fill += take;
        done += take;
        if (fill == kTile) {
          __syncthreads();
          evaluate(kTile);
          __syncthreads();
          fill = 0;
        }
      }
    }
#else
    for (int cz = cz0; cz <= cz1; ++cz) {
      const float gz = gap(bz0, bz1, cz * cs, (cz + 1) * cs);
      for (int cy = cy0; cy <= cy1; ++cy) {
        const float gy = gap(by0, by1, cy * cs, (cy + 1) * cs);
        const float d2 = gy * gy + gz * gz;
        if (d2 >= cm * cm) continue;  // uniform across the CTA
        const float rx = sqrtf(cm * cm - d2);
        const int cx0 = clampc((int)floorf((bx0 - rx) / cs)), cx1 = clampc((int)floorf((bx1 + rx) / cs));
        const int row = (cz * nc + cy) * nc;
        int a0 = __ldg(a.cell_start + row + cx0);
        const int a1 = __ldg(a.cell_start + row + cx1 + 1);
        while (a0 < a1) {
          const int take = min(kTile - fill, a1 - a0);
          if (t < take) tile[fill + t] = __ldg(reinterpret_cast<const float4*>(a.atoms) + a0 + t);
          fill += take;
          a0 += take;
          if (fill == kTile) {
            __syncthreads();
            evaluate(kTile);
            __syncthreads();
            fill = 0;
          }
        }
      }
    }
#endif
    if (fill) {
      __syncthreads();
      evaluate(fill);
    }
    __syncthreads();   // the CTA's next VG reuses the tile
    if (i < (int)a.nx && j < (int)a.ny) {
#pragma unroll
      for (int p = 0; p < kPts; ++p) {
        const int k = k0 + p;
        if (k < (int)a.nz) a.v[((size_t)k * a.ny + j) * a.nx + i] = r2min[p] < e2 ? 0.f : sum[p];
      }
    }
  }
};

}  // namespace accel
