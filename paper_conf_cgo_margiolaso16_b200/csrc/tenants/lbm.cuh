// lbm -- Parboil "lbm" (D3Q19 lattice Boltzmann; one of
// the 25 Parboil kernels of PAPER.md §7.2).  One launch = one
// pull-stream + BGK-collide step over the whole lattice (a request = `steps`
// launches, ping-pong like stencil, R-job-1).
//
// VG = 128 consecutive cells of one x row; thread = cell.  The 19 pulls
// g_q = f_q(x - c_q) (periodic) are coalesced along x for every q (SoA
// f[q][z][y][x]); obstacle cells bounce back (f'_q = g_opp(q)), fluid cells
// relax to the second-order equilibrium.  HBM-bound: 19 x 4 B read + 19 x 4 B
// written (+1 B of flags) per cell per step.
#pragma once
#include "../device/dispatch.cuh"
#include "accel_tenants.h"

namespace accel {

struct Lbm {
  using Args = accel_lbm_args;
  static constexpr int kThreads = 128;
  static constexpr uint32_t kChunk = 1;
  static constexpr int kMinBlocks = 8;   // 64 registers: the persistent loop keeps the native 8 CTAs/SM (at 6: +5 % per launch)
  static constexpr uint32_t kDynSmem = 0;

  static __device__ __forceinline__ void body(const Args& a, const VirtualBlock& vb, char*) {
    // velocity table (oracle/tenants.c order): rest, +-x, +-y, +-z, then the
    // 12 diagonals in opposite pairs
    constexpr int cx[19] = {0, 1, -1, 0, 0, 0, 0, 1, -1, 1, -1, 1, -1, 1, -1, 0, 0, 0, 0};
    constexpr int cy[19] = {0, 0, 0, 1, -1, 0, 0, 1, -1, -1, 1, 0, 0, 0, 0, 1, -1, 1, -1};
    constexpr int cz[19] = {0, 0, 0, 0, 0, 1, -1, 0, 0, 0, 0, 1, -1, -1, 1, 1, -1, -1, 1};
    const int nx = (int)a.nx, ny = (int)a.ny, nz = (int)a.nz;
    const int x = (int)vb.x * kThreads + (int)threadIdx.x;
    if (x >= nx) return;
    const int y = (int)vb.y, z = (int)vb.z;
    const uint32_t r = vb.launch_idx;
    const float* __restrict__ src = r == 0 ? a.f0 : ((r & 1u) ? a.buf0 : a.buf1);
    float* __restrict__ dst = (r & 1u) ? a.buf1 : a.buf0;
    const size_t n = (size_t)nx * ny * nz;
    const size_t i = ((size_t)z * ny + y) * nx + x;
    // neighbour rows / planes and x positions (periodic)
    const int xm = x == 0 ? nx - 1 : x - 1, xp = x == nx - 1 ? 0 : x + 1;
    const int ym = y == 0 ? ny - 1 : y - 1, yp = y == ny - 1 ? 0 : y + 1;
    const int zm = z == 0 ? nz - 1 : z - 1, zp = z == nz - 1 ? 0 : z + 1;
    float g[19];
#pragma unroll
    for (int q = 0; q < 19; ++q) {
      // source cell x - c_q
      const int xs = cx[q] == 1 ? xm : (cx[q] == -1 ? xp : x);
      const int ys = cy[q] == 1 ? ym : (cy[q] == -1 ? yp : y);
      const int zs = cz[q] == 1 ? zm : (cz[q] == -1 ? zp : z);
      g[q] = __ldcs(src + (size_t)q * n + ((size_t)zs * ny + ys) * nx + xs);
    }
    if (a.flags[i]) {   // bounce-back: f'_q = g_opp(q)
      constexpr int opp[19] = {0, 2, 1, 4, 3, 6, 5, 8, 7, 10, 9, 12, 11, 14, 13, 16, 15, 18, 17};
#pragma unroll
      for (int q = 0; q < 19; ++q) __stcs(dst + (size_t)q * n + i, g[opp[q]]);
      return;
    }
    float rho = 0.f, ux = 0.f, uy = 0.f, uz = 0.f;
#pragma unroll
    for (int q = 0; q < 19; ++q) {
      rho += g[q];
      ux += (float)cx[q] * g[q];
      uy += (float)cy[q] * g[q];
      uz += (float)cz[q] * g[q];
    }
    const float inv = 1.0f / rho;
    ux *= inv;
    uy *= inv;
    uz *= inv;
    const float uu = 1.5f * (ux * ux + uy * uy + uz * uz);
    const float om = a.omega;
#pragma unroll
    for (int q = 0; q < 19; ++q) {
      const float wq = q == 0 ? 1.0f / 3.0f : (q <= 6 ? 1.0f / 18.0f : 1.0f / 36.0f);
      const float cu = (float)cx[q] * ux + (float)cy[q] * uy + (float)cz[q] * uz;
      const float feq = wq * rho * (1.0f + 3.0f * cu + 4.5f * cu * cu - uu);
      __stcs(dst + (size_t)q * n + i, g[q] + om * (feq - g[q]));
    }
  }
};

}  // namespace accel
