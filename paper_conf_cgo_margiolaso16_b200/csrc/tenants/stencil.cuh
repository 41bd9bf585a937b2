// stencil -- 7-point 3-D Jacobi sweep (Parboil "stencil", named in PAPER.md
// lines 290-291), fp32, A[z][y][x] with x fastest.
//
// One VG = a 128 x 8 x 8 (x, y, z) tile; 256 threads = 8 warps, warp w owns
// row y0+w, lane l owns x0+4l..x0+4l+3 (one 16-B vector).  The tile is walked
// along z (fully unrolled, so the register rotation of the column
// z-1, z, z+1 costs nothing) with loads issued three planes ahead (HBM latency
// ~1 us needs ~40 KB in flight per SM).  y neighbours come from a
// double-buffered shared-memory plane of 10 rows (8 own rows + 2 halo rows),
// x neighbours from warp shuffles plus one scalar edge load per row end.  One
// __syncthreads per plane.
//
// Layout contract (include/accel_tenants.h): every volume has one readable
// plane before z = 0 and three after z = nz-1, so the halo / prefetch loads
// at the domain faces are plain in-bounds loads (their values only feed face
// cells, which copy the input) and the loop body has no bounds logic at all.
// Algorithmic traffic: 8 B per point per sweep.
#pragma once
#include "../device/dispatch.cuh"
#include "accel_tenants.h"

namespace accel {

struct Stencil {
  using Args = accel_stencil_args;
  static constexpr int kThreads = 256;
  static constexpr int kTX = 128, kTY = 8, kTZ = 8;
  static constexpr uint32_t kChunk = 1;
  static constexpr int kMinBlocks = 4;     // <= 64 regs: 32 warps/SM in both modes
  static constexpr int kRows = kTY + 2;
  static constexpr uint32_t kDynSmem = 2 * kRows * kTX * sizeof(float);  // 10 KB

  static __device__ __forceinline__ float4 ld4(const float* p) {
    return __ldg(reinterpret_cast<const float4*>(p));
  }

  static __device__ __forceinline__ void body(const Args& a, const VirtualBlock& vb, char* smem) {
    const uint32_t r = vb.launch_idx;
    const float* __restrict__ in = r == 0 ? a.a0 : ((r & 1) ? a.buf0 : a.buf1);
    float* __restrict__ out = (r & 1) ? a.buf1 : a.buf0;
    const int nx = (int)a.nx, ny = (int)a.ny, nz = (int)a.nz;
    const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
    const int x0 = (int)vb.x * kTX + 4 * lane;
    const int y0 = (int)vb.y * kTY;
    const int y = y0 + warp;
    const int z0 = (int)vb.z * kTZ;
    const int nzt = min(kTZ, nz - z0);     // planes in this tile (ragged last tile)
    const int plane = nx * ny;
    const bool active = x0 < nx && y < ny;
    // rows beyond the domain in x or y read an in-range neighbour row (clamped
    // once); z never needs clamping thanks to the padding planes
    const int xc = min(x0, nx - 4);
    const int col = min(y, ny - 1) * nx + xc;
    const bool hown = warp == 0 || warp == kTY - 1;
    const int hrow = warp == 0 ? 0 : kRows - 1;
    const int hcol = min(warp == 0 ? y0 - 1 : y0 + kTY, ny - 1) * nx + xc;  // y0-1 = -1 is padding
    const bool eown = lane == 0 || lane == 31;
    const int ecol = min(y, ny - 1) * nx + (lane == 0 ? x0 - 1 : min(x0 + 4, nx - 1));
    const float* pc = in + z0 * plane + col;   // own column at plane z0
    const float* ph = in + z0 * plane + hcol;
    const float* pe = in + z0 * plane + ecol;
    float* po = out + z0 * plane + y * nx + x0;

    const bool yint = y >= 1 && y <= ny - 2;
    bool mxy[4];
#pragma unroll
    for (int e = 0; e < 4; ++e) mxy[e] = yint && (x0 + e >= 1) && (x0 + e <= nx - 2);
    const float c0 = a.c0, c1 = a.c1;

    float4 zm = ld4(pc - plane), cur = ld4(pc), n1 = ld4(pc + plane), n2 = ld4(pc + 2 * plane);
    float4 hc = hown ? ld4(ph) : cur;
    float ec = eown ? __ldg(pe) : 0.f;
    float4* S = reinterpret_cast<float4*>(smem);  // [2][kRows][32]
#pragma unroll
    for (int i = 0; i < kTZ; ++i) {
      if (i >= nzt) break;
      const int z = z0 + i;
      const float4 n3 = ld4(pc + (i + 3) * plane);
      const float4 hn = hown ? ld4(ph + (i + 1) * plane) : cur;
      const float en = eown ? __ldg(pe + (i + 1) * plane) : 0.f;

      float4* Sb = S + (i & 1) * (kRows * 32);
      Sb[(warp + 1) * 32 + lane] = cur;
      if (hown) Sb[hrow * 32 + lane] = hc;
      float xl = __shfl_up_sync(0xffffffffu, cur.w, 1);
      float xr = __shfl_down_sync(0xffffffffu, cur.x, 1);
      if (lane == 0) xl = ec;
      if (lane == 31) xr = ec;
      __syncthreads();
      const float4 ym = Sb[warp * 32 + lane];
      const float4 yp = Sb[(warp + 2) * 32 + lane];

      // compute every element unconditionally, then select (no branches)
      const float vx = ((((((zm.x + n1.x) + ym.x) + yp.x) + xl) + cur.y) * c1 - cur.x * c0);
      const float vy = ((((((zm.y + n1.y) + ym.y) + yp.y) + cur.x) + cur.z) * c1 - cur.y * c0);
      const float vz = ((((((zm.z + n1.z) + ym.z) + yp.z) + cur.y) + cur.w) * c1 - cur.z * c0);
      const float vw = ((((((zm.w + n1.w) + ym.w) + yp.w) + cur.z) + xr) * c1 - cur.w * c0);
      const bool zint = z >= 1 && z <= nz - 2;
      float4 o;
      o.x = (zint && mxy[0]) ? vx : cur.x;
      o.y = (zint && mxy[1]) ? vy : cur.y;
      o.z = (zint && mxy[2]) ? vz : cur.z;
      o.w = (zint && mxy[3]) ? vw : cur.w;
      if (active) *reinterpret_cast<float4*>(po + i * plane) = o;
      zm = cur;
      cur = n1;
      n1 = n2;
      n2 = n3;
      hc = hn;
      ec = en;
    }
  }
};

}  // namespace accel
