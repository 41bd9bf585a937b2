// stencil -- 7-point 3-D Jacobi sweep (Parboil "stencil", named in PAPER.md
// lines 290-291), fp32, A[z][y][x] with x fastest.
//
// One VG = a 128 x 8 x 8 (x, y, z) tile; 256 threads = 8 warps, warp w owns
// row y0+w, lane l owns x0+4l..x0+4l+3 (one 16-B vector).  The tile is walked
// along z with the column (z-1, z, z+1) kept in registers and loads issued
// three planes ahead (HBM latency ~ 1 us needs ~40 KB in flight per SM).  y
// neighbours come from a double-buffered shared-memory plane of 10 rows (8 own
// rows + 2 halo rows), x neighbours from warp shuffles plus one scalar edge
// load per row end.  One __syncthreads per plane.  All bounds handling is
// hoisted out of the z loop: out-of-domain rows/planes are clamped to a valid
// address (their values only feed boundary cells, which copy the input), so
// the loop body is branch-free.  Algorithmic traffic: 8 B per point per sweep.
#pragma once
#include "../device/dispatch.cuh"
#include "accel_tenants.h"

namespace accel {

struct Stencil {
  using Args = accel_stencil_args;
  static constexpr int kThreads = 256;
  static constexpr int kTX = 128, kTY = 8, kTZ = 8;
  static constexpr uint32_t kChunk = 1;
  static constexpr int kMinBlocks = 4;     // <= 64 regs: 32 warps/SM in both modes, 3 planes in flight
  static constexpr int kRows = kTY + 2;
  static constexpr uint32_t kDynSmem = 2 * kRows * kTX * sizeof(float);  // 10 KB

  static __device__ __forceinline__ int clampi(int v, int lo, int hi) { return v < lo ? lo : (v > hi ? hi : v); }

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
    const int zend = min(z0 + kTZ, nz);
    const int plane = nx * ny;
    const bool active = x0 < nx && y < ny;
    // clamped (always valid) column, halo and edge offsets inside one plane
    const int xc = min(x0, nx - 4);
    const int col = clampi(y, 0, ny - 1) * nx + xc;
    const bool hown = warp == 0 || warp == kTY - 1;
    const int hrow = warp == 0 ? 0 : kRows - 1;  // smem row of the halo
    const int hcol = clampi(warp == 0 ? y0 - 1 : y0 + kTY, 0, ny - 1) * nx + xc;
    const bool eown = lane == 0 || lane == 31;
    const int ecol = clampi(y, 0, ny - 1) * nx + clampi(lane == 0 ? x0 - 1 : x0 + 4, 0, nx - 1);
    auto zoff = [&](int z) { return clampi(z, 0, nz - 1) * plane; };
    auto ld4 = [&](int off) { return __ldg(reinterpret_cast<const float4*>(in + off)); };

    // per-element interior masks (x, y fixed for the whole column)
    const bool yint = y >= 1 && y <= ny - 2;
    bool mxy[4];
#pragma unroll
    for (int e = 0; e < 4; ++e) mxy[e] = yint && (x0 + e >= 1) && (x0 + e <= nx - 2);
    const float c0 = a.c0, c1 = a.c1;

    // pipeline: zm, cur, n1 = planes z-1, z, z+1; n2, n3 in flight
    float4 zm = ld4(zoff(z0 - 1) + col), cur = ld4(zoff(z0) + col);
    float4 n1 = ld4(zoff(z0 + 1) + col), n2 = ld4(zoff(z0 + 2) + col);
    float4 hc = hown ? ld4(zoff(z0) + hcol) : cur;
    float ec = eown ? __ldg(in + zoff(z0) + ecol) : 0.f;
    float4* S = reinterpret_cast<float4*>(smem);  // [2][kRows][32]
    int buf = 0;
    for (int z = z0; z < zend; ++z) {
      const float4 n3 = ld4(zoff(z + 3) + col);
      const float4 hn = hown ? ld4(zoff(z + 1) + hcol) : cur;
      const float en = eown ? __ldg(in + zoff(z + 1) + ecol) : 0.f;

      float4* Sb = S + buf * (kRows * 32);
      Sb[(warp + 1) * 32 + lane] = cur;
      if (hown) Sb[hrow * 32 + lane] = hc;
      float xl = __shfl_up_sync(0xffffffffu, cur.w, 1);
      float xr = __shfl_down_sync(0xffffffffu, cur.x, 1);
      if (lane == 0) xl = ec;
      if (lane == 31) xr = ec;
      __syncthreads();
      const float4 ym = Sb[warp * 32 + lane];
      const float4 yp = Sb[(warp + 2) * 32 + lane];

      if (active) {
        const bool zint = z >= 1 && z <= nz - 2;
        float4 o;
        o.x = (zint && mxy[0]) ? ((((((zm.x + n1.x) + ym.x) + yp.x) + xl) + cur.y) * c1 - cur.x * c0) : cur.x;
        o.y = (zint && mxy[1]) ? ((((((zm.y + n1.y) + ym.y) + yp.y) + cur.x) + cur.z) * c1 - cur.y * c0) : cur.y;
        o.z = (zint && mxy[2]) ? ((((((zm.z + n1.z) + ym.z) + yp.z) + cur.y) + cur.w) * c1 - cur.z * c0) : cur.z;
        o.w = (zint && mxy[3]) ? ((((((zm.w + n1.w) + ym.w) + yp.w) + cur.z) + xr) * c1 - cur.w * c0) : cur.w;
        *reinterpret_cast<float4*>(out + z * plane + y * nx + x0) = o;
      }
      zm = cur;
      cur = n1;
      n1 = n2;
      n2 = n3;
      hc = hn;
      ec = en;
      buf ^= 1;
    }
  }
};

}  // namespace accel
