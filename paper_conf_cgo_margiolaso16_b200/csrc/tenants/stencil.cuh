// stencil -- 7-point 3-D Jacobi sweep (Parboil "stencil", named in PAPER.md
// lines 290-291), fp32, A[z][y][x] with x fastest.
//
// One VG = a 128 x 8 x 8 (x, y, z) tile; 256 threads = 8 warps, warp w owns
// row y0+w, lane l owns x0+4l..x0+4l+3 (one 16-B vector).  The tile is walked
// along z with the column (z-1, z, z+1) kept in registers, loads prefetched two
// planes ahead (HBM latency ~ 1 us needs ~35 KB in flight per SM).  y
// neighbours come from a double-buffered shared-memory plane of 10 rows (8 own
// rows + 2 halo rows), x neighbours from warp shuffles (+ one scalar edge load
// per row end).  One __syncthreads per plane.  Algorithmic traffic: 8 B per
// point per sweep (read + write once); halos come from L2.
#pragma once
#include "../device/dispatch.cuh"
#include "accel_tenants.h"

namespace accel {

struct Stencil {
  using Args = accel_stencil_args;
  static constexpr int kThreads = 256;
  static constexpr uint32_t kTX = 128, kTY = 8, kTZ = 8;
  static constexpr uint32_t kChunk = 1;
  static constexpr int kMinBlocks = 5;     // <= 51 regs: 40 warps/SM in both modes
  static constexpr uint32_t kRows = kTY + 2;
  static constexpr uint32_t kDynSmem = 2 * kRows * kTX * sizeof(float);  // 10 KB

  static __device__ __forceinline__ float4 zero4() { return make_float4(0.f, 0.f, 0.f, 0.f); }

  static __device__ __forceinline__ void body(const Args& a, const VirtualBlock& vb, char* smem) {
    const uint32_t r = vb.launch_idx;
    const float* __restrict__ in = r == 0 ? a.a0 : ((r & 1) ? a.buf0 : a.buf1);
    float* __restrict__ out = (r & 1) ? a.buf1 : a.buf0;
    const int nx = (int)a.nx, ny = (int)a.ny, nz = (int)a.nz;
    const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
    const int x0 = (int)vb.x * (int)kTX + 4 * lane;
    const int y0 = (int)vb.y * (int)kTY;
    const int y = y0 + warp;
    const int z0 = (int)vb.z * (int)kTZ;
    const int zend = min(z0 + (int)kTZ, nz);
    const size_t plane = (size_t)nx * (size_t)ny;
    const bool xin = x0 < nx, yin = y < ny;
    float4* S = reinterpret_cast<float4*>(smem);  // [2][kRows][32]

    auto row4 = [&](int zz, int yy) -> float4 {
      if (xin && yy >= 0 && yy < ny && zz >= 0 && zz < nz)
        return __ldg(reinterpret_cast<const float4*>(in + (size_t)zz * plane + (size_t)yy * nx + x0));
      return zero4();
    };
    // halo row owned by warp 0 (y0-1) and warp 7 (y0+8)
    const int hy = warp == 0 ? y0 - 1 : y0 + (int)kTY;
    const bool hown = warp == 0 || warp == (int)kTY - 1;
    auto halo = [&](int zz) -> float4 { return hown ? row4(zz, hy) : zero4(); };
    // scalar x-edge owned by lane 0 (x0-1) and lane 31 (x0+4)
    const int ex = lane == 0 ? x0 - 1 : x0 + 4;
    const bool eown = (lane == 0 || lane == 31) && yin && ex >= 0 && ex < nx;
    auto edge = [&](int zz) -> float {
      if (eown && zz >= 0 && zz < nz) return __ldg(in + (size_t)zz * plane + (size_t)y * nx + ex);
      return 0.f;
    };

    float4 zm = row4(z0 - 1, y), cur = row4(z0, y), n1 = row4(z0 + 1, y);
    float4 hc = halo(z0);
    float ec = edge(z0);
    const float c0 = a.c0, c1 = a.c1;
    const bool yint = y >= 1 && y <= ny - 2;
    int buf = 0;
    for (int z = z0; z < zend; ++z) {
      // prefetch: plane z+2 of the own column, halo/edges of plane z+1
      const float4 n2 = (z + 2 <= zend) ? row4(z + 2, y) : zero4();
      const float4 hn = (z + 1 < zend) ? halo(z + 1) : zero4();
      const float en = (z + 1 < zend) ? edge(z + 1) : 0.f;

      float4* Sb = S + buf * (kRows * 32);
      Sb[(warp + 1) * 32 + lane] = cur;
      if (hown) Sb[(warp == 0 ? 0 : kRows - 1) * 32 + lane] = hc;
      float xl = __shfl_up_sync(0xffffffffu, cur.w, 1);
      float xr = __shfl_down_sync(0xffffffffu, cur.x, 1);
      if (lane == 0) xl = ec;
      if (lane == 31) xr = ec;
      __syncthreads();
      const float4 ym = Sb[warp * 32 + lane];
      const float4 yp = Sb[(warp + 2) * 32 + lane];

      if (xin && yin) {
        const bool zint = z >= 1 && z <= nz - 2;
        const bool inner = yint && zint;
        float4 o;
        const float cx[4] = {cur.x, cur.y, cur.z, cur.w};
        const float mx[4] = {xl, cur.x, cur.y, cur.z};
        const float px[4] = {cur.y, cur.z, cur.w, xr};
        const float zmv[4] = {zm.x, zm.y, zm.z, zm.w};
        const float zpv[4] = {n1.x, n1.y, n1.z, n1.w};
        const float ymv[4] = {ym.x, ym.y, ym.z, ym.w};
        const float ypv[4] = {yp.x, yp.y, yp.z, yp.w};
        float ov[4];
#pragma unroll
        for (int e = 0; e < 4; ++e) {
          const int x = x0 + e;
          const bool in_x = x >= 1 && x <= nx - 2;
          const float s = ((((zmv[e] + zpv[e]) + ymv[e]) + ypv[e]) + mx[e]) + px[e];
          ov[e] = (inner && in_x) ? s * c1 - cx[e] * c0 : cx[e];
        }
        o = make_float4(ov[0], ov[1], ov[2], ov[3]);
        *reinterpret_cast<float4*>(out + (size_t)z * plane + (size_t)y * nx + x0) = o;
      }
      zm = cur;
      cur = n1;
      n1 = n2;
      hc = hn;
      ec = en;
      buf ^= 1;
    }
  }
};

}  // namespace accel
