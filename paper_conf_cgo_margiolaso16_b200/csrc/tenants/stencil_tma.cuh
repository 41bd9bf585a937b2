// stencil_tma -- the 7-point Jacobi sweep of stencil.cuh with its planes
// staged by the Tensor Memory Accelerator (PAPER.md names Parboil "stencil",
// lines 290-291; BASELINE.json: "shared-memory or TMA staging for stencil").
//
// Why: stencil is the HBM-bound tenant of the Fig. 2 mix.  Under space
// sharing it holds about a quarter of its solo CTAs, so its bandwidth is set
// by the bytes in flight PER CTA, not by how many warps it has.  With cp.async
// every byte in flight is a thread's outstanding copy and every plane a CTA
// barrier; here one producer thread keeps kNS - 2 planes (~33 KB) in flight
// per CTA through a ring of mbarrier-tracked TMA boxes, and the eight
// consumer warps never meet at a CTA barrier inside a VG.
//
// VG = 128 x 8 x 8 (x, y, z) tile, 288 threads:
//   warps 0..7  consumers: warp w owns row y0 + w, lane l owns x0+4l..x0+4l+3;
//               the column z-1, z, z+1 lives in registers, y neighbours and
//               the two x edges come from the staged plane, inner x
//               neighbours from shuffles (same arithmetic and association as
//               stencil.cuh, so the result is bit-identical)
//   warp 8      producer (lane 0): plane p of the tile (z0 - 1 + p) is ONE
//               cp.async.bulk.tensor.3d box (x0-4 .. x0+131, y0-1 .. y0+8, z)
//               into ring slot p % kNS; boxes partly outside the volume read
//               zeros (they only feed face cells, which copy the input)
// Ring protocol: full[s] (1 arrival + the box's transaction bytes) and
// empty[s] (one arrival per consumer warp once it last read the slot).  The
// barriers are initialised per VG; every box a VG issues is waited for by
// every consumer before the VG ends, so nothing asynchronous outlives it.
// The tensor maps are __grid_constant__ kernel parameters (no descriptor in
// global memory that a later job could overwrite).
#pragma once
#include "../device/dispatch.cuh"
#include "accel_tenants.h"
#include "tma.cuh"

namespace accel {

// diagnostic build switch (scripts/diag_tma_check.py, diag_tma_which.py):
// compare every staged plane row with an L2 load (the product build leaves
// it out: the extra code spilled the 40-register budget)
#ifndef ACCEL_XP_TMA_DBG
#define ACCEL_XP_TMA_DBG 0
#endif

// kBulk: the same ring filled by plain 1-D bulk copies (cp.async.bulk, one
// per in-volume row segment of a plane) instead of 3-D tensor boxes: no
// tensor map; rows and columns outside the volume are not copied (their smem
// holds stale values that only feed face cells, which copy the input).
template <bool kBulk>
struct StencilTmaT {
  using Args = accel_stencil_tma_args;
  static constexpr int kConsumers = 8;
  static constexpr int kThreads = 32 * (kConsumers + 1);
  static constexpr int kTX = 128, kTY = 8, kTZ = 8;
  static constexpr uint32_t kChunk = 1;
#ifndef STENCIL_TMA_NS
#define STENCIL_TMA_NS 8
#endif
  static constexpr int kNS = STENCIL_TMA_NS;            // ring slots (planes)
  static constexpr int kMinBlocks = 5;
  static constexpr int kRows = kTY + 2, kCols = kTX + 8;
  static constexpr uint32_t kPlaneBytes = kRows * kCols * 4;          // 5440 (one box)
  static constexpr uint32_t kSlot = (kPlaneBytes + 127) / 128 * 128;  // 5504
  static constexpr uint32_t kDynSmem = kNS * kSlot + 2 * kNS * 8 + 128;   // + barriers, + alignment

  // ((((((zm + zp) + ym) + yp) + xm) + xp) * c1) - (c * c0), each step fp32 RN
  static __device__ __forceinline__ float point(float zm, float zp, float ym, float yp, float xm, float xp, float c,
                                                float c0, float c1) {
    const float s = __fadd_rn(__fadd_rn(__fadd_rn(__fadd_rn(__fadd_rn(zm, zp), ym), yp), xm), xp);
    return __fsub_rn(__fmul_rn(s, c1), __fmul_rn(c, c0));
  }

  // The race behind the drift next to bfs (scripts/diag_tma_which.py): a
  // consumer warp released a ring slot right after ISSUING its ld.shared of
  // the slot; the producer, spinning on that empty barrier, issued the TMA of
  // plane z0+7 into slot 0, which landed before the load read it -- the staged
  // "plane z0-1" values equalled plane z0+7 exactly.  Slots are now released
  // with tma::mbar_release_after (the release waits for the loaded data).
  static __device__ __forceinline__ void body(const Args& a, const VirtualBlock& vb, char* smem_raw) {
    using namespace tma;
    const uint32_t r = vb.launch_idx;
    const int nx = (int)a.nx, ny = (int)a.ny, nz = (int)a.nz;
    const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
    const int x0 = (int)vb.x * kTX, y0 = (int)vb.y * kTY, z0 = (int)vb.z * kTZ;
    const int nzt = min(kTZ, nz - z0);
    const int nplanes = nzt + 2;
    const uint32_t sbase = (smem_u32(smem_raw) + 127u) & ~127u;
    const uint32_t full0 = sbase + kNS * kSlot, empty0 = full0 + 8u * kNS;
    auto slot = [&](int p) { return sbase + (uint32_t)(p % kNS) * kSlot; };
    auto full = [&](int p) { return full0 + 8u * (uint32_t)(p % kNS); };
    auto empty = [&](int p) { return empty0 + 8u * (uint32_t)(p % kNS); };
    if (threadIdx.x == 0) {
#pragma unroll
      for (int q = 0; q < kNS; ++q) {
        mbar_init(full0 + 8u * q, 1);
        mbar_init(empty0 + 8u * q, kConsumers);
      }
      asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
    }
    __syncthreads();

    if (warp == kConsumers) {
      // ---- producer: launch r reads a0 (r == 0), buf0 (r odd), buf1 (r even)
      if (lane == 0) {
        const int mi = r == 0 ? 0 : ((r & 1u) ? 1 : 2);
        const accel_tmap* map = a.gmaps ? a.gmaps + mi : &a.tmaps[mi];
        if (a.gmaps) tmap_acquire(map);
        // the input was written through the generic proxy (by the previous
        // launch, or -- for a RESOLVE top-up CTA -- by other CTAs of this
        // grid, ordered by the dispatch's wait_complete and the barrier above)
        asm volatile("fence.proxy.async.global;" ::: "memory");
        // bulk path: the plane's in-volume row segments (16-B aligned: nx % 4 == 0)
        const int xs = max(x0 - 4, 0), xe = min(x0 + kTX + 4, nx);
        const uint32_t rowb = 4u * (uint32_t)(xe - xs), dcol = 4u * (uint32_t)(xs - (x0 - 4));
        const int ys = max(y0 - 1, 0), ye = min(y0 + kTY + 1, ny);
        const float* in = r == 0 ? a.a0 : ((r & 1u) ? a.buf0 : a.buf1);
        // diagnostics (scripts/diag_tma_check.py): l2hint bit 3 = issue plane 1
        // before plane 0; bit 4 = wait 2 us after the proxy fence
        if (a.l2hint & 16u) __nanosleep(2000);
        for (int p0 = 0; p0 < nplanes; ++p0) {
          const int p = (a.l2hint & 8u) ? (p0 == 0 ? 1 : (p0 == 1 ? 0 : p0)) : p0;
          if (p >= kNS) mbar_wait(empty(p), (uint32_t)((p / kNS) - 1) & 1u);
          if constexpr (kBulk) {
            const int z = z0 - 1 + p;
            if (z < 0 || z >= nz) {
              mbar_arrive(full(p));   // nothing to copy: a face plane
              continue;
            }
            mbar_expect_tx(full(p), rowb * (uint32_t)(ye - ys));
            for (int y = ys; y < ye; ++y) {
              const float* g = in + ((size_t)z * ny + y) * nx + xs;
              const uint32_t dst = slot(p) + 4u * (uint32_t)((y - (y0 - 1)) * kCols) + dcol;
              asm volatile("cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes [%0], [%1], %2, [%3];"
                           ::"r"(dst), "l"(g), "r"(rowb), "r"(full(p)) : "memory");
            }
          } else {
            mbar_expect_tx(full(p), kPlaneBytes);
            if ((a.l2hint & 3u) == 0)
              tma_load_3d(slot(p), map, x0 - 4, y0 - 1, z0 - 1 + p, full(p));
            else
              tma_load_3d_hint(slot(p), map, x0 - 4, y0 - 1, z0 - 1 + p, full(p),
                               (a.l2hint & 3u) == 1 ? policy_evict_first() : policy_evict_last());
          }
        }
      }
      return;   // (the dispatch loop's barrier follows)
    }

    // ---- consumers
    float* __restrict__ out = (r & 1u) ? a.buf1 : a.buf0;
    const int y = y0 + warp;
    const bool active = x0 + 4 * lane < nx && y < ny;
    const bool yint = y >= 1 && y <= ny - 2;
    bool mxy[4];
#pragma unroll
    for (int e = 0; e < 4; ++e) {
      const int x = x0 + 4 * lane + e;
      mxy[e] = yint && x >= 1 && x <= nx - 2;
    }
    const float c0 = a.c0, c1 = a.c1;
    const uint32_t own = 4u * (uint32_t)((warp + 1) * kCols + 4 + 4 * lane);
    const uint32_t edge = 4u * (uint32_t)((warp + 1) * kCols + (lane == 31 ? 4 + kTX : 3));
    mbar_wait(full(0), 0);
    const float4 zm0 = lds_f4(slot(0) + own);
    // plane z0-1 is only a z neighbour: release its slot once this warp's
    // reads of it are ordered before the next TMA into it (release_after)
    const uint32_t zmask = (uint32_t)nz >> 31;   // 0 at run time (tma::mbar_release_after)
    mbar_release_after(empty(0), __float_as_uint(zm0.x), zmask, lane);
    mbar_wait(full(1), 0);
    float4 zm = zm0, cur = lds_f4(slot(1) + own);
    if (ACCEL_XP_TMA_DBG && a.dbg != nullptr) {
      // diagnostic: the first two planes (z0-1, z0) as staged vs an L2 load (tag 3 << 30: zm, 0 << 30 ... cur)
      const float* in = r == 0 ? a.a0 : ((r & 1u) ? a.buf0 : a.buf1);
#pragma unroll
      for (int s2 = 0; s2 < 2; ++s2) {
        const int zz = z0 - 1 + s2;
        const float4 st = s2 == 0 ? zm : cur;
        if (active && zz >= 0 && zz < nz) {
          const float4 g = __ldcg(reinterpret_cast<const float4*>(in + ((size_t)zz * ny + y) * nx + x0 + 4 * lane));
          const float sv[4] = {st.x, st.y, st.z, st.w}, gv[4] = {g.x, g.y, g.z, g.w};
#pragma unroll
          for (int e = 0; e < 4; ++e)
            if (__float_as_uint(sv[e]) != __float_as_uint(gv[e])) {
              const uint32_t k = atomicAdd(a.dbg, 1u);
              if (k < 16u) {
                uint32_t* rec = a.dbg + 8 + 8 * k;
                rec[0] = r; rec[1] = (uint32_t)zz | (3u << 30); rec[2] = (uint32_t)y;
                rec[3] = (uint32_t)(x0 + 4 * lane + e); rec[4] = __float_as_uint(sv[e]); rec[5] = __float_as_uint(gv[e]);
                rec[6] = smid(); rec[7] = (uint32_t)s2;
              }
            }
        }
      }
    }
    const long long pstr = (long long)nx * ny;
    float* po = out + ((size_t)z0 * ny + y) * nx + x0 + 4 * lane;
#pragma unroll 1
    for (int i = 0; i < nzt; ++i) {
      const int pz = i + 1;   // plane pz (= z0 + i) is `cur`
      mbar_wait(full(pz + 1), (uint32_t)((pz + 1) / kNS) & 1u);
      const uint32_t P = slot(pz);
      const float4 zp = lds_f4(slot(pz + 1) + own);
      if (ACCEL_XP_TMA_DBG && a.dbg != nullptr) {
        // diagnostic: the staged row of plane z0+i+1 vs an L2 load of the same input
        const int zz = z0 + i + 1;
        if (active && zz < nz) {
          const float* in = r == 0 ? a.a0 : ((r & 1u) ? a.buf0 : a.buf1);
          const float* ot = (r & 1u) ? a.buf1 : a.buf0;
          const size_t off = ((size_t)zz * ny + y) * nx + x0 + 4 * lane;
          const float4 g = __ldcg(reinterpret_cast<const float4*>(in + off));
          const float4 o = __ldcg(reinterpret_cast<const float4*>(ot + off));
          const float sv[4] = {zp.x, zp.y, zp.z, zp.w}, gv[4] = {g.x, g.y, g.z, g.w}, ov[4] = {o.x, o.y, o.z, o.w};
#pragma unroll
          for (int e = 0; e < 4; ++e)
            if (__float_as_uint(sv[e]) != __float_as_uint(gv[e])) {
              const uint32_t k = atomicAdd(a.dbg, 1u);
              if (k < 16u) {
                uint32_t* rec = a.dbg + 8 + 8 * k;
                rec[0] = r; rec[1] = (uint32_t)zz; rec[2] = (uint32_t)y; rec[3] = (uint32_t)(x0 + 4 * lane + e);
                rec[4] = __float_as_uint(sv[e]); rec[5] = __float_as_uint(gv[e]); rec[6] = smid();
                rec[7] = __float_as_uint(ov[e]);
              }
            }
        }
      }
      const float4 ym = lds_f4(P + own - 4u * kCols);
      const float4 yp = lds_f4(P + own + 4u * kCols);
      const float ev = lds_f32(P + edge);
      if (ACCEL_XP_TMA_DBG && a.dbg != nullptr) {
        // diagnostic: the y neighbours of plane z0+i as staged vs an L2 load (tag z | 1 << 30: ym, 2 << 30: yp)
        const int zc = z0 + i;
        const float* in = r == 0 ? a.a0 : ((r & 1u) ? a.buf0 : a.buf1);
#pragma unroll
        for (int s2 = 0; s2 < 2; ++s2) {
          const int yy = s2 == 0 ? y - 1 : y + 1;
          const float4 st = s2 == 0 ? ym : yp;
          if (x0 + 4 * lane < nx && yy >= 0 && yy < ny && zc < nz) {
            const float4 g = __ldcg(reinterpret_cast<const float4*>(in + ((size_t)zc * ny + yy) * nx + x0 + 4 * lane));
            const float sv[4] = {st.x, st.y, st.z, st.w}, gv[4] = {g.x, g.y, g.z, g.w};
#pragma unroll
            for (int e = 0; e < 4; ++e)
              if (__float_as_uint(sv[e]) != __float_as_uint(gv[e])) {
                const uint32_t k = atomicAdd(a.dbg, 1u);
                if (k < 16u) {
                  uint32_t* rec = a.dbg + 8 + 8 * k;
                  rec[0] = r; rec[1] = (uint32_t)zc | ((uint32_t)(s2 + 1) << 30); rec[2] = (uint32_t)yy;
                  rec[3] = (uint32_t)(x0 + 4 * lane + e); rec[4] = __float_as_uint(sv[e]); rec[5] = __float_as_uint(gv[e]);
                  rec[6] = smid(); rec[7] = 0xffffffffu;
                }
              }
          }
        }
      }
      // plane pz read for the last time (ym, yp and the edge; zp belongs to plane pz+1)
      mbar_release_after(empty(pz), __float_as_uint(ym.x) ^ __float_as_uint(yp.x) ^ __float_as_uint(ev), zmask, lane);
      float xl = __shfl_up_sync(0xffffffffu, cur.w, 1);
      float xr = __shfl_down_sync(0xffffffffu, cur.x, 1);
      if (lane == 0) xl = ev;
      if (lane == 31) xr = ev;
      const int z = z0 + i;
      float4 o = cur;
      if (z >= 1 && z <= nz - 2) {   // uniform: z-face planes copy the input
        // fp32 round-to-nearest, this association, no FMA contraction: the
        // compiler may contract a*c1 - b*c0 differently per instantiation
        // (native vs persistent), which would break output transparency
        const float vx = point(zm.x, zp.x, ym.x, yp.x, xl, cur.y, cur.x, c0, c1);
        const float vy = point(zm.y, zp.y, ym.y, yp.y, cur.x, cur.z, cur.y, c0, c1);
        const float vz = point(zm.z, zp.z, ym.z, yp.z, cur.y, cur.w, cur.z, c0, c1);
        const float vw = point(zm.w, zp.w, ym.w, yp.w, cur.z, xr, cur.w, c0, c1);
        if (mxy[0]) o.x = vx;
        if (mxy[1]) o.y = vy;
        if (mxy[2]) o.z = vz;
        if (mxy[3]) o.w = vw;
      }
      if (active) *reinterpret_cast<float4*>(po) = o;
      po += pstr;
      zm = cur;
      cur = zp;
    }
  }
};

using StencilTma = StencilTmaT<false>;
using StencilBulk = StencilTmaT<true>;

}  // namespace accel
