// stencil -- 7-point 3-D Jacobi sweep (Parboil "stencil", named in PAPER.md
// lines 290-291), fp32, A[z][y][x] with x fastest.
//
// One VG = a 128 x 8 x 8 (x, y, z) tile; 256 threads = 8 warps, warp w owns
// row y0+w, lane l owns x0+4l..x0+4l+3 (one 16-B vector).  The tile is walked
// along z (fully unrolled: ring slots and group counts are compile-time).
// Plane tiles (10 rows y0-1..y0+8 x 136 columns x0-4..x0+131: the tile plus
// its y and x halos) are staged in shared memory by cp.async (16-B LDGSTS,
// L2-only), kD planes ahead into a ring of kR slots, one commit group per
// plane and ONE __syncthreads per plane.  Out-of-volume pieces are
// zero-filled (src-size 0); they only feed face cells, which copy the input.
// The column z-1, z, z+1 of each thread lives in registers; y neighbours and
// the two x edges come from the staged plane, inner x neighbours from warp
// shuffles.  Occupancy is set by shared memory (6 CTAs/SM, ~130 KB in flight
// per SM).  Algorithmic traffic: 8 B per point per sweep.
//
// The TMA staging of the same tiles (stencil_tma.cuh) once drifted next to
// the bfs tenant: a ring-slot release raced its own ld.shared (root cause
// and fix in DESIGN.md, "stencil staging"; tma::mbar_release_after).  Fixed,
// it is correct but not faster than this cp.async kernel, which stays the
// default.
#pragma once
#include "../device/dispatch.cuh"
#include "accel_tenants.h"
#include "tma.cuh"

namespace accel {

// kAligned: nx % 4 == 0 (kernel "stencil": every row starts 16-B aligned).
// !kAligned: any nx (kernel "stencil_x"): the same tile staged with 4-B
// cp.async copies, each column checked against nx, outputs stored per
// element.  Two kernels rather than a branch: the ragged path's registers
// would otherwise count against the aligned one (it spilled).
#ifndef STENCIL_KD
#define STENCIL_KD 4
#endif
// kDepth: planes in flight beyond z+1 ("stencil_deep": the whole 10-plane
// tile in flight per VG -- more bytes in flight per CTA for a small share)
// kTZv: planes per VG ("stencil_z16": 16 -- the ring's refill at the start of
// every VG and the two z-halo planes are paid per 16 planes instead of 8)
template <bool kAligned, int kDepth = STENCIL_KD, int kTZv = 8>
struct StencilT {
  using Args = accel_stencil_args;
  static constexpr int kThreads = 256;
  static constexpr int kTX = 128, kTY = 8, kTZ = kTZv;
  static constexpr uint32_t kChunk = 1;
  // the ragged path needs a few more registers; the deep ring (55 KB) fits 4 per SM
#ifndef STENCIL_MINB
#define STENCIL_MINB 5
#endif
  static constexpr int kMinBlocks = (kAligned && kDepth <= 4) ? STENCIL_MINB : 4;
  static constexpr int kRows = kTY + 2;                 // y halo
  static constexpr int kCols = kTX + 8;                 // x0-4 .. x0+131 (16-B multiples)
  static constexpr uint32_t kPlaneBytes = kRows * kCols * 4;          // 5440
  static constexpr uint32_t kSlot = (kPlaneBytes + 127) / 128 * 128;  // 5504
  static constexpr int kD = kDepth;                     // planes in flight beyond z+1
  static constexpr int kR = kD + 2;                     // ring slots
#ifndef STENCIL_MBAR
#define STENCIL_MBAR 0
#endif
  // kMbar: per-slot mbarriers instead of one __syncthreads per plane --
  // "full" completes when all 256 threads' cp.async pieces of the plane landed
  // (cp.async.mbarrier.arrive.noinc), "empty" when all 8 warps released it, so
  // warps drift apart by up to a plane instead of meeting at every plane.
  static constexpr bool kMbar = STENCIL_MBAR != 0 && kTZv + 2 <= 2 * (kDepth + 2);   // (z16: barrier path)
  static_assert(!kMbar || kTZ + 2 <= 2 * kR, "a slot is filled at most twice per VG (parities 0, 1)");
  static constexpr uint32_t kBarBytes = kMbar ? 2 * kR * 8 : 0;
  static constexpr uint32_t kDynSmem = kR * kSlot + kBarBytes + 128;   // + alignment

  // cp.async (LDGSTS, 16 B per copy, L2-only .cg) staging: every thread
  // copies <= 2 of the 340 16-B pieces of a plane tile; out-of-volume pieces are
  // zero-filled (src-size 0).  One commit group per plane, planes kD ahead.
  // ((((((zm + zp) + ym) + yp) + xm) + xp) * c1) - (c * c0), each step fp32 RN
  static __device__ __forceinline__ float point(float zm, float zp, float ym, float yp, float xm, float xp, float c,
                                                float c0, float c1) {
    const float s = __fadd_rn(__fadd_rn(__fadd_rn(__fadd_rn(__fadd_rn(zm, zp), ym), yp), xm), xp);
    return __fsub_rn(__fmul_rn(s, c1), __fmul_rn(c, c0));
  }

  static __device__ __forceinline__ void body(const Args& a, const VirtualBlock& vb, char* smem_raw) {
    using namespace tma;
    const uint32_t r = vb.launch_idx;
    const float* __restrict__ in = r == 0 ? a.a0 : ((r & 1) ? a.buf0 : a.buf1);
    float* __restrict__ out = (r & 1) ? a.buf1 : a.buf0;
    const int nx = (int)a.nx, ny = (int)a.ny, nz = (int)a.nz;
    const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
    const int x0 = (int)vb.x * kTX;
    const int y0 = (int)vb.y * kTY;
    const int y = y0 + warp;
    const int z0 = (int)vb.z * kTZ;
    const int nzt = min(kTZ, nz - z0);
    const int nplanes = nzt + 2;
    const uint32_t sbase = (smem_u32(smem_raw) + 127u) & ~127u;
    const uint32_t fullb = sbase + kR * kSlot, emptyb = fullb + kR * 8;   // kMbar only
    if constexpr (kMbar) {
      // re-armed per VG: every plane of the previous VG was waited "full" by
      // every warp (no async arrival pending) and the dispatch barrier closed it
      if (threadIdx.x == 0) {
#pragma unroll
        for (int q = 0; q < kR; ++q) {
          mbar_init(fullb + 8u * q, kThreads);
          mbar_init(emptyb + 8u * q, kThreads / 32);
        }
      }
      __syncthreads();
    }
    // my two pieces: e = tid, tid + 256 (< 340); piece e = row e / 34, 16-B column e % 34.
    // The source address of a piece is fixed per VG up to the plane offset
    // p * nx * ny, so it is computed once here; per plane only the (uniform)
    // z range decides whether the piece is read or zero-filled.  Rows y0-1 and
    // y0+8 outside [0, ny) are zero-filled: they only feed y-face cells, which
    // copy the input.
    constexpr int kPieces = kRows * (kCols / 4);
    const int e0 = threadIdx.x, e1 = threadIdx.x + kThreads;
    const bool has1 = e1 < kPieces;
    const int rr0 = e0 / (kCols / 4), c0x = x0 - 4 + 4 * (e0 % (kCols / 4));
    const int rr1 = e1 / (kCols / 4), c1x = x0 - 4 + 4 * (e1 % (kCols / 4));
    const int ys0 = y0 - 1 + rr0, ys1 = y0 - 1 + rr1;
    const bool okxy0 = c0x >= 0 && c0x < nx && ys0 >= 0 && ys0 < ny;
    const bool okxy1 = has1 && c1x >= 0 && c1x < nx && ys1 >= 0 && ys1 < ny;
    const long long pstr = (long long)nx * ny;
    // plane p = z0 - 1 + p; offsets of plane 0 (may be negative: only used when valid)
    const long long off0 = (long long)(z0 - 1) * pstr + (long long)ys0 * nx + c0x;
    const long long off1 = (long long)(z0 - 1) * pstr + (long long)ys1 * nx + c1x;
    const uint32_t soff0 = 16u * (uint32_t)e0, soff1 = 16u * (uint32_t)e1;
    // aligned path: per-piece byte pointers to plane 0, advanced one plane per
    // issue.  A piece outside the x/y range reads 0 bytes from its clamped
    // (in-bounds) position, so every pointer advances by the same plane stride
    const long long pbytes = 4 * pstr;
    auto clamped = [&](int ys, int cx) {
      const int yc = min(max(ys, 0), ny - 1), xc = min(max(cx, 0), nx - 4);
      return reinterpret_cast<const char*>(in + ((long long)(z0 - 1) * pstr + (long long)yc * nx + xc));
    };
    const char* g0 = clamped(ys0, c0x);
    const char* g1 = clamped(ys1, c1x);
    // ragged x (nx % 4 != 0): a piece is four 4-B copies, column c + j read
    // only when c + j < nx (c >= 0 is all-or-nothing: x0 - 4 is a multiple of 4)
    auto piece4 = [&](uint32_t dst, long long off, int cx, bool okyz) {
#pragma unroll
      for (int j = 0; j < 4; ++j) {
        const bool ok = okyz && cx >= 0 && cx + j < nx;
        const float* src = ok ? in + (off + j) : in;
        asm volatile("cp.async.ca.shared.global [%0], [%1], 4, %2;" ::"r"(dst + 4u * j), "l"(src), "r"(ok ? 4 : 0)
                     : "memory");
      }
    };
    auto issue = [&](int p) {
      const uint32_t dst = sbase + (uint32_t)(p % kR) * kSlot;
      const int zs = z0 - 1 + p;
      const bool zok = (unsigned)zs < (unsigned)nz;   // uniform
      if constexpr (!kAligned) {
        piece4(dst + soff0, off0 + (long long)p * pstr, c0x, zok && ys0 >= 0 && ys0 < ny);
        if (has1) piece4(dst + soff1, off1 + (long long)p * pstr, c1x, zok && ys1 >= 0 && ys1 < ny);
        return;
      }
      // running source pointers (issue() is called for p = 0, 1, 2, ... in
      // order): one 64-bit add per piece and plane instead of recomputing
      // the offset (SASS: ~14 integer instructions per piece and plane)
      const char* s0 = zok ? g0 : reinterpret_cast<const char*>(in);
      asm volatile("cp.async.cg.shared.global [%0], [%1], 16, %2;" ::"r"(dst + soff0), "l"(s0),
                   "r"((zok && okxy0) ? 16 : 0)
                   : "memory");
      g0 += pbytes;
      if (has1) {
        const char* s1 = zok ? g1 : reinterpret_cast<const char*>(in);
        asm volatile("cp.async.cg.shared.global [%0], [%1], 16, %2;" ::"r"(dst + soff1), "l"(s1),
                     "r"((zok && okxy1) ? 16 : 0)
                     : "memory");
        g1 += pbytes;
      }
    };
    auto commit = [] { asm volatile("cp.async.commit_group;" ::: "memory"); };
    auto arrive_full = [&](int p) {   // fires when this thread's copies so far landed
      asm volatile("cp.async.mbarrier.arrive.noinc.shared::cta.b64 [%0];" ::"r"(fullb + 8u * (uint32_t)(p % kR))
                   : "memory");
    };
    // prologue: planes 0 .. kD+1 (one group each, empty groups past the tile)
#pragma unroll
    for (int p = 0; p < kD + 2; ++p) {
      if constexpr (kMbar) {
        if (p < nplanes) {
          issue(p);
          arrive_full(p);
        }
      } else {
        if (p < nplanes) issue(p);
        commit();
      }
    }
    auto slot = [&](int p) { return sbase + (uint32_t)(p % kR) * kSlot; };

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
    float4 zm, cur;
    if constexpr (kMbar) {
      mbar_wait(fullb, 0);
      mbar_wait(fullb + 8u, 0);
      zm = lds_f4(slot(0) + own);
      cur = lds_f4(slot(1) + own);
      mbar_release_after(emptyb, __float_as_uint(zm.x), (uint32_t)nz >> 31, lane);   // plane 0 released
    } else {
      // planes 0 and 1 landed (groups 0, 1 of kD + 2 committed)
      asm volatile("cp.async.wait_group %0;" ::"n"(kD) : "memory");
      __syncthreads();
      zm = lds_f4(slot(0) + own);
      cur = lds_f4(slot(1) + own);
    }
    float* po = out + ((size_t)z0 * ny + y) * nx + x0 + 4 * lane;
#pragma unroll
    for (int i = 0; i < kTZ; ++i) {
      if (i >= nzt) break;
      const int pz = i + 1;   // plane pz (= z) is `cur`; plane pz+1 must have landed
      // groups committed: kD + 2 + i; plane pz+1 is group i+2, so at most
      // kD - 1 may still be pending
      if constexpr (kMbar) {
        mbar_wait(fullb + 8u * (uint32_t)((pz + 1) % kR), (uint32_t)(((pz + 1) / kR) & 1));
      } else {
        asm volatile("cp.async.wait_group %0;" ::"n"(kD - 1) : "memory");
        __syncthreads();        // plane pz+1 visible; every thread done with iteration i-1
        // refill the slot of plane pz-1 (last read in iteration i-1) with plane pz+kD+1
        if (pz + kD + 1 < nplanes) issue(pz + kD + 1);
        commit();
      }
      const uint32_t P = slot(pz);
      const float4 zp = lds_f4(slot(pz + 1) + own);
      const float4 ym = lds_f4(P + own - 4u * kCols);
      const float4 yp = lds_f4(P + own + 4u * kCols);
      const float ev = lds_f32(P + edge);
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
      if constexpr (kMbar) {
        // plane pz read for the last time (ym, yp, edge): release it; then
        // refill the slot of plane pz-1 (released by every warp after its
        // iteration i-1) with plane pz+kD+1
        mbar_release_after(emptyb + 8u * (uint32_t)(pz % kR),
                           __float_as_uint(ym.x) ^ __float_as_uint(yp.x) ^ __float_as_uint(ev), (uint32_t)nz >> 31, lane);
        if (pz + kD + 1 < nplanes) {
          mbar_wait(emptyb + 8u * (uint32_t)((pz - 1) % kR), 0u);
          issue(pz + kD + 1);
          arrive_full(pz + kD + 1);
        }
      }
      if constexpr (kAligned) {
        if (active) *reinterpret_cast<float4*>(po) = o;
      } else if (active) {
        const int xr0 = nx - (x0 + 4 * lane);   // >= 1 elements of this vector in range
        po[0] = o.x;
        if (xr0 > 1) po[1] = o.y;
        if (xr0 > 2) po[2] = o.z;
        if (xr0 > 3) po[3] = o.w;
      }
      po += pstr;
      zm = cur;
      cur = zp;
    }
    asm volatile("cp.async.wait_all;" ::: "memory");
    __syncthreads();   // the CTA's next VG reuses the ring
  }

};

// stencil2 -- the same sweep, tile 128 x 16 x 8: every warp owns TWO rows
// (y0 + w and y0 + w + 8), so a thread updates 8 points per plane instead of 4.
// Measured on StencilT (SASS + ncu): ~100 instructions per plane per thread of
// which only 32 are the stencil's arithmetic, issue 70 % active -- the plane's
// fixed work (cp.async issue, barrier, shuffles, address updates, the output
// selects) dominated.  Here it is paid once per 8 points, and the y halo costs
// 18/16 instead of 10/8 staged rows.  18 x 136 plane tiles (9.6 KB), kD planes
// ahead in a ring of kD + 2 slots (4 CTAs/SM at kD = 3: ~118 KB in flight per
// SM); 612 16-B pieces per plane, <= 3 per thread.  nx % 4 == 0 only (the
// ragged path stays StencilT<false>).  Same per-point op sequence as StencilT
// (point()), so the output is bit-identical.
template <int kDepth>
struct Stencil2T {
  using Args = accel_stencil_args;
  static constexpr int kThreads = 256;
  static constexpr int kRPW = 2;                        // rows per warp
  static constexpr int kTX = 128, kTY = 8 * kRPW, kTZ = 8;
  static constexpr uint32_t kChunk = 1;
  static constexpr int kMinBlocks = 4;
  static constexpr int kRows = kTY + 2;                 // y halo
  static constexpr int kCols = kTX + 8;                 // x0-4 .. x0+131
  static constexpr int kPR = kCols / 4;                 // 16-B pieces per row (34)
  static constexpr int kPieces = kRows * kPR;           // 612
  static constexpr int kPPT = (kPieces + kThreads - 1) / kThreads;   // 3
  static_assert((kPPT - 1) * kThreads <= kPieces, "all but the last piece of a thread exist");
  static constexpr uint32_t kPlaneBytes = kRows * kCols * 4;          // 9792
  static constexpr uint32_t kSlot = (kPlaneBytes + 127) / 128 * 128;  // 9856
  static constexpr int kD = kDepth;
  static constexpr int kR = kD + 2;
  static constexpr uint32_t kDynSmem = kR * kSlot + 128;

  static __device__ __forceinline__ void body(const Args& a, const VirtualBlock& vb, char* smem_raw) {
    using namespace tma;
    const uint32_t r = vb.launch_idx;
    const float* __restrict__ in = r == 0 ? a.a0 : ((r & 1) ? a.buf0 : a.buf1);
    float* __restrict__ out = (r & 1) ? a.buf1 : a.buf0;
    const int nx = (int)a.nx, ny = (int)a.ny, nz = (int)a.nz;
    const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
    const int x0 = (int)vb.x * kTX;
    const int y0 = (int)vb.y * kTY;
    const int z0 = (int)vb.z * kTZ;
    const int nzt = min(kTZ, nz - z0);
    const int nplanes = nzt + 2;
    const uint32_t sbase = (smem_u32(smem_raw) + 127u) & ~127u;
    const long long pstr = (long long)nx * ny;
    const long long pbytes = 4 * pstr;
    // my pieces q: e = tid + 256 q -> staged row e / 34, 16-B column e % 34;
    // running source pointers to plane 0 (clamped in-bounds; an out-of-range
    // piece reads 0 bytes and zero-fills)
    const char* g[kPPT];
    bool okxy[kPPT];
#pragma unroll
    for (int q = 0; q < kPPT; ++q) {
      const int e = threadIdx.x + kThreads * q;
      const int rr = e / kPR, cx = x0 - 4 + 4 * (e % kPR), ys = y0 - 1 + rr;
      okxy[q] = (q < kPPT - 1 || e < kPieces) && cx >= 0 && cx < nx && ys >= 0 && ys < ny;
      const int yc = min(max(ys, 0), ny - 1), xc = min(max(cx, 0), nx - 4);
      g[q] = reinterpret_cast<const char*>(in + ((long long)(z0 - 1) * pstr + (long long)yc * nx + xc));
    }
    const bool has_last = threadIdx.x + kThreads * (kPPT - 1) < kPieces;
    auto issue = [&](int p) {
      const uint32_t dst = sbase + (uint32_t)(p % kR) * kSlot + 16u * threadIdx.x;
      const bool zok = (unsigned)(z0 - 1 + p) < (unsigned)nz;   // uniform
#pragma unroll
      for (int q = 0; q < kPPT; ++q) {
        if (q == kPPT - 1 && !has_last) break;
        const char* src = zok ? g[q] : reinterpret_cast<const char*>(in);
        asm volatile("cp.async.cg.shared.global [%0], [%1], 16, %2;" ::"r"(dst + 16u * kThreads * q), "l"(src),
                     "r"((zok && okxy[q]) ? 16 : 0)
                     : "memory");
        g[q] += pbytes;
      }
    };
    auto commit = [] { asm volatile("cp.async.commit_group;" ::: "memory"); };
#pragma unroll
    for (int p = 0; p < kD + 2; ++p) {
      if (p < nplanes) issue(p);
      commit();
    }
    auto slot = [&](int p) { return sbase + (uint32_t)(p % kR) * kSlot; };

    const int xl0 = x0 + 4 * lane;
    const bool xin = xl0 < nx;
    bool xint[4];
#pragma unroll
    for (int e = 0; e < 4; ++e) xint[e] = xl0 + e >= 1 && xl0 + e <= nx - 2;
    const float c0 = a.c0, c1 = a.c1;
    uint32_t own[kRPW], edge[kRPW];
    bool active[kRPW], yint[kRPW];
#pragma unroll
    for (int j = 0; j < kRPW; ++j) {
      const int row = warp + 8 * j;   // tile row; staged row row + 1
      const int y = y0 + row;
      own[j] = 4u * (uint32_t)((row + 1) * kCols + 4 + 4 * lane);
      edge[j] = 4u * (uint32_t)((row + 1) * kCols + (lane == 31 ? 4 + kTX : 3));
      active[j] = xin && y < ny;
      yint[j] = y >= 1 && y <= ny - 2;
    }
    float4 zm[kRPW], cur[kRPW];
    asm volatile("cp.async.wait_group %0;" ::"n"(kD) : "memory");
    __syncthreads();
#pragma unroll
    for (int j = 0; j < kRPW; ++j) {
      zm[j] = lds_f4(slot(0) + own[j]);
      cur[j] = lds_f4(slot(1) + own[j]);
    }
    float* po = out + ((size_t)z0 * ny + (y0 + warp)) * nx + xl0;
    const size_t row8 = (size_t)8 * nx;
#pragma unroll
    for (int i = 0; i < kTZ; ++i) {
      if (i >= nzt) break;
      const int pz = i + 1;
      asm volatile("cp.async.wait_group %0;" ::"n"(kD - 1) : "memory");
      __syncthreads();
      if (pz + kD + 1 < nplanes) issue(pz + kD + 1);
      commit();
      const uint32_t P = slot(pz), Z = slot(pz + 1);
      const int z = z0 + i;
      const bool zint = z >= 1 && z <= nz - 2;   // uniform: z-face planes copy the input
#pragma unroll
      for (int j = 0; j < kRPW; ++j) {
        const float4 zp = lds_f4(Z + own[j]);
        const float4 ym = lds_f4(P + own[j] - 4u * kCols);
        const float4 yp = lds_f4(P + own[j] + 4u * kCols);
        const float ev = lds_f32(P + edge[j]);
        const float4 c = cur[j];
        float xl = __shfl_up_sync(0xffffffffu, c.w, 1);
        float xr = __shfl_down_sync(0xffffffffu, c.x, 1);
        if (lane == 0) xl = ev;
        if (lane == 31) xr = ev;
        float4 o = c;
        if (zint && yint[j]) {
          const float vx = StencilT<true>::point(zm[j].x, zp.x, ym.x, yp.x, xl, c.y, c.x, c0, c1);
          const float vy = StencilT<true>::point(zm[j].y, zp.y, ym.y, yp.y, c.x, c.z, c.y, c0, c1);
          const float vz = StencilT<true>::point(zm[j].z, zp.z, ym.z, yp.z, c.y, c.w, c.z, c0, c1);
          const float vw = StencilT<true>::point(zm[j].w, zp.w, ym.w, yp.w, c.z, xr, c.w, c0, c1);
          if (xint[0]) o.x = vx;
          if (xint[1]) o.y = vy;
          if (xint[2]) o.z = vz;
          if (xint[3]) o.w = vw;
        }
        if (active[j]) *reinterpret_cast<float4*>(po + j * row8) = o;
        zm[j] = c;
        cur[j] = zp;
      }
      po += pstr;
    }
    asm volatile("cp.async.wait_all;" ::: "memory");
    __syncthreads();   // the CTA's next VG reuses the ring
  }
};

#ifndef STENCIL2_KD
#define STENCIL2_KD 3
#endif
using Stencil = StencilT<true>;
using StencilX = StencilT<false>;
using StencilDeep = StencilT<true, 8>;
using StencilZ16 = StencilT<true, STENCIL_KD, 16>;
using Stencil2 = Stencil2T<STENCIL2_KD>;

}  // namespace accel
