// sgemm_tc -- C = A . B^T in fp32 on the 5th-generation tensor cores
// (tcgen05.mma kind::tf32, accumulators in TMEM, operands staged by TMA),
// accurate to ~fp32 through the 3xTF32 split (DESIGN.md R-fp-3):
//   a = a_hi + a_lo,  a_hi = tf32_rn(a),  a_lo = a - a_hi (exact in fp32)
//   C = A_hi.B_hi + A_hi.B_lo + A_lo.B_hi      (fp32 accumulation in TMEM)
// 1xTF32 alone (10-bit mantissa) would miss the 1e-4 bound (~1e-3 error).
//
// Request = two steps: sgemm_split (A and B in one launch), sgemm_tc.
// sgemm_tc VG = one 128 x 256 tile of C; 640 threads (20 warps):
//   warp 0 lane 0  TMA producer  (4 tiles per 32-wide K slab, 2-stage ring, mbarriers)
//   warp 1 lane 0  MMA issuer    (12 x tcgen05.mma 128x256x8 per slab, commit frees the slot)
//   warp 2         TMEM allocator (2 accumulators x 256 columns)
//   warps 4..19    accumulators: every kGroup slabs the MMA issuer switches to
//                  the other TMEM accumulator and these warps add the finished
//                  one into fp32 registers (round-to-nearest), 64 columns x
//                  32 rows each; at the end they store C.
// Why the register accumulation: the tensor core accumulates into TMEM with a
// truncating (biased) fp32 add, so the error grows with the number of MMAs
// chained into one accumulator -- measured 3.3e-4 relative at K = 992 with a
// single chain, above the 1e-4 bound.  Chains of kGroup slabs (24 MMAs) summed
// in fp32 round-to-nearest keep 3xTF32 at fp32-level accuracy for any K.
// Barriers and TMEM are set up per VG (a VG is ~0.8 GFLOP, the setup ~1 us), so
// VGs stay independent as the dispatch contract requires.
#pragma once
#include <cuda.h>

#include "../device/dispatch.cuh"
#include "accel_tenants.h"
#include "tma.cuh"

namespace accel {

namespace tc {

using namespace accel::tma;

// UMMA shared-memory matrix descriptor, K-major, 128-B swizzle: rows of 128 B,
// 8-row groups 1024 B apart (SBO), LBO = 16 B (unused for SW128 K-major),
// version 1 (sm_100), layout type 2 = SWIZZLE_128B.
__device__ __forceinline__ uint64_t umma_desc_k_sw128(uint32_t saddr) {
  return (uint64_t)((saddr >> 4) & 0x3FFFu) | ((uint64_t)1u << 16) | ((uint64_t)(1024u >> 4) << 32) |
         ((uint64_t)1u << 46) | ((uint64_t)2u << 61);
}
__device__ __forceinline__ void mma_tf32(uint32_t d_tmem, uint64_t adesc, uint64_t bdesc, uint32_t idesc,
                                         uint32_t accumulate) {
  asm volatile(
      "{\n\t.reg .pred p;\n\t"
      "setp.ne.b32 p, %4, 0;\n\t"
      "tcgen05.mma.cta_group::1.kind::tf32 [%0], %1, %2, %3, p;\n\t}" ::"r"(d_tmem),
      "l"(adesc), "l"(bdesc), "r"(idesc), "r"(accumulate)
      : "memory");
}
__device__ __forceinline__ void mma_commit(uint32_t bar) {
  asm volatile("tcgen05.commit.cta_group::1.mbarrier::arrive::one.shared::cluster.b64 [%0];" ::"r"(bar)
               : "memory");
}
__device__ __forceinline__ void fence_before() { asm volatile("tcgen05.fence::before_thread_sync;" ::: "memory"); }
__device__ __forceinline__ void fence_after() { asm volatile("tcgen05.fence::after_thread_sync;" ::: "memory"); }

}  // namespace tc

// tf32 split: hi = round-to-nearest tf32 of a, lo = a - hi (exact)
struct SgemmSplit {
  using Args = accel_sgemm_split_args;
  static constexpr int kThreads = 256;
  static constexpr uint32_t kChunk = 2;
  static constexpr int kMinBlocks = 4;
  static constexpr uint32_t kDynSmem = 0;
  static constexpr uint32_t kPerVG = kThreads * 16;   // 4 x float4 per thread
  static __device__ __forceinline__ float hi_of(float a) {
    uint32_t h;
    asm("cvt.rna.tf32.f32 %0, %1;" : "=r"(h) : "f"(a));
    return __uint_as_float(h);
  }
  static __device__ __forceinline__ void body(const Args& a, const VirtualBlock& vb, char*) {
    // VGs [0, g0) split segment 0 (A), the rest segment 1 (B)
    const uint32_t g0 = (uint32_t)((a.n0 + kPerVG - 1) / kPerVG);
    const bool s1 = vb.linear >= g0;
    const float* __restrict__ src = s1 ? a.src1 : a.src0;
    float* __restrict__ hi = s1 ? a.hi1 : a.hi0;
    float* __restrict__ lo = s1 ? a.lo1 : a.lo0;
    const uint64_t n = s1 ? a.n1 : a.n0;
    const uint64_t base = (uint64_t)(s1 ? vb.linear - g0 : vb.linear) * kPerVG;
    if (a.cols != a.ld) {   // K % 4 != 0: rows of the outputs padded to ld
#pragma unroll
      for (int u = 0; u < 16; ++u) {
        const uint64_t i = base + (uint64_t)(u * kThreads + threadIdx.x);
        if (i < n) {
          const uint64_t o = (i / a.cols) * a.ld + i % a.cols;
          const float v = __ldcs(src + i), h = hi_of(v);
          hi[o] = h;
          lo[o] = v - h;
        }
      }
      return;
    }
#pragma unroll
    for (int u = 0; u < 4; ++u) {
      const uint64_t i = base + (uint64_t)(u * kThreads + threadIdx.x) * 4;
      if (i + 3 < n) {
        const float4 v = __ldcs(reinterpret_cast<const float4*>(src + i));
        const float4 h = make_float4(hi_of(v.x), hi_of(v.y), hi_of(v.z), hi_of(v.w));
        *reinterpret_cast<float4*>(hi + i) = h;
        *reinterpret_cast<float4*>(lo + i) = make_float4(v.x - h.x, v.y - h.y, v.z - h.z, v.w - h.w);
      } else {
        for (uint64_t j = i; j < n && j < i + 4; ++j) {
          const float h = hi_of(src[j]);
          hi[j] = h;
          lo[j] = src[j] - h;
        }
      }
    }
  }
};

struct SgemmTc {
  using Args = accel_sgemm_tc_args;
  static constexpr int kThreads = 640;
  static constexpr int kAccWarp0 = 4, kAccWarps = 16;   // warps 4..19
  static constexpr uint32_t kChunk = 1;
  static constexpr int kMinBlocks = 1;
  static constexpr int kBM = 128, kBN = 256, kBK = 32;   // 32 fp32 = one 128-B swizzle row
  static constexpr int kStages = 2;
  static constexpr int kGroup = 2;                        // slabs chained per TMEM accumulator
  static constexpr uint32_t kTileA = kBM * kBK * 4;      // 16 KB
  static constexpr uint32_t kTileB = kBN * kBK * 4;      // 32 KB
  static constexpr uint32_t kStage = 2 * kTileA + 2 * kTileB;   // hi + lo of A and B: 96 KB
  static constexpr uint32_t kTmemCols = 512;             // two 128 x 256 fp32 accumulators
  static constexpr uint32_t kDynSmem = kStages * kStage + 1024 + 1024;  // + barriers, + 1024-B alignment
  // instruction descriptor: D f32, A/B tf32, both K-major, N = 256, M = 128
  static constexpr uint32_t kIdesc = (1u << 4) | (2u << 7) | (2u << 10) | ((uint32_t)(kBN >> 3) << 17) |
                                     ((uint32_t)(kBM >> 4) << 24);

  // add 16 consecutive TMEM columns of this thread's lane into v[0..16)
  static __device__ __forceinline__ void ld16_add(uint32_t taddr, float* v) {
    uint32_t r[16];
    asm volatile(
        "tcgen05.ld.sync.aligned.32x32b.x16.b32 {%0,%1,%2,%3,%4,%5,%6,%7,%8,%9,%10,%11,%12,%13,%14,%15}, [%16];"
        : "=r"(r[0]), "=r"(r[1]), "=r"(r[2]), "=r"(r[3]), "=r"(r[4]), "=r"(r[5]), "=r"(r[6]), "=r"(r[7]),
          "=r"(r[8]), "=r"(r[9]), "=r"(r[10]), "=r"(r[11]), "=r"(r[12]), "=r"(r[13]), "=r"(r[14]), "=r"(r[15])
        : "r"(taddr));
    asm volatile("tcgen05.wait::ld.sync.aligned;" ::: "memory");
#pragma unroll
    for (int j = 0; j < 16; ++j) v[j] += __uint_as_float(r[j]);
  }

  static __device__ __forceinline__ void body(const Args& a, const VirtualBlock& vb, char* smem_raw) {
    using namespace tc;
    const uint32_t warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    char* smem = reinterpret_cast<char*>((reinterpret_cast<uintptr_t>(smem_raw) + 1023) & ~uintptr_t(1023));
    const uint32_t sbase = smem_u32(smem);
    // barriers: full[2], empty[2], accfull[2], accempty[2]: 8 B each
    const uint32_t bars = sbase + kStages * kStage;
    auto full = [&](int s) { return bars + 8u * s; };
    auto empty = [&](int s) { return bars + 16u + 8u * s; };
    auto accfull = [&](int b) { return bars + 32u + 8u * b; };
    auto accempty = [&](int b) { return bars + 48u + 8u * b; };
    uint32_t* tmem_slot = reinterpret_cast<uint32_t*>(smem + kStages * kStage + 128);
    const CUtensorMap* maps = reinterpret_cast<const CUtensorMap*>(a.tmaps);
    const int m0 = (int)vb.y * kBM, n0 = (int)vb.x * kBN;
    const int nk = ((int)a.k + kBK - 1) / kBK;
    const int ng = (nk + kGroup - 1) / kGroup;

    if (threadIdx.x == 0) {
      for (int s = 0; s < kStages; ++s) {
        mbar_init(full(s), 1);
        mbar_init(empty(s), 1);
      }
      for (int b = 0; b < 2; ++b) {
        mbar_init(accfull(b), 1);
        mbar_init(accempty(b), kAccWarps);
      }
      asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
      asm volatile("fence.proxy.async.shared::cta;" ::: "memory");
    }
    if (warp == 2) {
      // no relinquish_alloc_permit: a persistent CTA allocates again for its next VG
      asm volatile("tcgen05.alloc.cta_group::1.sync.aligned.shared::cta.b32 [%0], %1;" ::"r"(smem_u32(tmem_slot)),
                   "r"(kTmemCols)
                   : "memory");
    }
    fence_before();
    __syncthreads();
    fence_after();
    const uint32_t tmem = *tmem_slot;

    if (warp == 0 && lane == 0) {
      // ---- TMA producer
#pragma unroll
      for (int q = 0; q < 4; ++q) tmap_acquire(&maps[q]);
      for (int kb = 0; kb < nk; ++kb) {
        const int s = kb % kStages;
        if (kb >= kStages) mbar_wait(empty(s), ((kb / kStages) - 1) & 1);
        const uint32_t st = sbase + s * kStage;
        mbar_expect_tx(full(s), kStage);
        tma_load_2d(st, &maps[0], kb * kBK, m0, full(s));                       // A_hi
        tma_load_2d(st + kTileA, &maps[1], kb * kBK, m0, full(s));              // A_lo
        tma_load_2d(st + 2 * kTileA, &maps[2], kb * kBK, n0, full(s));          // B_hi
        tma_load_2d(st + 2 * kTileA + kTileB, &maps[3], kb * kBK, n0, full(s)); // B_lo
      }
    } else if (warp == 1 && lane == 0) {
      // ---- MMA issuer: groups of kGroup slabs per accumulator, ping-pong
      for (int g = 0; g < ng; ++g) {
        const int b = g & 1;
        if (g >= 2) mbar_wait(accempty(b), ((g >> 1) - 1) & 1);
        fence_after();
        const uint32_t dacc = tmem + (uint32_t)(b * kBN);
        const int kb1 = min(nk, (g + 1) * kGroup);
        for (int kb = g * kGroup; kb < kb1; ++kb) {
          const int s = kb % kStages;
          mbar_wait(full(s), (kb / kStages) & 1);
          fence_after();
          const uint32_t st = sbase + s * kStage;
#pragma unroll
          for (int ks = 0; ks < kBK / 8; ++ks) {
            const uint32_t koff = ks * 32;   // 8 tf32 = 32 B along the swizzled row
            const uint64_t ahi = umma_desc_k_sw128(st + koff);
            const uint64_t alo = umma_desc_k_sw128(st + kTileA + koff);
            const uint64_t bhi = umma_desc_k_sw128(st + 2 * kTileA + koff);
            const uint64_t blo = umma_desc_k_sw128(st + 2 * kTileA + kTileB + koff);
            mma_tf32(dacc, ahi, bhi, kIdesc, (kb != g * kGroup || ks != 0) ? 1u : 0u);
            mma_tf32(dacc, ahi, blo, kIdesc, 1u);
            mma_tf32(dacc, alo, bhi, kIdesc, 1u);
          }
          // slot s free once these MMAs read it; the last kStages slabs are
          // never refilled, so no arrival outlives the VG (barriers are
          // re-initialised by the next VG)
          if (kb + kStages < nk) mma_commit(empty(s));
        }
        mma_commit(accfull(b));   // accumulator b holds this group's partial sums
      }
    } else if (warp >= (uint32_t)kAccWarp0) {
      // ---- accumulator warps: TMEM lanes 32*(warp%4).., columns 64*h..
      const uint32_t q = warp & 3u, h = (warp - kAccWarp0) >> 2;
      float acc[64];
#pragma unroll
      for (int j = 0; j < 64; ++j) acc[j] = 0.f;
      for (int g = 0; g < ng; ++g) {
        const int b = g & 1;
        mbar_wait(accfull(b), (g >> 1) & 1);
        fence_after();
        const uint32_t taddr = tmem + ((q * 32u) << 16) + (uint32_t)(b * kBN) + h * 64u;
#pragma unroll
        for (int c = 0; c < 4; ++c) ld16_add(taddr + 16u * c, acc + 16 * c);
        fence_before();
        __syncwarp();
        if (lane == 0) mbar_arrive(accempty(b));
      }
      const int row = m0 + (int)(q * 32 + lane);
      const int c0 = n0 + (int)(h * 64);
      if (row < (int)a.m) {
        float* crow = a.c + (size_t)row * a.n;
        if (c0 + 63 < (int)a.n && (a.n & 3) == 0) {
#pragma unroll
          for (int j = 0; j < 64; j += 4)
            *reinterpret_cast<float4*>(crow + c0 + j) = make_float4(acc[j], acc[j + 1], acc[j + 2], acc[j + 3]);
        } else {
#pragma unroll
          for (int j = 0; j < 64; ++j)
            if (c0 + j < (int)a.n) crow[c0 + j] = acc[j];
        }
      }
    }
    fence_before();
    __syncthreads();
    fence_after();
    if (warp == 2)
      asm volatile("tcgen05.dealloc.cta_group::1.sync.aligned.b32 %0, %1;" ::"r"(tmem), "r"(kTmemCols) : "memory");
  }
};

}  // namespace accel

namespace accel {

// sgemm_tc1 -- the same 3xTF32 tensor-core GEMM in ONE step:
// TMA loads the fp32 A and B tiles as they are; the 16 accumulator warps,
// idle between accumulator hand-overs, split every landed slab in place and
// release it to the MMA issuer.  No split launch, no hi/lo operand arrays in
// HBM (4 x 64 MB at 4096^3), one launch per request.  Rows must be 16-B
// aligned for TMA (k % 4 == 0); other k keep the two-step path.
//
//  * hi = x truncated to TF32.  kind::tf32 reads the fp32 word and ignores its
//    low 13 mantissa bits, so the raw tile already IS A_hi / B_hi and only
//    lo = x - hi is written (to a second buffer at the same swizzled offsets:
//    the split is elementwise, the layout is unchanged).  Truncation leaves
//    |lo| < 2^-10 |x| (vs 2^-11 for a round-to-nearest hi), still far inside
//    the 3xTF32 error bound the parity tests hold.
//  * Slabs are 16 wide (64-B rows, SWIZZLE_64B) so that FOUR stages of
//    raw+lo (48 KB each) fit: a slab's conversion waits for the MMA four slabs
//    back, not two (with 32-wide slabs only two 96-KB stages fit and the
//    tensor pipe idled through every TMA + conversion).
//  * The converters read accumulator group h out of TMEM only after they
//    converted the first slab of group h+2 -- by then group h's MMAs are long
//    done, so the hand-over never stalls a conversion, while the MMAs of
//    group h+1 keep the tensor pipe busy.
#ifndef SGEMM1_TRUNC
#define SGEMM1_TRUNC 1
#endif

__device__ __forceinline__ uint64_t umma_desc_k_sw64(uint32_t saddr) {
  // K-major, 64-B swizzle: rows of 64 B, 8-row groups 512 B apart (SBO),
  // version 1 (sm_100), layout type 4 = SWIZZLE_64B
  return (uint64_t)((saddr >> 4) & 0x3FFFu) | ((uint64_t)1u << 16) | ((uint64_t)(512u >> 4) << 32) |
         ((uint64_t)1u << 46) | ((uint64_t)4u << 61);
}

struct SgemmTc1 {
  using Args = accel_sgemm_tc_args;   // tmaps: A, B (raw fp32, box 16 x 128 / 16 x 256, SWIZZLE_64B)
  static constexpr int kThreads = 640;
  static constexpr int kAccWarp0 = 4, kAccWarps = 16;
  static constexpr uint32_t kChunk = 1;
  static constexpr int kMinBlocks = 1;
  static constexpr int kBM = 128, kBN = 256, kBK = 16;
  static constexpr int kStages = 4;
#ifndef SGEMM1_GROUP
#define SGEMM1_GROUP 4
#endif
  static constexpr int kGroup = SGEMM1_GROUP;             // slabs per accumulator hand-over (64 k)
  static constexpr uint32_t kTileA = kBM * kBK * 4;      // 8 KB
  static constexpr uint32_t kTileB = kBN * kBK * 4;      // 16 KB
  // per stage: A (raw = hi), A_lo, B (raw = hi), B_lo
  static constexpr uint32_t kStage = 2 * kTileA + 2 * kTileB;   // 48 KB
  static constexpr uint32_t kTmemCols = 512;
  static constexpr uint32_t kDynSmem = kStages * kStage + 1024 + 1024;
  static constexpr uint32_t kIdesc = SgemmTc::kIdesc;
  static constexpr int kF4 = (int)(kTileA + kTileB) / 16 / 512;   // float4 per converter thread per slab

  static __device__ __forceinline__ float trunc_tf32(float x) { return __uint_as_float(__float_as_uint(x) & 0xFFFFE000u); }

  static __device__ __forceinline__ void body(const Args& a, const VirtualBlock& vb, char* smem_raw) {
    using namespace tc;
    const uint32_t warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    char* smem = reinterpret_cast<char*>((reinterpret_cast<uintptr_t>(smem_raw) + 1023) & ~uintptr_t(1023));
    const uint32_t sbase = smem_u32(smem);
    // barriers: full[S], empty[S], conv[S], accfull[2], accempty[2]
    const uint32_t bars = sbase + kStages * kStage;
    auto full = [&](int s) { return bars + 8u * s; };
    auto empty = [&](int s) { return bars + 8u * (kStages + s); };
    auto conv = [&](int s) { return bars + 8u * (2 * kStages + s); };
    auto accfull = [&](int b) { return bars + 8u * (3 * kStages + b); };
    auto accempty = [&](int b) { return bars + 8u * (3 * kStages + 2 + b); };
    uint32_t* tmem_slot = reinterpret_cast<uint32_t*>(smem + kStages * kStage + 256);
    const CUtensorMap* maps = reinterpret_cast<const CUtensorMap*>(a.tmaps);
    const int m0 = (int)vb.y * kBM, n0 = (int)vb.x * kBN;
    const int nk = ((int)a.k + kBK - 1) / kBK;
    const int ng = (nk + kGroup - 1) / kGroup;
    // stage s: A at +0, A_lo at +kTileA, B at +2 kTileA, B_lo at +2 kTileA + kTileB
    auto st = [&](int s) { return sbase + (uint32_t)s * kStage; };

    if (threadIdx.x == 0) {
      for (int s = 0; s < kStages; ++s) {
        mbar_init(full(s), 1);
        mbar_init(empty(s), 1);
        mbar_init(conv(s), kAccWarps);
      }
      for (int b = 0; b < 2; ++b) {
        mbar_init(accfull(b), 1);
        mbar_init(accempty(b), kAccWarps);
      }
      asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
      asm volatile("fence.proxy.async.shared::cta;" ::: "memory");
    }
    if (warp == 2) {
      asm volatile("tcgen05.alloc.cta_group::1.sync.aligned.shared::cta.b32 [%0], %1;" ::"r"(smem_u32(tmem_slot)),
                   "r"(kTmemCols)
                   : "memory");
    }
    fence_before();
    __syncthreads();
    fence_after();
    const uint32_t tmem = *tmem_slot;

    if (warp == 0 && lane == 0) {
      // ---- TMA producer: raw fp32 slabs of A and B
      tmap_acquire(&maps[0]);
      tmap_acquire(&maps[1]);
      for (int kb = 0; kb < nk; ++kb) {
        const int s = kb % kStages;
        if (kb >= kStages) mbar_wait(empty(s), ((kb / kStages) - 1) & 1);
        mbar_expect_tx(full(s), kTileA + kTileB);
        tma_load_2d(st(s), &maps[0], kb * kBK, m0, full(s));
        tma_load_2d(st(s) + 2 * kTileA, &maps[1], kb * kBK, n0, full(s));
      }
    } else if (warp == 1 && lane == 0) {
      // ---- MMA issuer: waits for the converted slab (conv), not for TMA
      for (int g = 0; g < ng; ++g) {
        const int b = g & 1;
        if (g >= 2) mbar_wait(accempty(b), ((g >> 1) - 1) & 1);
        fence_after();
        const uint32_t dacc = tmem + (uint32_t)(b * kBN);
        const int kb1 = min(nk, (g + 1) * kGroup);
        for (int kb = g * kGroup; kb < kb1; ++kb) {
          const int s = kb % kStages;
          mbar_wait(conv(s), (kb / kStages) & 1);
          fence_after();
          const uint32_t sa = st(s);
#pragma unroll
          for (int ks = 0; ks < kBK / 8; ++ks) {
            const uint32_t koff = ks * 32;   // 8 tf32 = 32 B along the 64-B swizzled row
            const uint64_t ahi = umma_desc_k_sw64(sa + koff);
            const uint64_t alo = umma_desc_k_sw64(sa + kTileA + koff);
            const uint64_t bhi = umma_desc_k_sw64(sa + 2 * kTileA + koff);
            const uint64_t blo = umma_desc_k_sw64(sa + 2 * kTileA + kTileB + koff);
            mma_tf32(dacc, ahi, bhi, kIdesc, (kb != g * kGroup || ks != 0) ? 1u : 0u);
            mma_tf32(dacc, ahi, blo, kIdesc, 1u);
            mma_tf32(dacc, alo, bhi, kIdesc, 1u);
          }
          // the last kStages slabs are never refilled: no arrival outlives the VG
          if (kb + kStages < nk) mma_commit(empty(s));
        }
        mma_commit(accfull(b));
      }
    } else if (warp >= (uint32_t)kAccWarp0) {
      // ---- converters + accumulators
      const uint32_t q = warp & 3u, h = (warp - kAccWarp0) >> 2;
      const uint32_t ct = threadIdx.x - 32u * kAccWarp0;   // 0..511
      float acc[64];
#pragma unroll
      for (int j = 0; j < 64; ++j) acc[j] = 0.f;
      auto split_slab = [&](int kb) {
        const int s = kb % kStages;
        mbar_wait(full(s), (kb / kStages) & 1);
        const uint32_t sa = st(s);
        constexpr uint32_t kA4 = kTileA / 16;   // float4 of A; then those of B
        float4 xs[kF4];
#pragma unroll
        for (int i = 0; i < kF4; ++i) {   // all loads in flight before the first store
          const uint32_t f = ct + 512u * (uint32_t)i;
          xs[i] = lds_f4(f < kA4 ? sa + 16u * f : sa + 2 * kTileA + 16u * (f - kA4));
        }
#pragma unroll
        for (int i = 0; i < kF4; ++i) {
          const uint32_t f = ct + 512u * (uint32_t)i;
          const uint32_t raw = f < kA4 ? sa + 16u * f : sa + 2 * kTileA + 16u * (f - kA4);
          const uint32_t lo = f < kA4 ? raw + kTileA : raw + kTileB;
          const float4 x = xs[i];
#if SGEMM1_TRUNC
          const float4 hi = make_float4(trunc_tf32(x.x), trunc_tf32(x.y), trunc_tf32(x.z), trunc_tf32(x.w));
#else
          const float4 hi = make_float4(SgemmSplit::hi_of(x.x), SgemmSplit::hi_of(x.y), SgemmSplit::hi_of(x.z),
                                        SgemmSplit::hi_of(x.w));
          asm volatile("st.shared.v4.f32 [%0], {%1, %2, %3, %4};" ::"r"(raw), "f"(hi.x), "f"(hi.y), "f"(hi.z),
                       "f"(hi.w)
                       : "memory");
#endif
          asm volatile("st.shared.v4.f32 [%0], {%1, %2, %3, %4};" ::"r"(lo), "f"(x.x - hi.x), "f"(x.y - hi.y),
                       "f"(x.z - hi.z), "f"(x.w - hi.w)
                       : "memory");
        }
        // generic-proxy writes -> read by the tensor cores (async proxy)
        asm volatile("fence.proxy.async.shared::cta;" ::: "memory");
        __syncwarp();
        if (lane == 0) mbar_arrive(conv(s));
      };
      auto accumulate = [&](int g) {
        const int b = g & 1;
        mbar_wait(accfull(b), (g >> 1) & 1);
        fence_after();
        const uint32_t taddr = tmem + ((q * 32u) << 16) + (uint32_t)(b * kBN) + h * 64u;
#pragma unroll
        for (int c = 0; c < 4; ++c) SgemmTc::ld16_add(taddr + 16u * c, acc + 16 * c);
        fence_before();
        __syncwarp();
        if (lane == 0) mbar_arrive(accempty(b));
      };
      int next_acc = 0;
      for (int kb = 0; kb < nk; ++kb) {
        split_slab(kb);
        if (kb % kGroup == 0 && kb / kGroup >= 2) accumulate(next_acc++);
      }
      while (next_acc < ng) accumulate(next_acc++);
      const int row = m0 + (int)(q * 32 + lane);
      const int c0 = n0 + (int)(h * 64);
      if (row < (int)a.m) {
        float* crow = a.c + (size_t)row * a.n;
        if (c0 + 63 < (int)a.n && (a.n & 3) == 0) {
#pragma unroll
          for (int j = 0; j < 64; j += 4)
            *reinterpret_cast<float4*>(crow + c0 + j) = make_float4(acc[j], acc[j + 1], acc[j + 2], acc[j + 3]);
        } else {
#pragma unroll
          for (int j = 0; j < 64; ++j)
            if (c0 + j < (int)a.n) crow[c0 + j] = acc[j];
        }
      }
    }
    fence_before();
    __syncthreads();
    fence_after();
    if (warp == 2)
      asm volatile("tcgen05.dealloc.cta_group::1.sync.aligned.b32 %0, %1;" ::"r"(tmem), "r"(kTmemCols) : "memory");
  }
};

}  // namespace accel
