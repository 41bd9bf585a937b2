// sad -- Parboil "sad" (H.264 motion-estimation sums of absolute differences;
// SURVEY.md §8(f) f3, one of the 25 Parboil kernels of PAPER.md §7.2 lines
// 853-860).  Three kernels, the three steps of one request (R-solver-8):
//
//   Sad4  VG = one 16x16 macroblock.  The macroblock (16 x 16 u16) and its
//         reference search window ((16 + 2R)^2, coordinates clamped to the
//         frame) are staged in shared memory as u32 pixel PAIRS -- the window
//         twice, once pairing columns (2k, 2k+1) and once (2k+1, 2k+2), so a
//         displacement of either parity reads aligned pairs -- and thread t
//         takes displacements t, t+256, ...: per row 8 __vabsdiffu2 + 8
//         __vadd2 into 16 packed sub-block sums (a 4x4 sum of 8 pairs cannot
//         overflow a 16-bit half), then 16 u16 SADs written as two 16-B stores.
//   Sad8 / Sad16  VG = one macroblock, thread per displacement: 4 (1) sums of
//         the 16 (4) finer SADs (HBM-bound).
// Integer arithmetic: bit-exact against the oracle.
#pragma once
#include "../device/dispatch.cuh"
#include "accel_tenants.h"

namespace accel {

struct SadBase {
  using Args = accel_sad_args;
  static constexpr int kThreads = 256;
  static constexpr uint32_t kChunk = 1;
  static __device__ __forceinline__ uint32_t npos(const Args& a) { return (2 * a.R + 1) * (2 * a.R + 1); }
  static __device__ __forceinline__ uint32_t mb_of(const Args& a, const VirtualBlock& vb) {
    return vb.y * (a.w / 16) + vb.x;
  }
};

struct Sad4 : SadBase {
  static constexpr int kMinBlocks = 4;
  static constexpr int kMaxR = 16;
  static constexpr int kWin = 16 + 2 * kMaxR;            // 48
  static constexpr int kPairs = kWin / 2;                // 24 pairs per window row
  // cur: 16 rows x 8 pairs; win0 / win1: 48 x 24 pairs; win1 offset by 16
  // words so that a warp's even / odd displacements hit disjoint banks
  static constexpr uint32_t kCurWords = 16 * 8, kWinWords = kWin * kPairs;
  static constexpr uint32_t kDynSmem = 4 * (kCurWords + 2 * kWinWords + 16);

  static __device__ __forceinline__ void body(const Args& a, const VirtualBlock& vb, char* smem) {
    uint32_t* cur = reinterpret_cast<uint32_t*>(smem);
    uint32_t* win0 = cur + kCurWords;
    uint32_t* win1 = win0 + kWinWords + 16;
    const int R = (int)a.R, W = 16 + 2 * R, P = W / 2 + 1;   // pairs per staged row (win1 needs W/2)
    const int w = (int)a.w, h = (int)a.h;
    const int x0 = 16 * (int)vb.x, y0 = 16 * (int)vb.y;
    const int t = threadIdx.x;
    if (t < 128) {
      const int row = t >> 3, k = t & 7;
      const uint16_t* c = a.cur + (size_t)(y0 + row) * w + x0 + 2 * k;
      cur[t] = (uint32_t)c[0] | ((uint32_t)c[1] << 16);
    }
    auto px = [&](int r, int c) -> uint32_t {   // window pixel (r, c), clamped to the frame
      const int y = min(max(y0 - R + r, 0), h - 1), x = min(max(x0 - R + c, 0), w - 1);
      return a.ref[(size_t)y * w + x];
    };
    for (int e = t; e < W * P; e += kThreads) {
      const int r = e / P, k = e % P;
      if (2 * k + 1 < W) win0[r * kPairs + k] = px(r, 2 * k) | (px(r, 2 * k + 1) << 16);
      if (2 * k + 2 < W) win1[r * kPairs + k] = px(r, 2 * k + 1) | (px(r, 2 * k + 2) << 16);
    }
    __syncthreads();
    const uint32_t np = npos(a), side = 2 * a.R + 1;
    const size_t base = (size_t)mb_of(a, vb) * np;
    for (uint32_t p = t; p < np; p += kThreads) {
      const uint32_t dy = p / side, dx = p - dy * side;   // window offsets 0..2R
      const uint32_t* wb = (dx & 1u) ? win1 + (dx >> 1) : win0 + (dx >> 1);
      uint32_t s[16];
#pragma unroll
      for (int b = 0; b < 16; ++b) s[b] = 0u;
#pragma unroll   // fully: the sub-block sums s[] must stay in registers
      for (int row = 0; row < 16; ++row) {
        const uint32_t* wr = wb + (row + dy) * kPairs;
        const uint4 c0 = *reinterpret_cast<const uint4*>(cur + row * 8);
        const uint4 c1 = *reinterpret_cast<const uint4*>(cur + row * 8 + 4);
        const int sb = (row >> 2) * 4;
        s[sb + 0] = __vadd2(s[sb + 0], __vadd2(__vabsdiffu2(c0.x, wr[0]), __vabsdiffu2(c0.y, wr[1])));
        s[sb + 1] = __vadd2(s[sb + 1], __vadd2(__vabsdiffu2(c0.z, wr[2]), __vabsdiffu2(c0.w, wr[3])));
        s[sb + 2] = __vadd2(s[sb + 2], __vadd2(__vabsdiffu2(c1.x, wr[4]), __vabsdiffu2(c1.y, wr[5])));
        s[sb + 3] = __vadd2(s[sb + 3], __vadd2(__vabsdiffu2(c1.z, wr[6]), __vabsdiffu2(c1.w, wr[7])));
      }
      uint32_t o[8];
#pragma unroll
      for (int b = 0; b < 8; ++b) {
        const uint32_t lo = (s[2 * b] & 0xffffu) + (s[2 * b] >> 16);
        const uint32_t hi = (s[2 * b + 1] & 0xffffu) + (s[2 * b + 1] >> 16);
        o[b] = lo | (hi << 16);
      }
      uint4* dst = reinterpret_cast<uint4*>(a.sad4 + (base + p) * 16);
      dst[0] = make_uint4(o[0], o[1], o[2], o[3]);
      dst[1] = make_uint4(o[4], o[5], o[6], o[7]);
    }
  }
};

struct Sad8 : SadBase {
  static constexpr int kMinBlocks = 6;
  static constexpr uint32_t kDynSmem = 0;
  static __device__ __forceinline__ void body(const Args& a, const VirtualBlock& vb, char*) {
    const uint32_t np = npos(a);
    const size_t base = (size_t)mb_of(a, vb) * np;
    for (uint32_t p = threadIdx.x; p < np; p += kThreads) {
      const uint4* src = reinterpret_cast<const uint4*>(a.sad4 + (base + p) * 16);
      const uint4 v0 = __ldcs(src), v1 = __ldcs(src + 1);   // sub-blocks 0-7, 8-15 (u16 pairs)
      // 8x8 q = (qx, qy): 4x4 blocks (2qy..2qy+1) x (2qx..2qx+1); pair word k holds blocks 2k, 2k+1
      auto hs = [](uint32_t v) { return (v & 0xffffu) + (v >> 16); };
      const uint32_t q0 = hs(v0.x) + hs(v0.z), q1 = hs(v0.y) + hs(v0.w);
      const uint32_t q2 = hs(v1.x) + hs(v1.z), q3 = hs(v1.y) + hs(v1.w);
      *reinterpret_cast<uint2*>(a.sad8 + (base + p) * 4) = make_uint2(q0 | (q1 << 16), q2 | (q3 << 16));
    }
  }
};

struct Sad16 : SadBase {
  static constexpr int kMinBlocks = 6;
  static constexpr uint32_t kDynSmem = 0;
  static __device__ __forceinline__ void body(const Args& a, const VirtualBlock& vb, char*) {
    const uint32_t np = npos(a);
    const size_t base = (size_t)mb_of(a, vb) * np;
    for (uint32_t p = threadIdx.x; p < np; p += kThreads) {
      const uint2 v = __ldcs(reinterpret_cast<const uint2*>(a.sad8 + (base + p) * 4));
      a.sad16[base + p] = (uint16_t)((v.x & 0xffffu) + (v.x >> 16) + (v.y & 0xffffu) + (v.y >> 16));
    }
  }
};

}  // namespace accel
