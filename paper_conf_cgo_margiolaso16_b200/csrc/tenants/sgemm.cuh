// sgemm -- C = A . B^T, fp32 (Parboil "sgemm"),
// A[m][k] and B[n][k] both K-major, C[m][n] row-major.
//
// SIMT version (FP32 FFMA): one VG = one 128 x 128 tile of C, 256 threads
// with an 8 x 8 register tile each, K staged through double-buffered shared
// memory in slabs of 8 (transposed on the way in), next slab prefetched into
// registers while the current one is consumed.  DESIGN.md §sgemm: the
// tcgen05 (TMEM, 3xTF32) path is the tensor-core kernel; this one is the
// portable fp32 body with the same VG decomposition.
#pragma once
#include "../device/dispatch.cuh"
#include "accel_tenants.h"

namespace accel {

struct Sgemm {
  using Args = accel_sgemm_args;
  static constexpr int kThreads = 256;
  static constexpr int kBM = 128, kBN = 128, kBK = 8, kPad = 4;
  static constexpr uint32_t kChunk = 1;
  static constexpr int kMinBlocks = 2;
  static constexpr uint32_t kDynSmem = 2 * 2 * kBK * (kBM + kPad) * sizeof(float);  // 16.5 KB

  static __device__ __forceinline__ void body(const Args& a, const VirtualBlock& vb, char* smem) {
    float* As = reinterpret_cast<float*>(smem);              // [2][kBK][kBM + kPad]
    float* Bs = As + 2 * kBK * (kBM + kPad);                 // [2][kBK][kBN + kPad]
    const int t = threadIdx.x;
    const int tx = t & 15, ty = t >> 4;
    const int m0 = (int)vb.y * kBM, n0 = (int)vb.x * kBN;
    const int M = (int)a.m, N = (int)a.n, K = (int)a.k;
    // loader: thread t owns row (t >> 1) of the A and B slabs, k-offset 4*(t & 1)
    const int lr = t >> 1, lk = (t & 1) * 4;
    const float* ag = a.a + (size_t)(m0 + lr) * K + lk;
    const float* bg = a.b + (size_t)(n0 + lr) * K + lk;
    const bool arow = m0 + lr < M, brow = n0 + lr < N;
    auto ld = [&](const float* p, bool row_ok, int k) -> float4 {
      if (row_ok && k + lk + 3 < K) return __ldg(reinterpret_cast<const float4*>(p + k));
      float4 r = make_float4(0.f, 0.f, 0.f, 0.f);
      if (row_ok) {
        if (k + lk + 0 < K) r.x = __ldg(p + k + 0);
        if (k + lk + 1 < K) r.y = __ldg(p + k + 1);
        if (k + lk + 2 < K) r.z = __ldg(p + k + 2);
      }
      return r;
    };
    auto st = [&](float* S, int buf, float4 v) {
      float* s = S + buf * kBK * (kBM + kPad) + lk * (kBM + kPad) + lr;
      s[0] = v.x;
      s[(kBM + kPad)] = v.y;
      s[2 * (kBM + kPad)] = v.z;
      s[3 * (kBM + kPad)] = v.w;
    };
    float acc[8][8];
#pragma unroll
    for (int i = 0; i < 8; ++i)
#pragma unroll
      for (int j = 0; j < 8; ++j) acc[i][j] = 0.f;

    float4 ra = ld(ag, arow, 0), rb = ld(bg, brow, 0);
    st(As, 0, ra);
    st(Bs, 0, rb);
    __syncthreads();
    const int nk = (K + kBK - 1) / kBK;
    for (int kt = 0; kt < nk; ++kt) {
      const int buf = kt & 1;
      if (kt + 1 < nk) {
        ra = ld(ag, arow, (kt + 1) * kBK);
        rb = ld(bg, brow, (kt + 1) * kBK);
      }
      const float* Ab = As + buf * kBK * (kBM + kPad);
      const float* Bb = Bs + buf * kBK * (kBN + kPad);
#pragma unroll
      for (int kk = 0; kk < kBK; ++kk) {
        const float4 a0 = *reinterpret_cast<const float4*>(Ab + kk * (kBM + kPad) + ty * 4);
        const float4 a1 = *reinterpret_cast<const float4*>(Ab + kk * (kBM + kPad) + 64 + ty * 4);
        const float4 b0 = *reinterpret_cast<const float4*>(Bb + kk * (kBN + kPad) + tx * 4);
        const float4 b1 = *reinterpret_cast<const float4*>(Bb + kk * (kBN + kPad) + 64 + tx * 4);
        const float av[8] = {a0.x, a0.y, a0.z, a0.w, a1.x, a1.y, a1.z, a1.w};
        const float bv[8] = {b0.x, b0.y, b0.z, b0.w, b1.x, b1.y, b1.z, b1.w};
#pragma unroll
        for (int i = 0; i < 8; ++i)
#pragma unroll
          for (int j = 0; j < 8; ++j) acc[i][j] = fmaf(av[i], bv[j], acc[i][j]);
      }
      if (kt + 1 < nk) {
        st(As, buf ^ 1, ra);
        st(Bs, buf ^ 1, rb);
      }
      __syncthreads();
    }
    // rows ty*4 + {0..3} and 64 + ty*4 + {0..3}; cols tx*4 + {0..3} and 64 + tx*4 + {0..3}
#pragma unroll
    for (int i = 0; i < 8; ++i) {
      const int r = m0 + (i < 4 ? ty * 4 + i : 64 + ty * 4 + i - 4);
      if (r >= M) continue;
      float* crow = a.c + (size_t)r * N;
#pragma unroll
      for (int h = 0; h < 2; ++h) {
        const int c = n0 + h * 64 + tx * 4;
        if (c + 3 < N && (N & 3) == 0) {
          *reinterpret_cast<float4*>(crow + c) =
              make_float4(acc[i][4 * h], acc[i][4 * h + 1], acc[i][4 * h + 2], acc[i][4 * h + 3]);
        } else {
#pragma unroll
          for (int j = 0; j < 4; ++j)
            if (c + j < N) crow[c + j] = acc[i][4 * h + j];
        }
      }
    }
  }
};

}  // namespace accel
