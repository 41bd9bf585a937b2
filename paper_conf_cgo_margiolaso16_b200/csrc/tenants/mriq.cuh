// mri-q -- non-Cartesian MRI reconstruction Q matrix (Parboil "mri-q":
// ComputePhiMag + ComputeQ).
//
// ComputePhiMag: phiMag_k = phiR^2 + phiI^2 (fp32, round-to-nearest, no FMA:
// bit-exact vs the oracle).  ComputeQ: Qr + i Qi = sum_k phiMag_k
// exp(2 pi i (kx x + ky y + kz z)).  One VG = 256 voxels, one per thread; the
// k-samples are staged through shared memory in tiles of 256.  The phase is
// reduced exactly in "turns": every product k_d * x_d is split into its fp32
// value p and its FMA residual e (p + e exact), p - rint(p) is exact, so
// t = frac(sum) is accurate to ~1e-7 turns although |k.x| reaches ~90 turns
// (plain fp32 would give ~5e-4 relative error in Q, DESIGN.md R-fp-2); then
// one MUFU sin/cos pair.  SFU/ALU-bound.
#pragma once
#include "../device/dispatch.cuh"
#include "accel_tenants.h"

namespace accel {

struct MriqPhiMag {
  using Args = accel_mriq_phimag_args;
  static constexpr int kThreads = 256;
  static constexpr uint32_t kChunk = 4;
  static constexpr int kMinBlocks = 8;
  static constexpr uint32_t kDynSmem = 0;
  static __device__ __forceinline__ void body(const Args& a, const VirtualBlock& vb, char*) {
    const uint32_t k = vb.linear * kThreads + threadIdx.x;
    if (k >= a.numk) return;
    const float r = a.phir[k], i = a.phii[k];
    a.phimag[k] = __fadd_rn(__fmul_rn(r, r), __fmul_rn(i, i));
  }
};

struct MriqQ {
  using Args = accel_mriq_q_args;
  static constexpr int kThreads = 256;
  static constexpr int kTile = 256;
  static constexpr uint32_t kChunk = 1;
  static constexpr int kMinBlocks = 6;
  // useful occupancy in a mix (R-solver-10; scripts/occ_scaling.py, isolated
  // SHARED-static): 6.34 ms at 1 CTA/SM = 92 % of the 5.80 ms at 3..6 -- one
  // CTA per SM nearly saturates the issue slots; its 2nd..6th CTA would take
  // them from a co-runner on the same SM (bfs next to 3 mri-q CTAs/SM: 12x)
  static constexpr uint32_t kMaxCtasPerSm = 1;
  // R-disp-9: four VG ranges per request in SHARED mode.  mri-q's sin/cos keep
  // the MUFU pipe busy, and the pipe goes to the OLDER warps: a persistent
  // mri-q that arrived first starved a later cutcp (rsqrt) for its whole run
  // (C4; scripts/starve.py).  Fresh CTAs every quarter of the request hand
  // the age priority back to its co-runners.
  static constexpr uint32_t kSlices = 4;
  static constexpr uint32_t kDynSmem = 4 * kTile * sizeof(float);

  static __device__ __forceinline__ float frac_prod(float k, float x, float& err) {
    const float p = __fmul_rn(k, x);  // no contraction: p + residual == k*x exactly
    err += __fmaf_rn(k, x, -p);       // exact residual of the product
    return __fsub_rn(p, rintf(p));    // exact
  }

  static __device__ __forceinline__ void body(const Args& a, const VirtualBlock& vb, char* smem) {
    // (kx, ky, kz, phiMag) of a k-sample packed in one 16-B slot: the inner
    // loop issues ONE broadcast LDS.128 per sample instead of four LDS.32.
    // Measured: with four, mri-q's 24 warps/SM kept the LSU queue full and a
    // latency-bound co-runner on the same SM (bfs) ran 10x slower.
    float4* sk = reinterpret_cast<float4*>(smem);
    const int t = threadIdx.x;
    const uint32_t v = vb.linear * kThreads + t;
    const bool have = v < a.numx;
    const float x = have ? __ldg(a.x + v) : 0.f;
    const float y = have ? __ldg(a.y + v) : 0.f;
    const float z = have ? __ldg(a.z + v) : 0.f;
    float qr = 0.f, qi = 0.f;
    const float two_pi = 6.2831853071795864769f;
    for (uint32_t k0 = 0; k0 < a.numk; k0 += kTile) {
      __syncthreads();
      const uint32_t k = k0 + t;
      if (k < a.numk)   // phiMag was written by the previous launch (L2)
        sk[t] = make_float4(__ldg(a.kx + k), __ldg(a.ky + k), __ldg(a.kz + k), __ldcg(a.phimag + k));
      __syncthreads();
      const int n = min(kTile, (int)(a.numk - k0));
#pragma unroll 4
      for (int j = 0; j < n; ++j) {
        const float4 kj = sk[j];
        float err = 0.f;
        const float f = frac_prod(kj.x, x, err) + frac_prod(kj.y, y, err) + frac_prod(kj.z, z, err);
        float tt = f + err;
        tt -= rintf(tt);                 // turns in [-0.5, 0.5]
        float s, c;
        __sincosf(two_pi * tt, &s, &c);
        qr = fmaf(kj.w, c, qr);
        qi = fmaf(kj.w, s, qi);
      }
    }
    if (have) {
      a.qr[v] = qr;
      a.qi[v] = qi;
    }
  }
};

}  // namespace accel
