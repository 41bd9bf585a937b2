// intercept_app.cu -- an application that knows nothing about accelOS beyond
// declaring its kernels with ACCEL_WRAP_KERNEL (include/accel_wrap.cuh).  It
// launches two kernels on two streams with <<<>>> and checks their results on
// the host.  Run plainly it uses the hardware's standard sharing; run with
// LD_PRELOAD=libaccel_intercept.so its launches become accelOS requests
// (persistent CTAs, fair quotas) -- same results.
//
//   nvcc -gencode arch=compute_100a,code=sm_100a -cudart shared -I include examples/intercept_app.cu
#include <cstdio>
#include <cstdlib>
#include <vector>

#include "accel_wrap.cuh"

// saxpy over n floats: HBM-bound, one 1024-element tile per CTA
struct SaxpyArgs {
  const float* x;
  float* y;
  float a;
  uint32_t n;
};
struct Saxpy {
  using Args = SaxpyArgs;
  static constexpr int kThreads = 256;
  static constexpr uint32_t kChunk = 1;
  static constexpr uint32_t kDynSmem = 0;
  static __device__ __forceinline__ void body(const Args& p, const accel::VirtualBlock& vb, char*) {
    for (uint32_t k = 0; k < 4; ++k) {
      const uint32_t i = vb.linear * 1024u + k * 256u + threadIdx.x;
      if (i < p.n) p.y[i] = __fadd_rn(__fmul_rn(p.a, p.x[i]), p.y[i]);
    }
  }
};

// an ALU-bound kernel: iterate a logistic map per element (one CTA per 256 elements)
struct LogisticArgs {
  float* v;
  uint32_t n, iters;
};
struct Logistic {
  using Args = LogisticArgs;
  static constexpr int kThreads = 256;
  static constexpr uint32_t kChunk = 1;
  static constexpr uint32_t kDynSmem = 0;
  static __device__ __forceinline__ void body(const Args& p, const accel::VirtualBlock& vb, char*) {
    const uint32_t i = vb.linear * 256u + threadIdx.x;
    if (i >= p.n) return;
    float x = p.v[i];
    for (uint32_t t = 0; t < p.iters; ++t) x = __fmul_rn(__fmul_rn(3.7f, x), __fsub_rn(1.0f, x));
    p.v[i] = x;
  }
};

ACCEL_WRAP_KERNEL(saxpy_kernel, Saxpy)
ACCEL_WRAP_KERNEL(logistic_kernel, Logistic)

#define CK(x)                                                                      \
  do {                                                                             \
    cudaError_t e = (x);                                                           \
    if (e != cudaSuccess) {                                                        \
      std::fprintf(stderr, "%s: %s\n", #x, cudaGetErrorString(e));                 \
      return 2;                                                                    \
    }                                                                              \
  } while (0)

int main() {
  const uint32_t n = 1u << 24, m = 1u << 20, iters = 2000, reps = 3;
  std::vector<float> hx(n), hy(n), hv(m);
  for (uint32_t i = 0; i < n; ++i) {
    hx[i] = (float)(i % 1000) * 1e-3f;
    hy[i] = (float)(i % 7);
  }
  for (uint32_t i = 0; i < m; ++i) hv[i] = 0.1f + 0.8f * (float)(i % 997) / 997.0f;
  float *x, *y, *v;
  CK(cudaMalloc(&x, n * 4));
  CK(cudaMalloc(&y, n * 4));
  CK(cudaMalloc(&v, m * 4));
  CK(cudaMemcpy(x, hx.data(), n * 4, cudaMemcpyHostToDevice));
  CK(cudaMemcpy(y, hy.data(), n * 4, cudaMemcpyHostToDevice));
  CK(cudaMemcpy(v, hv.data(), m * 4, cudaMemcpyHostToDevice));
  cudaStream_t s0, s1;
  CK(cudaStreamCreateWithFlags(&s0, cudaStreamNonBlocking));
  CK(cudaStreamCreateWithFlags(&s1, cudaStreamNonBlocking));
  for (uint32_t r = 0; r < reps; ++r) {   // dependent launches on each stream
    logistic_kernel<<<(m + 255) / 256, 256, 0, s0>>>(LogisticArgs{v, m, iters});
    saxpy_kernel<<<(n + 1023) / 1024, 256, 0, s1>>>(SaxpyArgs{x, y, 0.5f, n});
  }
  CK(cudaGetLastError());
  CK(cudaDeviceSynchronize());
  std::vector<float> gy(n), gv(m);
  CK(cudaMemcpy(gy.data(), y, n * 4, cudaMemcpyDeviceToHost));
  CK(cudaMemcpy(gv.data(), v, m * 4, cudaMemcpyDeviceToHost));
  // host reference, same fp32 RN sequence
  size_t bad = 0;
  double sum = 0.0;
  for (uint32_t i = 0; i < n; ++i) {
    float ry = hy[i];
    for (uint32_t r = 0; r < reps; ++r) {
      volatile float p = 0.5f * hx[i];
      ry = p + ry;
    }
    if (gy[i] != ry) ++bad;
    sum += gy[i];
  }
  for (uint32_t i = 0; i < m; i += 97) {   // sampled: the host replay is slow
    float rv = hv[i];
    for (uint32_t t = 0; t < reps * iters; ++t) {
      volatile float a = 3.7f * rv;
      volatile float b = 1.0f - rv;
      rv = a * b;
    }
    if (gv[i] != rv) ++bad;
    sum += gv[i];
  }
  std::printf("intercept_app: %s bad=%zu checksum=%.6f\n", bad ? "FAIL" : "OK", bad, sum);
  return bad ? 1 : 0;
}
