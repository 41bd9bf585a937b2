// Micro-benchmark: throughput of returning atomicAdd on S counters (each on its
// own 128-B line) from G CTAs, thread 0 of each CTA in a loop of `iters`,
// optionally with `work` cycles of spin between atomics.
#include <cstdio>
#include <cuda_runtime.h>
__global__ void k(unsigned* ctr, int shards, int iters, int work, unsigned* sink) {
  __shared__ unsigned s;
  unsigned acc = 0;
  for (int i = 0; i < iters; ++i) {
    if (threadIdx.x == 0) s = atomicAdd(ctr + 32 * ((blockIdx.x + i) % shards), 1u);
    __syncthreads();
    acc += s;
    long long t0 = clock64();
    while (clock64() - t0 < work) {}
    __syncthreads();
  }
  if (acc == 0xdeadbeef) sink[0] = acc;
}
int main() {
  unsigned *ctr, *sink;
  cudaMalloc(&ctr, 32 * 128 * 4);
  cudaMalloc(&sink, 4);
  cudaEvent_t a, b;
  cudaEventCreate(&a);
  cudaEventCreate(&b);
  int grids[] = {148, 592, 888, 1184};
  int shardsv[] = {1, 2, 4, 8, 16, 32};
  int works[] = {0, 2000};
  for (int w : works)
    for (int g : grids)
      for (int s : shardsv) {
        int iters = 50;
        k<<<g, 256>>>(ctr, s, iters, w, sink);
        cudaEventRecord(a);
        k<<<g, 256>>>(ctr, s, iters, w, sink);
        cudaEventRecord(b);
        cudaEventSynchronize(b);
        float ms;
        cudaEventElapsedTime(&ms, a, b);
        double n = (double)g * iters;
        printf("work=%d grid=%d shards=%d: %.1f us, %.1f atomics/us, %.2f us per iteration\n", w, g, s,
               ms * 1e3, n / (ms * 1e3), ms * 1e3 / iters);
      }
  return 0;
}
