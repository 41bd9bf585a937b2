// Test pin: NVIDIA's header-only occupancy calculator (cuda_occupancy.h, CUDA 12.9)
// evaluated for a B200 (sm_100) device description.  Used by tests to pin the
// K = 1 quota of the solver oracle against a library routine.
#include <cuda_occupancy.h>
#include <climits>
extern "C" int occ_blocks_per_sm(int block, int regs, int static_smem, int dyn_smem) {
  cudaOccDeviceProp p;
  p.computeMajor = 10; p.computeMinor = 0;
  p.maxThreadsPerBlock = 1024; p.maxThreadsPerMultiprocessor = 2048;
  p.regsPerBlock = 65536; p.regsPerMultiprocessor = 65536; p.warpSize = 32;
  p.sharedMemPerBlock = 49152; p.sharedMemPerMultiprocessor = 233472; p.numSms = 148;
  p.sharedMemPerBlockOptin = 232448; p.reservedSharedMemPerBlock = 1024;
  cudaOccFuncAttributes a;
  a.maxThreadsPerBlock = 1024; a.numRegs = regs; a.sharedSizeBytes = static_smem;
  a.partitionedGCConfig = PARTITIONED_GC_OFF; a.shmemLimitConfig = FUNC_SHMEM_LIMIT_OPTIN;
  a.maxDynamicSharedSizeBytes = 232448 - static_smem; a.numBlockBarriers = 1;
  cudaOccDeviceState s;
  s.carveoutConfig = SHAREDMEM_CARVEOUT_MAX_SHARED;
  cudaOccResult r;
  if (cudaOccMaxActiveBlocksPerMultiprocessor(&r, &p, &a, &s, block, dyn_smem) != CUDA_OCC_SUCCESS)
    return -1;
  return r.activeBlocksPerMultiprocessor;
}
