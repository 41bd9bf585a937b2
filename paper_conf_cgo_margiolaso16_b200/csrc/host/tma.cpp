// tma.cpp -- accel_tma_map_2d: encode a 2-D TMA tensor map (CUtensorMap) for a
// row-major fp32 matrix, for tenant kernels that stage tiles with
// cp.async.bulk.tensor (sgemm).  The driver entry point is resolved through
// the runtime, so libaccel needs no link-time libcuda dependency.
#include <cuda.h>
#include <cuda_runtime.h>

#include <cstdlib>
#include <cstring>

#include "accel.h"

namespace {
using EncodeFn = CUresult (*)(CUtensorMap*, CUtensorMapDataType, cuuint32_t, void*, const cuuint64_t*,
                              const cuuint64_t*, const cuuint32_t*, const cuuint32_t*, CUtensorMapInterleave,
                              CUtensorMapSwizzle, CUtensorMapL2promotion, CUtensorMapFloatOOBfill);
EncodeFn encode_fn() {
  static EncodeFn fn = nullptr;
  if (!fn) {
    void* p = nullptr;
    cudaDriverEntryPointQueryResult q;
    if (cudaGetDriverEntryPoint("cuTensorMapEncodeTiled", &p, cudaEnableDefault, &q) == cudaSuccess &&
        q == cudaDriverEntryPointSuccess)
      fn = reinterpret_cast<EncodeFn>(p);
  }
  return fn;
}
}  // namespace

extern "C" int accel_tma_map_2d(void* out128, const void* gaddr, uint64_t inner, uint64_t outer,
                                uint64_t row_stride_bytes, uint32_t box_inner, uint32_t box_outer,
                                int32_t swizzle) {
  if (!out128 || !gaddr || !inner || !outer || !box_inner || !box_outer) return ACCEL_EINVAL;
  EncodeFn fn = encode_fn();
  if (!fn) return ACCEL_ECUDA;
  CUtensorMap map;
  const cuuint64_t dims[2] = {inner, outer};
  const cuuint64_t strides[1] = {row_stride_bytes};
  const cuuint32_t box[2] = {box_inner, box_outer};
  const cuuint32_t estr[2] = {1, 1};
  const CUtensorMapSwizzle sw = swizzle == 128 ? CU_TENSOR_MAP_SWIZZLE_128B
                                : swizzle == 64 ? CU_TENSOR_MAP_SWIZZLE_64B
                                : swizzle == 32 ? CU_TENSOR_MAP_SWIZZLE_32B
                                                : CU_TENSOR_MAP_SWIZZLE_NONE;
  CUresult r = fn(&map, CU_TENSOR_MAP_DATA_TYPE_FLOAT32, 2, const_cast<void*>(gaddr), dims, strides, box, estr,
                  CU_TENSOR_MAP_INTERLEAVE_NONE, sw, CU_TENSOR_MAP_L2_PROMOTION_L2_256B,
                  CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE);
  if (r != CUDA_SUCCESS) return ACCEL_EINVAL;
  std::memcpy(out128, &map, sizeof(map));
  return ACCEL_OK;
}

extern "C" int accel_tma_map_3d(void* out128, const void* gaddr, uint64_t d0, uint64_t d1, uint64_t d2,
                                uint32_t box0, uint32_t box1, uint32_t box2) {
  if (!out128 || !gaddr || !d0 || !d1 || !d2 || !box0 || !box1 || !box2) return ACCEL_EINVAL;
  if ((d0 * 4) % 16 != 0) return ACCEL_EINVAL;
  EncodeFn fn = encode_fn();
  if (!fn) return ACCEL_ECUDA;
  CUtensorMap map;
  const cuuint64_t dims[3] = {d0, d1, d2};
  const cuuint64_t strides[2] = {d0 * 4, d0 * d1 * 4};
  const cuuint32_t box[3] = {box0, box1, box2};
  const cuuint32_t estr[3] = {1, 1, 1};
  // diagnostic knob (scripts/diag_tma.py): L2 promotion of the boxes
  CUtensorMapL2promotion promo = CU_TENSOR_MAP_L2_PROMOTION_L2_256B;
  if (const char* e = std::getenv("ACCEL_TMA_PROMO"))
    promo = static_cast<CUtensorMapL2promotion>(std::atoi(e) & 3);
  CUresult r = fn(&map, CU_TENSOR_MAP_DATA_TYPE_FLOAT32, 3, const_cast<void*>(gaddr), dims, strides, box, estr,
                  CU_TENSOR_MAP_INTERLEAVE_NONE, CU_TENSOR_MAP_SWIZZLE_NONE, promo, CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE);
  if (r != CUDA_SUCCESS) return ACCEL_EINVAL;
  std::memcpy(out128, &map, sizeof(map));
  return ACCEL_OK;
}
