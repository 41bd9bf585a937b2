// internal.h -- interfaces between the host runtime and the device code of libaccel.
#pragma once
#include <cstdint>

#include <cuda_runtime.h>

#include "accel.h"

namespace accel {

struct Desc;  // csrc/device/dispatch.cuh
struct Ctl;

struct InitStep {
  uint32_t first;      // first descriptor of the step
  uint32_t launches;   // repeat count
  uint32_t total;      // VGs per launch (static)
  uint32_t gx, gy, gz;
  uint32_t chunk;
  uint32_t cov_offset; // coverage offset of the step's first launch
  const uint32_t* order; // dequeue order (nullptr: linear)
  uint64_t qa0;          // initial queue word (alive << 32 | next): main grids with
                         // static first chunks start at grid*chunk (alive = grid
                         // under RESOLVE); 0 otherwise
  uint32_t slices;       // > 1: a single launch split into this many VG ranges
  uint32_t slice_vgs;    //      of slice_vgs VGs each (the last may be shorter)
};

struct InitParams {
  Desc* d;
  Ctl* ctl;               // RESOLVE control block, nullptr under STATIC
  uint32_t live_init;     // initial live quota of the main step
  uint32_t main_step;     // the step the live quota governs
  uint32_t* coverage;     // nullptr unless verify
  accel_vg_record* trace; // nullptr unless ACCEL_REQ_TRACE
  uint32_t flags;
  uint32_t n_steps;
  InitStep steps[ACCEL_MAX_STEPS];
};

// Fill the descriptors of one request on `s` (one tiny kernel).
cudaError_t launch_desc_init(const InitParams& p, uint32_t n_desc, cudaStream_t s);
constexpr size_t kDescBytes = 384;
// cost-model dequeue order (dispatch.cuh accel_lpt_order): one CTA sorts up to
// kMaxOrderVGs 64-bit keys in dynamic shared memory
constexpr uint32_t kMaxOrderVGs = 8192;
constexpr uint32_t kOrderThreads = 512;
constexpr size_t kCtlBytes = 256;

}  // namespace accel
