// intercept.cpp -- libaccel_intercept.so, the transparent-interception shim
// (SURVEY.md §8(f) f4).  PAPER.md §4 (lines 558-563) and §5 (lines 636-646):
// ProxyCL sits between an unmodified application and the OpenCL runtime, its
// App Monitor turns kernel launches into kernel execution requests for the
// Kernel Scheduler.  Here: an LD_PRELOAD library that interposes the CUDA
// runtime's cudaLaunchKernel.
//
//   * A launch of a kernel registered through include/accel_wrap.cuh
//     (accel_intercept_register: original host stub -> its persistent forms)
//     becomes one SHARED-mode accelOS request on a library context: the
//     original grid is the request's Virtual NDRange, args[0] its argument
//     struct (copied at submit).  Every distinct application stream is a
//     tenant; the request is ordered after the work already on that stream
//     (event -> the tenant's stream) and later work on it waits for the
//     request (event after the request's join -> the application stream), so
//     stream semantics are unchanged.  cudaLaunchKernel returns cudaSuccess.
//   * Every other launch (including the library's own persistent grids, which
//     reach this symbol too) goes to the real cudaLaunchKernel (dlsym
//     RTLD_NEXT).  A launch the library cannot take (block or dynamic shared
//     memory other than the registered ones, a submit error) also falls back.
//
// Environment: ACCEL_INTERCEPT_POLICY=static|resolve (default resolve),
// ACCEL_INTERCEPT_VERBOSE=1 prints the redirected / passed-through counts and
// each request's quota at exit.  Requires the application to use the shared
// CUDA runtime (nvcc -cudart shared), the same one libaccel_rt.so links.
#include <cuda_runtime.h>
#include <dlfcn.h>

#include <atomic>
#include <cstdio>
#include <cstdlib>
#include <cstring>
#include <map>
#include <mutex>
#include <string>
#include <vector>

#include "accel.h"

namespace {

using LaunchFn = cudaError_t (*)(const void*, dim3, dim3, void**, size_t, cudaStream_t);

struct Wrapped {
  accel_kernel_desc desc;
  std::string name;
  int32_t kid = -1;   // id in the context (registered on first use)
};

struct Shim {
  std::mutex reg_mu;                        // registry (static-init time)
  std::map<const void*, Wrapped> wrapped;
  std::mutex mu;                            // context, streams, stats
  accel_ctx* ctx = nullptr;
  bool init_failed = false;
  std::map<cudaStream_t, int32_t> tenant_of;
  std::vector<cudaEvent_t> events;          // reusable events
  std::vector<uint64_t> ids;                // submitted requests (verbose stats)
  std::vector<std::pair<std::string, accel_req_stats>> done;
  std::atomic<uint64_t> redirected{0}, passed{0}, fallbacks{0};
  uint64_t since_release = 0;
  bool verbose = std::getenv("ACCEL_INTERCEPT_VERBOSE") != nullptr;
  std::map<uint64_t, std::string> name_of;
};

Shim& shim() {
  static Shim* s = new Shim();   // leaked on purpose: must outlive the app's static destructors
  return *s;
}

LaunchFn real_launch() {
  static LaunchFn fn = reinterpret_cast<LaunchFn>(dlsym(RTLD_NEXT, "cudaLaunchKernel"));
  return fn;
}

cudaEvent_t get_event(Shim& s) {
  if (!s.events.empty()) {
    cudaEvent_t e = s.events.back();
    s.events.pop_back();
    return e;
  }
  cudaEvent_t e = nullptr;
  if (cudaEventCreateWithFlags(&e, cudaEventDisableTiming) != cudaSuccess) return nullptr;
  return e;
}

void collect(Shim& s, bool all) {
  // completed requests: keep their stats (verbose) and free their descriptors
  std::vector<uint64_t> keep;
  for (uint64_t id : s.ids) {
    accel_req_stats st;
    const int rc = accel_stats(s.ctx, id, &st);
    if (rc == ACCEL_OK) {
      if (s.verbose) s.done.emplace_back(s.name_of[id], st);
      s.name_of.erase(id);
    } else if (rc == ACCEL_ENOTREADY && !all) {
      keep.push_back(id);
    }
  }
  s.ids.swap(keep);
  accel_release(s.ctx, ACCEL_ALL);
}

void shim_exit();

// Returns true if the launch was taken as an accelOS request.
bool redirect(Wrapped& w, dim3 grid, dim3 block, void** args, size_t smem, cudaStream_t stream) {
  Shim& s = shim();
  std::lock_guard<std::mutex> g(s.mu);
  if (s.init_failed) return false;
  if (!s.ctx) {
    int dev = 0;
    cudaGetDevice(&dev);
    accel_config cfg{};
    cfg.device = dev;
    cfg.mode = ACCEL_MODE_SHARED;
    const char* p = std::getenv("ACCEL_INTERCEPT_POLICY");
    cfg.policy = (p && std::strcmp(p, "static") == 0) ? ACCEL_POLICY_STATIC : ACCEL_POLICY_RESOLVE;
    if (accel_init(&cfg, &s.ctx) != ACCEL_OK) {
      std::fprintf(stderr, "[accel-intercept] accel_init failed: %s (running natively)\n", accel_last_error(nullptr));
      s.init_failed = true;
      return false;
    }
    std::atexit(shim_exit);
  }
  if (block.x * block.y * block.z != w.desc.block.x * w.desc.block.y * w.desc.block.z || smem != w.desc.dyn_smem)
    return false;
  if (w.kid < 0 && accel_kernel_register(s.ctx, &w.desc, &w.kid) != ACCEL_OK) {
    std::fprintf(stderr, "[accel-intercept] cannot register %s: %s\n", w.name.c_str(), accel_last_error(s.ctx));
    return false;
  }
  auto it = s.tenant_of.find(stream);
  if (it == s.tenant_of.end())
    it = s.tenant_of.emplace(stream, (int32_t)(s.tenant_of.size() % ACCEL_MAX_TENANTS)).first;
  const int32_t tenant = it->second;
  void* main_stream = nullptr;
  if (accel_tenant_stream(s.ctx, tenant, &main_stream, nullptr) != ACCEL_OK) return false;
  cudaStream_t ts = static_cast<cudaStream_t>(main_stream);
  // order after the application's earlier work on its stream
  cudaEvent_t before = get_event(s), after = get_event(s);
  if (!before || !after) return false;
  if (cudaEventRecord(before, stream) != cudaSuccess || cudaStreamWaitEvent(ts, before, 0) != cudaSuccess) return false;
  accel_launch L{};
  L.kernel_id = w.kid;
  L.grid = accel_dim3{grid.x, grid.y, grid.z};
  L.args = args[0];
  L.args_size = w.desc.args_size;
  L.repeat = 1;
  L.order_device = nullptr;
  accel_request r{};
  r.tenant = tenant;
  r.weight = 1;
  r.main_step = 0;
  r.n_steps = 1;
  r.steps = &L;
  uint64_t id = 0;
  if (accel_submit(s.ctx, &r, &id) != ACCEL_OK) {
    std::fprintf(stderr, "[accel-intercept] submit of %s failed: %s (running natively)\n", w.name.c_str(),
                 accel_last_error(s.ctx));
    s.events.push_back(before);
    s.events.push_back(after);
    return false;
  }
  // the application's later work on its stream waits for the request (its
  // last main grid retires after any RESOLVE growth grids: kCfgLast)
  cudaEventRecord(after, ts);
  cudaStreamWaitEvent(stream, after, 0);
  s.events.push_back(before);   // reusable: recorded and waited on
  s.events.push_back(after);
  s.ids.push_back(id);
  s.name_of[id] = w.name;
  if (++s.since_release >= 64) {
    s.since_release = 0;
    collect(s, false);
  }
  return true;
}

// Registered with atexit() when the context is created, i.e. after the CUDA
// runtime initialised -- so it runs before the runtime's own exit handlers.
void shim_exit() {
  Shim& s = shim();
  std::lock_guard<std::mutex> g(s.mu);
  if (s.ctx) {
    accel_sync(s.ctx, ACCEL_ALL);
    collect(s, true);
  }
  if (s.verbose) {
    std::fprintf(stderr, "[accel-intercept] redirected %llu launches, passed through %llu, fell back %llu\n",
                 (unsigned long long)s.redirected.load(), (unsigned long long)s.passed.load(),
                 (unsigned long long)s.fallbacks.load());
    for (auto& d : s.done)
      std::fprintf(stderr, "[accel-intercept] request %s: %u VGs, quota %u (min %u max %u), %.3f ms\n",
                   d.first.c_str(), d.second.vgs_total, d.second.quota_initial, d.second.quota_min,
                   d.second.quota_max, d.second.elapsed_ms);
  }
  if (s.ctx) accel_finalize(s.ctx);
  s.ctx = nullptr;
}

}  // namespace

extern "C" {

__attribute__((visibility("default"))) int accel_intercept_register(const void* original_fn,
                                                                    const accel_kernel_desc* d) {
  if (!original_fn || !d || !d->persistent_fn) return ACCEL_EINVAL;
  Shim& s = shim();
  std::lock_guard<std::mutex> g(s.reg_mu);
  Wrapped w;
  w.desc = *d;
  w.name = d->name ? d->name : "?";
  w.desc.name = nullptr;   // the string lives in w.name
  auto& slot = s.wrapped[original_fn];
  slot = w;
  slot.desc.name = slot.name.c_str();
  return ACCEL_OK;
}

__attribute__((visibility("default"))) cudaError_t cudaLaunchKernel(const void* func, dim3 grid, dim3 block,
                                                                    void** args, size_t smem,
                                                                    cudaStream_t stream) {
  Shim& s = shim();
  Wrapped* w = nullptr;
  {
    std::lock_guard<std::mutex> g(s.reg_mu);
    auto it = s.wrapped.find(func);
    if (it != s.wrapped.end()) w = &it->second;
  }
  if (w) {
    if (redirect(*w, grid, block, args, smem, stream)) {
      s.redirected.fetch_add(1);
      return cudaSuccess;
    }
    s.fallbacks.fetch_add(1);
  } else {
    s.passed.fetch_add(1);
  }
  LaunchFn real = real_launch();
  if (!real) return cudaErrorUnknown;
  return real(func, grid, block, args, smem, stream);
}

}  // extern "C"
