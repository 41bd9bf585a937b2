// runtime.cpp -- host runtime of libaccel: context, kernel registry, request
// table, the Kernel Scheduler of PAPER.md §5 (lines 647-655) and stats.
//
// Kernel Scheduler, restated: for every kernel execution request select the
// number of work-groups with the resource-sharing algorithm (§3), construct the
// Virtual NDRange in accelerator memory, change the global size to the new
// number of work-groups keeping the work-group size and dimensions, launch.
// Here: accel_solve() over the active requests, one descriptor per launch
// written by a tiny kernel on the tenant's stream, then cudaLaunchKernel of
// accel_persistent<T> with grid = quota.  NATIVE mode launches accel_native<T>
// on the original grid instead (the standard-sharing baseline, Fig. 1a).
#include <cuda_runtime.h>

#include <algorithm>
#include <cmath>
#include <atomic>
#include <chrono>
#include <cstdio>
#include <cstdlib>
#include <cstring>
#include <map>
#include <memory>
#include <mutex>
#include <string>
#include <thread>
#include <vector>

#include "accel.h"
#include "internal.h"

namespace {

using accel::InitParams;
using accel::kCtlBytes;
using accel::kDescBytes;

constexpr uint32_t kPoolSlots = 16384;      // 4 MiB of descriptors
constexpr uint32_t kFlagStamps = 1u, kFlagAlive = 2u;  // dispatch.cuh

bool is_resolve(int policy) { return policy == ACCEL_POLICY_RESOLVE; }

struct Kernel {
  std::string name;
  const void* pfn;   // accel_persistent<T, STATIC>
  const void* prfn;  // accel_persistent<T, RESOLVE>
  const void* nfn;
  const void* tfn;
  const void* ofn;   // accel_lpt_order<T> (cost-model dequeue order), nullptr = none
  dim3 block;
  uint32_t dyn_smem;
  uint32_t chunk;
  uint32_t args_size;
  int num_regs;
  int static_smem;
  int occ_p, occ_n;
  uint32_t max_per_sm;   // useful occupancy cap (0 = none)
  uint32_t slices;       // R-disp-9: SHARED single launches split into VG ranges (<= 1: none)
  uint32_t threads() const { return block.x * block.y * block.z; }
};

// A cost-model dequeue order computed on the device (accel_lpt_order<T>) for
// one (kernel, grid, args).  Computed synchronously on the context's order
// stream the first time a submit needs it -- before anything of the group is
// enqueued, so a group's first launches still reach the device together (an
// order kernel on the tenant stream delayed that request's grid and the block
// scheduler then placed it into whatever room the others left, measured:
// cutcp 7 CTAs on one SM where the solver's model F had 3).
struct OrderEntry {
  uint32_t* dev = nullptr;
};

struct Step {
  int kid;
  accel_dim3 grid;
  uint32_t total;
  std::vector<unsigned char> args;
  uint32_t repeat;
  uint32_t quota;
  uint32_t first;       // first descriptor (relative to the request's slot)
  uint64_t cov_offset;  // coverage offset of the first launch
  const uint32_t* order = nullptr;  // dequeue order (device), nullptr = linear
  uint32_t slices = 1;     // R-disp-9: > 1 = one launch run as `repeat` VG ranges
  uint32_t slice_vgs = 0;  //            of slice_vgs VGs
  bool sticky_main = false;  // ACCEL_STICKY_MAIN experiment: one grid serves every launch
};

struct Request {
  uint64_t id;
  int tenant;
  uint32_t flags;
  uint32_t weight;
  int mode;
  std::vector<Step> steps;
  int main_step;
  std::vector<accel_clear> clears;
  std::vector<accel_copy> h2d, d2h;
  cudaEvent_t ev_arrival = nullptr, ev_done = nullptr;
  // recorded on the tenant stream right after the descriptor init: everything
  // that touches the request's descriptors or control block from another
  // stream (growth grids, live-quota writes, the early main grid) waits on it
  cudaEvent_t ev_init = nullptr;
  std::vector<cudaEvent_t> ev_launch;  // ACCEL_REQ_LAUNCH_EVENTS: n_desc + 1
  // RESOLVE: one event after every top-up grid.  The request's descriptors
  // may only be released (and reused) once its sticky top-up CTAs retired.
  std::vector<cudaEvent_t> ev_topups;
  // ACCEL_DEBUG: (tag, quota, event) of each re-solve -- 'L' after the live-quota
  // write on the ctl stream, 'T' on the top-up stream just before a growth grid
  struct DbgEv { char tag; uint32_t q; cudaEvent_t ev; };
  std::vector<DbgEv> dbg;
  uint32_t slot = 0, n_desc = 0;
  uint32_t* cov = nullptr;
  uint64_t cov_elems = 0;
  accel_vg_record* trace = nullptr;   // ACCEL_REQ_TRACE, cov layout
  uint64_t trace_elems = 0;
  uint32_t quota_initial = 0, quota_min = 0, quota_max = 0, resolves = 0;
  size_t enq_step = 0;       // enqueue cursor (enqueue_next)
  uint32_t enq_launch = 0, enq_li = 0;
  bool early_main = false;   // R-place-3: main step launched ahead on a side stream
  bool grown = false;        // RESOLVE: a top-up grid was launched (device Ctl::grown)
  uint32_t early_sms = 0;    // SMs its waiting grid may hold (released when done)
  cudaEvent_t ev_early = nullptr;  // recorded after that launch (the main stream waits for it)
  uint32_t live = 0;         // RESOLVE: current live quota of the main step
  uint32_t provisioned = 0;  // RESOLVE: main-grid CTAs + sticky top-up CTAs
  std::chrono::steady_clock::time_point t_submit;
  bool done = false;
  bool departed_seen = false;  // monitor already re-solved for this departure
  bool fetched = false;
  int cov_ok = -1;
  std::vector<unsigned char> desc_host;
};

bool is_sticky(cudaError_t e) {
  switch (e) {
    case cudaErrorIllegalAddress:
    case cudaErrorLaunchFailure:
    case cudaErrorIllegalInstruction:
    case cudaErrorMisalignedAddress:
    case cudaErrorInvalidAddressSpace:
    case cudaErrorInvalidPc:
    case cudaErrorHardwareStackError:
    case cudaErrorAssert:
    case cudaErrorLaunchTimeout:
    case cudaErrorECCUncorrectable:
      return true;
    default:
      return false;
  }
}

std::string g_init_error;

// Host view of the device descriptor (csrc/device/dispatch.cuh accel::Desc).
struct DescHost {
  // line 0
  uint32_t total, gx, gy, gz, chunk, launch_idx, flags, req_idx;
  uint64_t ctl, coverage;
  uint32_t has_prev, vg_base;
  uint64_t trace;
  uint32_t governed, slice;
  uint64_t order;
  uint32_t pad0[12];
  // line 1
  unsigned long long qa;  // alive << 32 | next
  uint32_t pad1[30];
  // line 2
  unsigned long long t_first, t_last;
  uint32_t total_seen, ctas_started, tu_alive, max_alive, topped, admit_fail, evicted, last_live, pad_adm, draining, pad2[18];
};
static_assert(sizeof(DescHost) == accel::kDescBytes, "host view of the descriptor");

}  // namespace

struct accel_ctx {
  accel_config cfg{};
  accel_caps caps{};
  std::mutex mu;
  std::string err;
  bool poisoned = false;
  std::vector<Kernel> kernels;
  cudaStream_t main[ACCEL_MAX_TENANTS] = {};
  // RESOLVE top-up grids are sticky (they follow a request's launches), so two
  // of them must never share a stream: a pool with its own hardware queues
  // (16 main + 12 top-up + 1 control <= CUDA_DEVICE_MAX_CONNECTIONS = 32).
  uint32_t early_sms = 0;   // R-place-3: SMs held by early grids still waiting on the device
  static constexpr int kTopupStreams = 12;
  cudaStream_t topup[kTopupStreams] = {};
  // a growth grid is sticky (it follows its step's later launches), so a grid
  // queued behind another request's on the same stream would not start until
  // that one's step ends: take an idle top-up stream when there is one
  // Coverage / trace buffers recycled by size: a cudaMalloc per submit stalls
  // the submitting thread (and so the arrival of the next request) for 0.1-1 ms
  std::multimap<size_t, void*> buf_pool;
  cudaError_t buf_get(void** p, size_t bytes) {
    auto it = buf_pool.find(bytes);
    if (it != buf_pool.end()) {
      *p = it->second;
      buf_pool.erase(it);
      return cudaSuccess;
    }
    return cudaMalloc(p, bytes);
  }
  void buf_put(void* p, size_t bytes) {
    if (buf_pool.size() >= 64) {
      cudaFree(p);
      return;
    }
    buf_pool.emplace(bytes, p);
  }
  cudaStream_t pick_topup_stream() {
    for (int i = 0; i < kTopupStreams; ++i) {
      const uint32_t k = (topup_rr + (uint32_t)i) % kTopupStreams;
      if (cudaStreamQuery(topup[k]) == cudaSuccess) {
        topup_rr = k + 1;
        return topup[k];
      }
    }
    return topup[topup_rr++ % kTopupStreams];
  }
  uint32_t topup_rr = 0;
  cudaStream_t ctl = nullptr;
  cudaStream_t ostream = nullptr;   // cost-model orders (synchronous, first use)
  cudaEvent_t epoch = nullptr;
  bool epoch_set = false;
  unsigned char* pool = nullptr;
  unsigned char* ctl_pool = nullptr;      // accel::Ctl per descriptor slot
  uint32_t* pinned_ring = nullptr;        // staging for live-quota writes
  uint32_t ring_pos = 0;
  std::thread monitor;
  std::atomic<bool> stop{false};
  uint64_t monitor_solves = 0;
  uint32_t ablate = 0;
  std::chrono::steady_clock::time_point t_init = std::chrono::steady_clock::now();   // ACCEL_DEBUG stamps   // env ACCEL_ABLATE: measurement-only cfg bits (dispatch.cuh kAbl*)
  bool pdl = true;       // programmatic dependent launch between a request's launches (env ACCEL_PDL=0: off)
  std::vector<uint8_t> slot_used;
  std::map<uint64_t, std::unique_ptr<Request>> reqs;
  std::map<std::string, OrderEntry> orders;   // cost-model orders by (kernel, grid, args)
  uint64_t next_id = 1;
  std::vector<cudaEvent_t> free_events;

  int fail(int code, const std::string& msg) {
    err = msg;
    return code;
  }
  int cuda(cudaError_t e, const char* what) {
    if (e == cudaSuccess) return ACCEL_OK;
    err = std::string(what) + ": " + cudaGetErrorString(e);
    if (is_sticky(e)) poisoned = true;
    cudaGetLastError();
    return ACCEL_ECUDA;
  }
  cudaError_t get_event(cudaEvent_t* ev) {
    if (!free_events.empty()) {
      *ev = free_events.back();
      free_events.pop_back();
      return cudaSuccess;
    }
    return cudaEventCreate(ev);
  }
  int64_t alloc_slots(uint32_t n) {
    uint32_t run = 0;
    for (uint32_t i = 0; i < kPoolSlots; ++i) {
      run = slot_used[i] ? 0 : run + 1;
      if (run == n) {
        const uint32_t s = i + 1 - n;
        std::fill(slot_used.begin() + s, slot_used.begin() + s + n, 1);
        return s;
      }
    }
    return -1;
  }
  void free_slots(uint32_t s, uint32_t n) { std::fill(slot_used.begin() + s, slot_used.begin() + s + n, 0); }
  accel::Desc* desc_ptr(uint32_t slot) { return reinterpret_cast<accel::Desc*>(pool + (size_t)slot * kDescBytes); }
  accel::Ctl* ctl_ptr(uint32_t slot) { return reinterpret_cast<accel::Ctl*>(ctl_pool + (size_t)slot * kCtlBytes); }
};

#define CK(ctx, call)                                  \
  do {                                                 \
    int _rc = (ctx)->cuda((call), #call);              \
    if (_rc != ACCEL_OK) return _rc;                   \
  } while (0)

namespace {

bool debug_on();
double host_us(const accel_ctx* ctx);

int refresh_done(accel_ctx* ctx, Request* r) {
  if (r->done) return ACCEL_OK;
  cudaError_t e = cudaEventQuery(r->ev_done);
  for (size_t i = 0; e == cudaSuccess && i < r->ev_topups.size(); ++i) e = cudaEventQuery(r->ev_topups[i]);
  if (e == cudaSuccess) {
    r->done = true;
    ctx->early_sms -= r->early_sms;
    r->early_sms = 0;
  } else if (e != cudaErrorNotReady) {
    return ctx->cuda(e, "cudaEventQuery");
  }
  return ACCEL_OK;
}


// The solver's upper bound on a kernel's CTAs is its grid (PAPER.md lines
// 538-541: work-groups are added "until resource saturation"), lowered -- when
// the request shares the device (in_mix) -- to the kernel's declared useful
// occupancy x SMs (R-solver-10).  Alone, a request keeps its full share.
int demand_for(accel_ctx* ctx, const Step& s, uint32_t weight, accel_demand* d, bool in_mix = false) {
  const Kernel& k = ctx->kernels[s.kid];
  uint32_t cap = s.total;
  if (in_mix && k.max_per_sm) cap = std::min<uint64_t>(cap, (uint64_t)k.max_per_sm * (uint32_t)ctx->caps.sms);
  return accel_demand_of(&ctx->caps, k.threads(), (uint32_t)k.num_regs,
                         (uint32_t)(k.static_smem + k.dyn_smem), cap, weight, d);
}

int fetch_result(accel_ctx* ctx, Request* r) {
  if (r->fetched) return ACCEL_OK;
  r->desc_host.resize((size_t)r->n_desc * kDescBytes);
  CK(ctx, cudaMemcpy(r->desc_host.data(), ctx->desc_ptr(r->slot), r->desc_host.size(),
                     cudaMemcpyDeviceToHost));
  if (r->cov) {
    std::vector<uint32_t> cov(r->cov_elems);
    CK(ctx, cudaMemcpy(cov.data(), r->cov, cov.size() * sizeof(uint32_t), cudaMemcpyDeviceToHost));
    bool ok = true;
    for (const Step& s : r->steps)
      for (uint32_t l = 0; l < (s.slices > 1 ? 1u : s.repeat); ++l) {   // a sliced step: one grid
        const DescHost* d = reinterpret_cast<const DescHost*>(r->desc_host.data() + (size_t)(s.first + l) * kDescBytes);
        // dynamic-total kernels (bfs) cover only the live part of the static grid
        const uint32_t live = s.slices > 1 ? s.total : (d->total_seen <= s.total ? d->total_seen : s.total);
        const uint32_t* c = cov.data() + s.cov_offset + (uint64_t)l * s.total;
        uint32_t bad = 0, first_bad = 0, got = 0;
        for (uint32_t v = 0; v < s.total; ++v) {
          const uint32_t want = v < live ? 1u : 0u;
          if (c[v] != want) {
            if (bad++ == 0) {
              first_bad = v;
              got = c[v];
            }
          }
        }
        if (bad) {
          ok = false;
          if (debug_on())
            std::fprintf(stderr,
                         "[accel] coverage: req %llu tenant %d launch %u: %u bad VGs (first %u ran %u times), "
                         "total %u seen %u next %u topped %u alive %u refused %u evicted %u live %u\n",
                         (unsigned long long)r->id, r->tenant, s.first + l, bad, first_bad, got, s.total,
                         d->total_seen, (uint32_t)d->qa, d->topped, (uint32_t)(d->qa >> 32), d->admit_fail, d->evicted, d->last_live);
        }
      }
    r->cov_ok = ok ? 1 : 0;
  }
  if (debug_on()) {
    uint64_t ev = 0, af = 0, mx = 0, tu = 0;
    for (uint32_t l = 0; l < r->n_desc; ++l) {
      const DescHost* d = reinterpret_cast<const DescHost*>(r->desc_host.data() + (size_t)l * kDescBytes);
      ev += d->evicted;
      af += d->admit_fail;
      mx = std::max<uint64_t>(mx, d->max_alive);
      tu += d->topped;
    }
    std::fprintf(stderr, "[accel] req %llu tenant %d: %u launches, evicted %llu, refused %llu, max_alive %llu, topped %llu\n",
                 (unsigned long long)r->id, r->tenant, r->n_desc, (unsigned long long)ev, (unsigned long long)af,
                 (unsigned long long)mx, (unsigned long long)tu);
  }
  for (const Request::DbgEv& x : r->dbg) {
    float ms = -1.f;
    cudaEventElapsedTime(&ms, r->ev_arrival, x.ev);
    std::fprintf(stderr, "[accel] req %llu tenant %d re-solve %c q=%u at +%.1f us after arrival\n",
                 (unsigned long long)r->id, r->tenant, x.tag, x.q, 1e3f * ms);
    cudaEventDestroy(x.ev);
  }
  r->dbg.clear();
  r->fetched = true;
  return ACCEL_OK;
}

// Enqueue of one request, in three parts so that a group's requests can be
// interleaved (enqueue_group): begin = arrival event, clears, copies,
// descriptor init; then its launch units (one per launch) in order; end =
// join, copies back, done event.
int enqueue_begin(accel_ctx* ctx, Request* r) {
  const bool shared = r->mode == ACCEL_MODE_SHARED;
  cudaStream_t s = ctx->main[r->tenant];
  CK(ctx, ctx->get_event(&r->ev_arrival));
  CK(ctx, ctx->get_event(&r->ev_done));
  CK(ctx, cudaEventRecord(r->ev_arrival, s));
  for (const accel_clear& c : r->clears) CK(ctx, cudaMemsetAsync(c.dst_device, c.value, c.bytes, s));
  for (const accel_copy& c : r->h2d) CK(ctx, cudaMemcpyAsync(c.dst, c.src, c.bytes, cudaMemcpyHostToDevice, s));
  if (r->cov) CK(ctx, cudaMemsetAsync(r->cov, 0, r->cov_elems * sizeof(uint32_t), s));
  if (r->trace) CK(ctx, cudaMemsetAsync(r->trace, 0, r->trace_elems * sizeof(accel_vg_record), s));
  InitParams p{};
  p.d = ctx->desc_ptr(r->slot);
  const bool resolve = shared && is_resolve(ctx->cfg.policy);
  p.ctl = resolve ? ctx->ctl_ptr(r->slot) : nullptr;
  p.live_init = r->steps[r->main_step].quota;
  p.main_step = (uint32_t)r->main_step;
  p.coverage = r->cov;
  p.trace = r->trace;
  p.flags = kFlagStamps | (shared ? kFlagAlive : 0u);
  p.n_steps = (uint32_t)r->steps.size();
  static const bool sticky_env = std::getenv("ACCEL_STICKY_MAIN") != nullptr;
  for (size_t j = 0; j < r->steps.size(); ++j) {
    Step& st = r->steps[j];
    st.sticky_main = sticky_env && resolve && (int)j == r->main_step && st.repeat > 1 && st.slices <= 1;
  }
  for (size_t j = 0; j < r->steps.size(); ++j) {
    const Step& st = r->steps[j];
    const Kernel& k = ctx->kernels[st.kid];
    // main grids (SHARED) take static first chunks: the queue head starts
    // past them and, under RESOLVE, every main-grid CTA is admitted
    // (a sliced step counts its CTAs under both policies: its last slice
    // waits for the others, R-disp-9)
    const uint64_t qa0 = st.sticky_main ? 0ull   // every CTA joins through the queue word
        : shared ? ((resolve || st.slices > 1 ? (uint64_t)st.quota << 32 : 0ull) | ((uint64_t)st.quota * k.chunk))
        : 0ull;
    p.steps[j] = accel::InitStep{st.first, st.repeat, st.total, st.grid.x, st.grid.y, st.grid.z,
                                 k.chunk, (uint32_t)st.cov_offset, shared ? st.order : nullptr, qa0,
                                 st.slices, st.slice_vgs};
  }
  CK(ctx, accel::launch_desc_init(p, r->n_desc, s));
  if (resolve) {
    CK(ctx, ctx->get_event(&r->ev_init));
    CK(ctx, cudaEventRecord(r->ev_init, s));
  }
  if (r->flags & ACCEL_REQ_LAUNCH_EVENTS) {
    r->ev_launch.resize(r->n_desc + 1);
    for (auto& ev : r->ev_launch) CK(ctx, ctx->get_event(&ev));
  }
  r->enq_step = 0;
  r->enq_launch = 0;
  r->enq_li = 0;
  // R-place-3: a request whose main step is its last, single launch of CTAs
  // that take at least half an SM (the tensor-core GEMM after its operand
  // split) launches that grid NOW, on a side stream, so the block scheduler
  // places it before the co-runners' small CTAs fragment every SM; its CTAs
  // wait on the device for the earlier steps (kCfgWaitPrev).  RESOLVE only
  // (the wait needs the alive accounting) and only with a quota below the
  // SM count (a quota holding every SM would leave the earlier steps nowhere
  // to run).
  r->early_main = false;
  const size_t ms = (size_t)r->main_step;
  if (shared && resolve && ms > 0 && ms + 1 == r->steps.size() && r->steps[ms].repeat == 1 &&
      // the early grids' CTAs wait on the device while holding (up to) an SM
      // each: together they may hold at most half the device, so the earlier
      // steps and every co-runner always have SMs to make progress on (two
      // early GEMMs of 74 CTAs each would otherwise hold all 148 SMs and wait
      // for split steps that can run nowhere)
      ctx->early_sms + r->steps[ms].quota <= (uint32_t)ctx->caps.sms / 2) {
    const Step& st = r->steps[ms];
    const Kernel& k = ctx->kernels[st.kid];
    accel_demand dm{};
    if (demand_for(ctx, st, 1, &dm) == ACCEL_OK &&
        (2 * (int64_t)dm.thr >= ctx->caps.thr_per_sm || 2 * (int64_t)dm.regs >= ctx->caps.regs_per_sm ||
         2 * (int64_t)dm.smem >= ctx->caps.smem_per_sm)) {
      r->early_main = true;
      r->early_sms = st.quota;
      ctx->early_sms += st.quota;
      cudaStream_t es = ctx->pick_topup_stream();
      CK(ctx, cudaStreamWaitEvent(es, r->ev_init, 0));  // descriptors initialised
      accel::Desc* d = ctx->desc_ptr(r->slot + st.first);
      // kCfgResolve | kCfgStamps | kCfgHasPrev | kCfgStaticFirst | kCfgWaitPrev
      uint32_t cfg = (k.chunk & 0xffffu) | (1u << 16) | (1u << 17) | (1u << 18) | (1u << 19) | (1u << 20) | ctx->ablate;
      void* params[3] = {const_cast<unsigned char*>(st.args.data()), &d, &cfg};
      CK(ctx, cudaLaunchKernel(k.prfn, dim3(st.quota, 1, 1), k.block, params, k.dyn_smem, es));
      CK(ctx, ctx->get_event(&r->ev_early));
      CK(ctx, cudaEventRecord(r->ev_early, es));
    }
  }
  return ACCEL_OK;
}

// Enqueue the request's next launch unit; *more = false once all are enqueued.
int enqueue_next(accel_ctx* ctx, Request* r, bool* more) {
  const bool shared = r->mode == ACCEL_MODE_SHARED;
  const bool resolve = shared && is_resolve(ctx->cfg.policy);
  const bool lev = (r->flags & ACCEL_REQ_LAUNCH_EVENTS) != 0;
  cudaStream_t s = ctx->main[r->tenant];
  const size_t n_units = r->early_main ? (size_t)r->main_step : r->steps.size();
  if (r->enq_step >= n_units) {
    *more = false;
    return ACCEL_OK;
  }
  const Step& st = r->steps[r->enq_step];
  const Kernel& k = ctx->kernels[st.kid];
  const uint32_t li = r->enq_li;
  if (st.sticky_main) {
    // ACCEL_STICKY_MAIN: one grid of `quota` CTAs serves the step's launches
    // in order (accel_topup with the main-grid flag)
    for (uint32_t l = 0; lev && l < st.repeat; ++l) CK(ctx, cudaEventRecord(r->ev_launch[li + l], s));
    accel::Desc* d = ctx->desc_ptr(r->slot + st.first);
    uint32_t sticky = st.repeat | (1u << 31);
    void* params[3] = {const_cast<unsigned char*>(st.args.data()), &d, &sticky};
    CK(ctx, cudaLaunchKernel(k.tfn, dim3(st.quota, 1, 1), k.block, params, k.dyn_smem, s));
    r->enq_li += st.repeat;
    r->enq_launch = 0;
    r->enq_step += 1;
    *more = r->enq_step < (r->early_main ? (size_t)r->main_step : r->steps.size());
    return ACCEL_OK;
  }
  if (lev) CK(ctx, cudaEventRecord(r->ev_launch[li], s));
  {
    const uint32_t l = r->enq_launch;
    accel::Desc* d = ctx->desc_ptr(r->slot + st.first + l);
    // accel_persistent cfg word (dispatch.cuh): chunk | kCfgResolve | kCfgStamps
    // | kCfgHasPrev (a request-relative launch precedes this one) | kCfgStaticFirst
    // | kCfgAccount (RESOLVE, a request with an early main grid: its CTAs keep
    // the fenced alive decrement the early grid's wait_complete counts on)
    // | kCfgLast (RESOLVE: the request's join).  A sliced step (R-disp-9):
    // every slice accounts (kCfgAccount), the later ones depend on nothing
    // before them (kCfgIndep: no predecessor wait, no griddepcontrol.wait),
    // the last one joins the others (kCfgSliceJoin)
    const bool sliced = st.slices > 1, indep = sliced && l > 0;
    uint32_t cfg = (k.chunk & 0xffffu) | (resolve ? (1u << 16) : 0u) | (1u << 17) |
                   (li > 0 && !indep ? (1u << 18) : 0u) | (1u << 19) |
                   ((resolve && r->early_main) || sliced ? (1u << 21) : 0u) |
                   (resolve && li + 1 == r->n_desc ? (1u << 23) : 0u) | (indep ? (1u << 29) : 0u) |
                   (sliced && l + 1 == st.repeat ? (1u << 30) : 0u) | ctx->ablate;
    void* params[3] = {const_cast<unsigned char*>(st.args.data()), &d, &cfg};
    const dim3 grid = shared ? dim3(st.quota, 1, 1) : dim3(st.grid.x, st.grid.y, st.grid.z);
    const void* fn = shared ? (resolve ? k.prfn : k.pfn) : k.nfn;
    if (li > 0 && ctx->pdl) {
      // Programmatic dependent launch (both modes): launch l directly follows
      // launch l-1 of the same request on this stream; its CTAs may become
      // resident as l-1's CTAs retire and wait on the device
      // (griddepcontrol.wait) instead of after a host-visible kernel boundary
      cudaLaunchConfig_t lc = {};
      lc.gridDim = grid;
      lc.blockDim = k.block;
      lc.dynamicSmemBytes = k.dyn_smem;
      lc.stream = s;
      cudaLaunchAttribute at[1];
      at[0].id = cudaLaunchAttributeProgrammaticStreamSerialization;
      at[0].val.programmaticStreamSerializationAllowed = 1;
      lc.attrs = at;
      lc.numAttrs = 1;
      CK(ctx, cudaLaunchKernelExC(&lc, fn, params));
    } else {
      CK(ctx, cudaLaunchKernel(fn, grid, k.block, params, k.dyn_smem, s));
    }
    r->enq_li += 1;
    if (++r->enq_launch >= st.repeat) {
      r->enq_launch = 0;
      r->enq_step += 1;
    }
  }
  *more = r->enq_step < n_units;
  return ACCEL_OK;
}

int enqueue_end(accel_ctx* ctx, Request* r) {
  const bool shared = r->mode == ACCEL_MODE_SHARED;
  const bool resolve = shared && is_resolve(ctx->cfg.policy);
  cudaStream_t s = ctx->main[r->tenant];
  if (r->early_main) {
    // launch-time stamps: the early grid's work starts once the earlier
    // steps are complete, i.e. here on the main stream
    if (r->flags & ACCEL_REQ_LAUNCH_EVENTS) CK(ctx, cudaEventRecord(r->ev_launch[r->enq_li], s));
    CK(ctx, cudaStreamWaitEvent(s, r->ev_early, 0));
    r->enq_li = r->n_desc;   // the early launch was the last one
  }
  if (r->flags & ACCEL_REQ_LAUNCH_EVENTS) CK(ctx, cudaEventRecord(r->ev_launch[r->enq_li], s));
  for (const accel_copy& c : r->d2h) CK(ctx, cudaMemcpyAsync(c.dst, c.src, c.bytes, cudaMemcpyDeviceToHost, s));
  CK(ctx, cudaEventRecord(r->ev_done, s));
  return ACCEL_OK;
}

// Enqueue requests that arrive together (order = the order their first
// launches reach the device): every request's arrival, set-up and FIRST launch
// first, then the remaining launches round-robin.  Enqueueing request by
// request held a 100-launch request's co-runners back by its whole host
// enqueue time (~0.4 ms of C2, measured with scripts/timeline.py).
int enqueue_group(accel_ctx* ctx, const std::vector<Request*>& rs) {
  std::vector<bool> more(rs.size(), true);
  for (size_t i = 0; i < rs.size(); ++i) {
    int rc = enqueue_begin(ctx, rs[i]);
    if (rc) return rc;
    bool m = false;
    rc = enqueue_next(ctx, rs[i], &m);
    if (rc) return rc;
    more[i] = m;
  }
  for (bool any = true; any;) {
    any = false;
    for (size_t i = 0; i < rs.size(); ++i) {
      if (!more[i]) continue;
      bool m = false;
      int rc = enqueue_next(ctx, rs[i], &m);
      if (rc) return rc;
      more[i] = m;
      any = any || m;
    }
  }
  for (Request* r : rs) {
    int rc = enqueue_end(ctx, r);
    if (rc) return rc;
  }
  return ACCEL_OK;
}

int build_request(accel_ctx* ctx, const accel_request& in, std::unique_ptr<Request>* out) {
  if (in.tenant < 0 || in.tenant >= ACCEL_MAX_TENANTS) return ctx->fail(ACCEL_EINVAL, "tenant out of range");
  if (in.n_steps < 1 || in.n_steps > ACCEL_MAX_STEPS || !in.steps) return ctx->fail(ACCEL_EINVAL, "bad n_steps");
  if ((in.n_clear && !in.clear) || (in.n_h2d && !in.h2d) || (in.n_d2h && !in.d2h))
    return ctx->fail(ACCEL_EINVAL, "null clear/copy array");
  auto r = std::make_unique<Request>();
  r->tenant = in.tenant;
  r->flags = in.flags;
  r->weight = in.weight ? in.weight : 1;
  r->mode = ctx->cfg.mode;
  r->t_submit = std::chrono::steady_clock::now();
  uint32_t n_desc = 0;
  uint64_t cov = 0;
  if (in.main_step >= (int32_t)in.n_steps) return ctx->fail(ACCEL_EINVAL, "main_step out of range");
  r->main_step = in.main_step >= 0 ? in.main_step : 0;
  for (uint32_t j = 0; j < in.n_steps; ++j) {
    const accel_launch& L = in.steps[j];
    if (L.kernel_id < 0 || L.kernel_id >= (int)ctx->kernels.size()) return ctx->fail(ACCEL_EINVAL, "bad kernel_id");
    const Kernel& k = ctx->kernels[L.kernel_id];
    if (L.args_size != k.args_size || !L.args) return ctx->fail(ACCEL_EINVAL, "args_size mismatch for " + k.name);
    if (L.repeat < 1) return ctx->fail(ACCEL_EINVAL, "repeat < 1");
    const uint64_t total = (uint64_t)L.grid.x * L.grid.y * L.grid.z;
    if (total == 0 || total >= 0x7fffffffull || L.grid.y > 65535 || L.grid.z > 65535)
      return ctx->fail(ACCEL_EINVAL, "bad grid");
    Step s;
    s.kid = L.kernel_id;
    s.grid = L.grid;
    s.total = (uint32_t)total;
    s.args.assign((const unsigned char*)L.args, (const unsigned char*)L.args + L.args_size);
    s.repeat = L.repeat;
    s.order = L.order_device;
    if (!s.order && k.ofn && r->mode == ACCEL_MODE_SHARED && !(in.flags & ACCEL_REQ_LINEAR_ORDER) &&
        total <= accel::kMaxOrderVGs) {
      std::string key(reinterpret_cast<const char*>(&L.kernel_id), sizeof(L.kernel_id));
      key.append(reinterpret_cast<const char*>(&L.grid), sizeof(L.grid));
      key.append(s.args.begin(), s.args.end());
      OrderEntry& oe = ctx->orders[key];
      if (oe.dev == nullptr) {   // first use: sort the VGs by the kernel's cost model now
        CK(ctx, cudaMalloc(&oe.dev, total * sizeof(uint32_t)));
        uint32_t gx = L.grid.x, gy = L.grid.y, gz = L.grid.z;
        uint32_t* dst = oe.dev;
        void* params[5] = {const_cast<void*>(L.args), &gx, &gy, &gz, &dst};
        CK(ctx, cudaLaunchKernel(k.ofn, dim3(1), dim3(accel::kOrderThreads), params,
                                 accel::kMaxOrderVGs * sizeof(unsigned long long), ctx->ostream));
        CK(ctx, cudaStreamSynchronize(ctx->ostream));
      }
      s.order = oe.dev;
    }
    s.quota = s.total;
    s.first = n_desc;
    s.cov_offset = cov;
    if (r->mode == ACCEL_MODE_SHARED && k.slices > 1 && L.repeat == 1 && total >= 2ull * k.slices) {
      // R-disp-9: the launch as `slices` consecutive VG ranges (one coverage region)
      s.slices = k.slices;
      s.slice_vgs = (uint32_t)((total + k.slices - 1) / k.slices);
      s.repeat = (uint32_t)((total + s.slice_vgs - 1) / s.slice_vgs);
      n_desc += s.repeat;
      cov += s.total;
    } else {
      n_desc += L.repeat;
      cov += (uint64_t)L.repeat * s.total;
    }
    r->steps.push_back(std::move(s));
    if (in.main_step < 0 && r->steps.back().total > r->steps[r->main_step].total) r->main_step = (int)j;
  }
  r->n_desc = n_desc;
  r->cov_elems = ctx->cfg.verify ? cov : 0;
  r->trace_elems = (in.flags & ACCEL_REQ_TRACE) ? cov : 0;
  r->clears.assign(in.clear, in.clear + in.n_clear);
  r->h2d.assign(in.h2d, in.h2d + in.n_h2d);
  r->d2h.assign(in.d2h, in.d2h + in.n_d2h);
  *out = std::move(r);
  return ACCEL_OK;
}

constexpr uint32_t kRing = 4096;

// RESOLVE: set a running request's live quota (copy engine, no SM needed) and
// add sticky top-up CTAs when it grows beyond what is provisioned.
bool debug_on() {
  static const bool on = std::getenv("ACCEL_DEBUG") != nullptr;
  return on;
}

int apply_quota(accel_ctx* ctx, Request* r, uint32_t q) {
  if (debug_on())
    std::fprintf(stderr, "[accel] resolve req %llu tenant %d live %u -> %u (provisioned %u)\n",
                 (unsigned long long)r->id, r->tenant, r->live, q, r->provisioned);
  if (q == r->live || r->ev_init == nullptr) return ACCEL_OK;
  if (cudaEventQuery(r->ev_done) == cudaSuccess) return ACCEL_OK;  // finished: nothing to grow
  // {live, grown} (Ctl line 0), one 8-byte copy; grown is set before the
  // request's first top-up grid (that grid waits for this copy), so main CTAs
  // that see it account at retire (dispatch.cuh "completion accounting")
  const bool grow = q > r->provisioned && !r->early_main;
  uint32_t* h = ctx->pinned_ring + 2 * (ctx->ring_pos++ % (kRing / 2));
  h[0] = q;
  h[1] = (r->grown || grow) ? 1u : 0u;
  // both the live-quota write and a growth grid must follow the request's
  // descriptor init (which writes live_init and resets the queue words): a
  // re-solve may come while the tenant stream is still copying its inputs
  const double t_a = debug_on() ? host_us(ctx) : 0.0;
  CK(ctx, cudaStreamWaitEvent(ctx->ctl, r->ev_init, 0));
  const double t_b = debug_on() ? host_us(ctx) : 0.0;
  CK(ctx, cudaMemcpyAsync(ctx->ctl_pool + (size_t)r->slot * kCtlBytes /* Ctl::live, Ctl::grown */, h,
                          2 * sizeof(uint32_t), cudaMemcpyHostToDevice, ctx->ctl));
  cudaEvent_t ev_ctl = nullptr;
  if (grow) {
    CK(ctx, ctx->get_event(&ev_ctl));
    CK(ctx, cudaEventRecord(ev_ctl, ctx->ctl));
    r->ev_topups.push_back(ev_ctl);   // (recycled with the request's events)
  }
  if (debug_on()) {
    cudaEvent_t ev;
    CK(ctx, cudaEventCreate(&ev));
    CK(ctx, cudaEventRecord(ev, ctx->ctl));
    r->dbg.push_back({'L', q, ev});
  }
  const double t_c = debug_on() ? host_us(ctx) : 0.0;
  double t_d = t_c, t_e = t_c;
  // (no growth grids for an early main step: they would wait beside it for
  // the earlier steps and could hold the SMs those need)
  if (grow) {
    r->grown = true;
    const Step& st = r->steps[r->main_step];
    const Kernel& k = ctx->kernels[st.kid];
    accel::Desc* d = ctx->desc_ptr(r->slot + st.first);
    uint32_t sticky = st.repeat;
    void* params[3] = {const_cast<unsigned char*>(st.args.data()), &d, &sticky};
    cudaStream_t ts = ctx->pick_topup_stream();
    CK(ctx, cudaStreamWaitEvent(ts, r->ev_init, 0));
    CK(ctx, cudaStreamWaitEvent(ts, ev_ctl, 0));   // Ctl::grown is set before any top-up CTA runs
    if (debug_on()) {
      cudaEvent_t ev;
      CK(ctx, cudaEventCreate(&ev));
      CK(ctx, cudaEventRecord(ev, ts));
      r->dbg.push_back({'T', q - r->provisioned, ev});
    }
    t_d = debug_on() ? host_us(ctx) : 0.0;
    CK(ctx, cudaLaunchKernel(k.tfn, dim3(q - r->provisioned, 1, 1), k.block, params, k.dyn_smem, ts));
    t_e = debug_on() ? host_us(ctx) : 0.0;
    cudaEvent_t ev;
    CK(ctx, ctx->get_event(&ev));
    r->ev_topups.push_back(ev);
    CK(ctx, cudaEventRecord(ev, ts));
    r->provisioned = q;
  }
  if (debug_on())
    std::fprintf(stderr, "[accel] apply_quota us: wait %.1f memcpy %.1f prep %.1f launch %.1f rest %.1f\n", t_b - t_a,
                 t_c - t_b, t_d - t_c, t_e - t_d, host_us(ctx) - t_e);
  // the CTAs a shrink evicts leave the running launch: a later growth must top up again
  if (q < r->live) r->provisioned = std::min(r->provisioned, q);
  r->live = q;
  r->resolves += 1;
  r->quota_min = std::min(r->quota_min, q);
  r->quota_max = std::max(r->quota_max, q);
  return ACCEL_OK;
}

// Solve over the active requests (arrival order) + the new ones.  STATIC:
// running requests keep their quota and only the new
// ones are assigned.  RESOLVE: every active request gets its new quota.
int assign_quotas(accel_ctx* ctx, std::vector<std::unique_ptr<Request>>& fresh) {
  std::vector<Request*> order;
  for (auto& kv : ctx->reqs) {
    Request* r = kv.second.get();
    int rc = refresh_done(ctx, r);
    if (rc) return rc;
    if (!r->done && r->mode == ACCEL_MODE_SHARED) order.push_back(r);
  }
  for (auto& r : fresh) order.push_back(r.get());
  if (order.empty()) return ACCEL_OK;
  std::vector<accel_demand> ds(order.size());
  for (size_t i = 0; i < order.size(); ++i) {
    Request* r = order[i];
    int rc = demand_for(ctx, r->steps[r->main_step], r->weight, &ds[i], order.size() > 1);
    if (rc) return ctx->fail(rc, "kernel does not fit on an SM");
  }
  std::vector<uint32_t> q(order.size());
  int rc = accel_solve(&ctx->caps, ds.data(), (int32_t)ds.size(), q.data());
  if (rc) return ctx->fail(rc, "accel_solve failed");
  ctx->monitor_solves += 1;
  const size_t first_new = order.size() - fresh.size();
  if (is_resolve(ctx->cfg.policy))
    for (size_t i = 0; i < first_new; ++i) {
      rc = apply_quota(ctx, order[i], q[i]);
      if (rc) return rc;
    }
  for (size_t i = first_new; i < order.size(); ++i) {
    Request* r = order[i];
    for (size_t j = 0; j < r->steps.size(); ++j) {
      Step& s = r->steps[j];
      if ((int)j == r->main_step) {
        s.quota = q[i];
      } else {
        // R-solver-8: a secondary step is solved against the same active set,
        // with this request represented by the step's own kernel
        std::vector<accel_demand> dsj = ds;
        rc = demand_for(ctx, s, r->weight, &dsj[i], order.size() > 1);
        if (rc) return ctx->fail(rc, "kernel does not fit on an SM");
        std::vector<uint32_t> qj(order.size());
        rc = accel_solve(&ctx->caps, dsj.data(), (int32_t)dsj.size(), qj.data());
        if (rc) return ctx->fail(rc, "accel_solve failed");
        s.quota = qj[i];
      }
    }
    if (const char* e = std::getenv("ACCEL_QUOTA_MULT")) {
      // experiment knob (scripts/vg_trace.py): oversubscribe every step's grid
      // by a factor, e.g. a multiple large enough for one VG per CTA
      const double m = std::atof(e);
      for (Step& s : r->steps) s.quota = (uint32_t)std::min<double>(s.total, std::max(1.0, s.quota * m));
      q[i] = r->steps[r->main_step].quota;
    }
    r->quota_initial = r->quota_min = r->quota_max = q[i];
    r->live = r->provisioned = q[i];
  }
  return ACCEL_OK;
}

// Host monitor (RESOLVE): detects departures without host synchronisation by
// polling the requests' completion events, and re-solves the survivors.
double host_us(const accel_ctx* ctx) {
  return std::chrono::duration<double, std::micro>(std::chrono::steady_clock::now() - ctx->t_init).count();
}

void monitor_loop(accel_ctx* ctx) {
  cudaSetDevice(ctx->cfg.device);
  bool busy = false;
  while (!ctx->stop.load()) {
    std::this_thread::sleep_for(std::chrono::microseconds(busy ? 20 : 500));
    std::unique_lock<std::mutex> g(ctx->mu);
    busy = false;
    if (ctx->poisoned || ctx->cfg.mode != ACCEL_MODE_SHARED || ctx->cfg.policy == ACCEL_POLICY_STATIC)
      continue;
    bool departed = false, running = false;
    for (auto& kv : ctx->reqs) {
      Request* r = kv.second.get();
      if (r->mode != ACCEL_MODE_SHARED || r->departed_seen) continue;
      if (refresh_done(ctx, r)) break;
      if (r->done) {
        r->departed_seen = true;
        departed = true;
      } else {
        running = true;
      }
    }
    busy = running;
    if (departed && debug_on()) std::fprintf(stderr, "[accel] monitor: departure (running=%d) at host %.1f us\n",
                                             (int)running, host_us(ctx));
    if (departed && running) {
      std::vector<std::unique_ptr<Request>> none;
      assign_quotas(ctx, none);
      if (debug_on()) std::fprintf(stderr, "[accel] monitor: re-solved at host %.1f us\n", host_us(ctx));
    }
  }
}

int submit_locked(accel_ctx* ctx, uint32_t n, const accel_request* rs, uint64_t* ids) {
  if (ctx->poisoned) return ACCEL_ESTATE;
  CK(ctx, cudaSetDevice(ctx->cfg.device));
  std::vector<std::unique_ptr<Request>> fresh(n);
  for (uint32_t i = 0; i < n; ++i) {
    int rc = build_request(ctx, rs[i], &fresh[i]);
    if (rc) return rc;
  }
  if (ctx->cfg.mode == ACCEL_MODE_SHARED) {
    int rc = assign_quotas(ctx, fresh);
    if (rc) return rc;
  } else {
    for (auto& r : fresh) r->quota_initial = r->quota_min = r->quota_max = r->steps[r->main_step].total;
  }
  // resources
  for (uint32_t i = 0; i < n; ++i) {
    Request* r = fresh[i].get();
    const int64_t s = ctx->alloc_slots(r->n_desc);
    if (s < 0) {
      for (uint32_t j = 0; j < i; ++j) ctx->free_slots(fresh[j]->slot, fresh[j]->n_desc);
      return ctx->fail(ACCEL_ENOMEM, "descriptor pool exhausted (release finished requests)");
    }
    r->slot = (uint32_t)s;
    if (r->cov_elems) CK(ctx, ctx->buf_get(reinterpret_cast<void**>(&r->cov), r->cov_elems * sizeof(uint32_t)));
    if (r->trace_elems)
      CK(ctx, ctx->buf_get(reinterpret_cast<void**>(&r->trace), r->trace_elems * sizeof(accel_vg_record)));
  }
  // SHARED: requests that arrive together are enqueued largest per-CTA
  // footprint first (dominant share of one SM, DESIGN.md R-place-1).  The
  // block scheduler places each grid breadth-first over the SMs with room
  // left; the solver's packing (F) puts ceil(n_i / S) CTAs of every kernel
  // on an SM, which a big-CTA kernel (tensor-core sgemm: one CTA per SM by
  // shared memory) only gets if it is placed before small CTAs fragment the
  // SMs -- otherwise it waits for a whole co-runner to finish.  NATIVE keeps
  // the mix order (its FCFS winner is the point of the baseline).
  std::vector<int32_t> ord(n);
  for (uint32_t i = 0; i < n; ++i) ord[i] = (int32_t)i;
  if (ctx->cfg.mode == ACCEL_MODE_SHARED && n > 1) {
    std::vector<accel_demand> ds(n);
    bool ok = true;
    for (uint32_t i = 0; i < n; ++i)
      ok = ok && demand_for(ctx, fresh[i]->steps[fresh[i]->main_step], 1, &ds[i]) == ACCEL_OK;
    if (ok && accel_placement_order(&ctx->caps, ds.data(), (int32_t)n, ord.data()) != ACCEL_OK)
      for (uint32_t i = 0; i < n; ++i) ord[i] = (int32_t)i;
  }
  // ids (= arrival order for later re-solves) follow the array order
  const uint64_t base = ctx->next_id;
  ctx->next_id += n;
  std::vector<Request*> in_order;
  for (int32_t i : ord) in_order.push_back(fresh[(size_t)i].get());
  int rc = enqueue_group(ctx, in_order);
  for (uint32_t i = 0; i < n; ++i) {
    Request* r = fresh[i].get();
    r->id = base + (uint64_t)i;
    ids[i] = r->id;
    ctx->reqs[r->id] = std::move(fresh[i]);
  }
  return rc;
}

void release_request(accel_ctx* ctx, Request* r) {
  ctx->free_slots(r->slot, r->n_desc);
  if (r->cov) ctx->buf_put(r->cov, r->cov_elems * sizeof(uint32_t));
  if (r->trace) ctx->buf_put(r->trace, r->trace_elems * sizeof(accel_vg_record));
  if (r->ev_arrival) ctx->free_events.push_back(r->ev_arrival);
  if (r->ev_done) ctx->free_events.push_back(r->ev_done);
  if (r->ev_early) ctx->free_events.push_back(r->ev_early);
  if (r->ev_init) ctx->free_events.push_back(r->ev_init);
  for (cudaEvent_t ev : r->ev_launch) ctx->free_events.push_back(ev);
  for (cudaEvent_t ev : r->ev_topups) ctx->free_events.push_back(ev);
}

}  // namespace

extern "C" {

const char* accel_last_error(const accel_ctx* ctx) {
  return ctx ? ctx->err.c_str() : g_init_error.c_str();
}

bool policy_enabled(int32_t policy) {
  return policy == ACCEL_POLICY_STATIC || policy == ACCEL_POLICY_RESOLVE;
}

int accel_init(const accel_config* cfg, accel_ctx** out) {
  if (!cfg || !out) return ACCEL_EINVAL;
  if (cfg->mode != ACCEL_MODE_NATIVE && cfg->mode != ACCEL_MODE_SHARED) return ACCEL_EINVAL;
  if (!policy_enabled(cfg->policy)) {
    g_init_error = "bad policy";
    return ACCEL_EINVAL;
  }
  auto ctx = std::make_unique<accel_ctx>();
  ctx->cfg = *cfg;
  auto init_fail = [&](cudaError_t e, const char* what) {
    g_init_error = std::string(what) + ": " + cudaGetErrorString(e);
    return ACCEL_ECUDA;
  };
  cudaError_t e = cudaSetDevice(cfg->device);
  if (e != cudaSuccess) return init_fail(e, "cudaSetDevice");
  int sms = 0;
  e = cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, cfg->device);
  if (e != cudaSuccess) return init_fail(e, "cudaDeviceGetAttribute");
  ctx->caps = cfg->caps;
  if (ctx->caps.sms <= 0) ctx->caps.sms = sms;
  for (int t = 0; t < ACCEL_MAX_TENANTS; ++t)
    if ((e = cudaStreamCreateWithFlags(&ctx->main[t], cudaStreamNonBlocking)) != cudaSuccess)
      return init_fail(e, "cudaStreamCreate");
  for (int t = 0; t < accel_ctx::kTopupStreams; ++t)
    if ((e = cudaStreamCreateWithFlags(&ctx->topup[t], cudaStreamNonBlocking)) != cudaSuccess)
      return init_fail(e, "cudaStreamCreate");
  if ((e = cudaStreamCreateWithFlags(&ctx->ctl, cudaStreamNonBlocking)) != cudaSuccess)
    return init_fail(e, "cudaStreamCreate");
  if ((e = cudaStreamCreateWithFlags(&ctx->ostream, cudaStreamNonBlocking)) != cudaSuccess)
    return init_fail(e, "cudaStreamCreate");
  if ((e = cudaEventCreate(&ctx->epoch)) != cudaSuccess) return init_fail(e, "cudaEventCreate");
  if ((e = cudaMalloc(&ctx->pool, (size_t)kPoolSlots * kDescBytes)) != cudaSuccess)
    return init_fail(e, "cudaMalloc(pool)");
  if ((e = cudaMalloc(&ctx->ctl_pool, (size_t)kPoolSlots * kCtlBytes)) != cudaSuccess)
    return init_fail(e, "cudaMalloc(ctl)");
  if ((e = cudaHostAlloc(reinterpret_cast<void**>(&ctx->pinned_ring), kRing * sizeof(uint32_t),
                         cudaHostAllocDefault)) != cudaSuccess)
    return init_fail(e, "cudaHostAlloc(ring)");
  ctx->slot_used.assign(kPoolSlots, 0);
  if (const char* ab = std::getenv("ACCEL_ABLATE")) ctx->ablate = ((uint32_t)std::atoi(ab) & 31u) << 24;
  if (const char* pd = std::getenv("ACCEL_PDL")) ctx->pdl = std::atoi(pd) != 0;
  accel_ctx* raw = ctx.release();
  raw->monitor = std::thread(monitor_loop, raw);
  *out = raw;
  return ACCEL_OK;
}

int accel_finalize(accel_ctx* ctx) {
  if (!ctx) return ACCEL_OK;
  ctx->stop.store(true);
  if (ctx->monitor.joinable()) ctx->monitor.join();
  cudaSetDevice(ctx->cfg.device);
  for (auto& kv : ctx->reqs) {
    if (kv.second->ev_done) cudaEventSynchronize(kv.second->ev_done);
    for (cudaEvent_t ev : kv.second->ev_topups) cudaEventSynchronize(ev);
    release_request(ctx, kv.second.get());
  }
  ctx->reqs.clear();
  for (auto& kv : ctx->orders)
    if (kv.second.dev) cudaFree(kv.second.dev);
  ctx->orders.clear();
  for (cudaEvent_t ev : ctx->free_events) cudaEventDestroy(ev);
  for (int t = 0; t < ACCEL_MAX_TENANTS; ++t)
    if (ctx->main[t]) cudaStreamDestroy(ctx->main[t]);
  for (int t = 0; t < accel_ctx::kTopupStreams; ++t)
    if (ctx->topup[t]) cudaStreamDestroy(ctx->topup[t]);
  if (ctx->ctl) cudaStreamDestroy(ctx->ctl);
  if (ctx->ostream) cudaStreamDestroy(ctx->ostream);
  if (ctx->epoch) cudaEventDestroy(ctx->epoch);
  for (auto& kv : ctx->buf_pool) cudaFree(kv.second);
  if (ctx->pool) cudaFree(ctx->pool);
  if (ctx->ctl_pool) cudaFree(ctx->ctl_pool);
  if (ctx->pinned_ring) cudaFreeHost(ctx->pinned_ring);
  delete ctx;
  return ACCEL_OK;
}

int accel_set_mode(accel_ctx* ctx, int32_t mode, int32_t policy) {
  if (!ctx) return ACCEL_EINVAL;
  std::lock_guard<std::mutex> g(ctx->mu);
  if (ctx->poisoned) return ACCEL_ESTATE;
  if (mode != ACCEL_MODE_NATIVE && mode != ACCEL_MODE_SHARED) return ctx->fail(ACCEL_EINVAL, "bad mode");
  if (!policy_enabled(policy))
    return ctx->fail(ACCEL_EINVAL, "bad policy");
  for (auto& kv : ctx->reqs) {
    int rc = refresh_done(ctx, kv.second.get());
    if (rc) return rc;
    if (!kv.second->done) return ctx->fail(ACCEL_EINVAL, "requests still running");
  }
  ctx->cfg.mode = mode;
  ctx->cfg.policy = policy;
  return ACCEL_OK;
}

int accel_kernel_register(accel_ctx* ctx, const accel_kernel_desc* d, int32_t* kernel_id) {
  if (!ctx || !d || !kernel_id || !d->persistent_fn || !d->native_fn) return ACCEL_EINVAL;
  std::lock_guard<std::mutex> g(ctx->mu);
  if (ctx->poisoned) return ACCEL_ESTATE;
  CK(ctx, cudaSetDevice(ctx->cfg.device));
  Kernel k;
  k.name = d->name ? d->name : "?";
  k.pfn = d->persistent_fn;
  k.prfn = d->persistent_resolve_fn ? d->persistent_resolve_fn : d->persistent_fn;
  k.nfn = d->native_fn;
  k.tfn = d->topup_fn ? d->topup_fn : d->persistent_fn;
  k.ofn = d->order_fn;
  if (k.ofn)
    CK(ctx, cudaFuncSetAttribute(k.ofn, cudaFuncAttributeMaxDynamicSharedMemorySize,
                                 (int)(accel::kMaxOrderVGs * sizeof(unsigned long long))));
  k.block = dim3(d->block.x, d->block.y ? d->block.y : 1, d->block.z ? d->block.z : 1);
  k.dyn_smem = d->dyn_smem;
  k.chunk = d->chunk ? d->chunk : 1;
  k.args_size = d->args_size;
  // ACCEL_NO_OCC_CAP=1: ignore the useful-occupancy caps (A/B measurements)
  k.max_per_sm = std::getenv("ACCEL_NO_OCC_CAP") ? 0u : d->max_ctas_per_sm;
  k.slices = std::getenv("ACCEL_NO_SLICES") ? 1u : std::max<uint32_t>(1u, d->slices);
  if (const char* e = std::getenv("ACCEL_SLICES")) {   // experiment: "name:n,name:n"
    const std::string spec(e), key = k.name + ":";
    const size_t at = spec.find(key);
    if (at != std::string::npos && (at == 0 || spec[at - 1] == ','))
      k.slices = std::max<uint32_t>(1u, (uint32_t)std::atoi(spec.c_str() + at + key.size()));
  }
  cudaFuncAttributes a;
  CK(ctx, cudaFuncGetAttributes(&a, k.pfn));
  if ((int)k.threads() > a.maxThreadsPerBlock) return ctx->fail(ACCEL_ENOFIT, "block larger than the kernel allows");
  cudaFuncAttributes ar;
  CK(ctx, cudaFuncGetAttributes(&ar, k.prfn));
  // the solver uses the larger of the two persistent instances (the one a
  // request runs depends on the policy at submit time)
  k.num_regs = d->regs > 0 ? d->regs : std::max(a.numRegs, ar.numRegs);
  k.static_smem = (int)std::max(a.sharedSizeBytes, ar.sharedSizeBytes);
  for (const void* fn : {k.pfn, k.prfn, k.nfn, k.tfn}) {
    if (k.dyn_smem > 48 * 1024)
      CK(ctx, cudaFuncSetAttribute(fn, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)k.dyn_smem));
    // one carveout for every tenant so CTAs of different kernels can share an SM
    CK(ctx, cudaFuncSetAttribute(fn, cudaFuncAttributePreferredSharedMemoryCarveout, 100));
  }
  CK(ctx, cudaOccupancyMaxActiveBlocksPerMultiprocessor(&k.occ_p, k.pfn, (int)k.threads(), k.dyn_smem));
  CK(ctx, cudaOccupancyMaxActiveBlocksPerMultiprocessor(&k.occ_n, k.nfn, (int)k.threads(), k.dyn_smem));
  accel_demand dem;
  int rc = accel_demand_of(&ctx->caps, k.threads(), (uint32_t)k.num_regs,
                           (uint32_t)(k.static_smem + k.dyn_smem), 1, 1, &dem);
  if (rc) return ctx->fail(rc, "one CTA of " + k.name + " fits on no SM");
  ctx->kernels.push_back(k);
  *kernel_id = (int32_t)ctx->kernels.size() - 1;
  return ACCEL_OK;
}

int accel_kernel_info_get(accel_ctx* ctx, int32_t kernel_id, accel_kernel_info* out) {
  if (!ctx || !out) return ACCEL_EINVAL;
  std::lock_guard<std::mutex> g(ctx->mu);
  if (kernel_id < 0 || kernel_id >= (int)ctx->kernels.size()) return ctx->fail(ACCEL_EINVAL, "bad kernel_id");
  const Kernel& k = ctx->kernels[kernel_id];
  accel_demand dem;
  int rc = accel_demand_of(&ctx->caps, k.threads(), (uint32_t)k.num_regs,
                           (uint32_t)(k.static_smem + k.dyn_smem), 1, 1, &dem);
  if (rc) return rc;
  out->thr = dem.thr;
  out->regs = dem.regs;
  out->smem = dem.smem;
  out->cta = dem.cta;
  out->num_regs = k.num_regs;
  out->static_smem = k.static_smem;
  out->occ_persistent = k.occ_p;
  out->occ_native = k.occ_n;
  return ACCEL_OK;
}

int accel_submit_group(accel_ctx* ctx, uint32_t n, const accel_request* rs, uint64_t* ids) {
  if (!ctx || (n && (!rs || !ids))) return ACCEL_EINVAL;
  std::lock_guard<std::mutex> g(ctx->mu);
  if (debug_on()) std::fprintf(stderr, "[accel] submit %u requests at host %.1f us\n", n, host_us(ctx));
  const int rc = submit_locked(ctx, n, rs, ids);
  if (debug_on()) std::fprintf(stderr, "[accel] submit done at host %.1f us\n", host_us(ctx));
  return rc;
}

int accel_submit(accel_ctx* ctx, const accel_request* r, uint64_t* id) {
  return accel_submit_group(ctx, 1, r, id);
}

// Debug (ACCEL_SYNC_TIMEOUT_S): print every unfinished request's launches as
// the device sees them (descriptors copied on a fresh stream by the copy
// engine, which works while kernels spin).
void dump_stuck(accel_ctx* ctx, const std::vector<uint64_t>& ids) {
  cudaStream_t st;
  if (cudaStreamCreateWithFlags(&st, cudaStreamNonBlocking) != cudaSuccess) return;
  for (uint64_t id : ids) {
    auto it = ctx->reqs.find(id);
    if (it == ctx->reqs.end()) continue;
    Request* r = it->second.get();
    if (cudaEventQuery(r->ev_done) == cudaSuccess) continue;
    std::vector<unsigned char> h((size_t)r->n_desc * kDescBytes);
    uint32_t ctl[2] = {0, 0};
    void* hp = nullptr;
    if (cudaHostAlloc(&hp, h.size() + 256, cudaHostAllocDefault) != cudaSuccess) break;
    cudaMemcpyAsync(hp, ctx->desc_ptr(r->slot), h.size(), cudaMemcpyDeviceToHost, st);
    cudaMemcpyAsync((char*)hp + h.size(), ctx->ctl_pool + (size_t)r->slot * kCtlBytes, 256, cudaMemcpyDeviceToHost, st);
    const auto t0 = std::chrono::steady_clock::now();
    while (cudaStreamQuery(st) == cudaErrorNotReady &&
           std::chrono::steady_clock::now() - t0 < std::chrono::seconds(5))
      std::this_thread::sleep_for(std::chrono::milliseconds(1));
    std::memcpy(h.data(), hp, h.size());
    std::memcpy(ctl, (char*)hp + h.size(), sizeof(uint32_t));
    std::memcpy(ctl + 1, (char*)hp + h.size() + 128, sizeof(uint32_t));
    cudaFreeHost(hp);
    std::fprintf(stderr, "[accel] STUCK req %llu tenant %d live(host) %u provisioned %u topups %zu | ctl live %u cur %u\n",
                 (unsigned long long)id, r->tenant, r->live, r->provisioned, r->ev_topups.size(), ctl[0], ctl[1]);
    for (uint32_t l = 0; l < r->n_desc; ++l) {
      const DescHost* d = reinterpret_cast<const DescHost*>(h.data() + (size_t)l * kDescBytes);
      const uint32_t next = (uint32_t)d->qa, alive = (uint32_t)(d->qa >> 32);
      // (main-grid CTAs retire without decrementing `alive`: dispatch.cuh)
      if (d->total_seen != 0xffffffffu && next >= d->total_seen && d->tu_alive == 0 && d->draining == 0) continue;
      std::fprintf(stderr, "[accel]   launch %u: total %u seen %u next %u alive %u tu_alive %u draining %u topped %u "
                           "started %u refused %u evicted %u\n", l, d->total, d->total_seen, next, alive, d->tu_alive,
                   d->draining, d->topped, d->ctas_started, d->admit_fail, d->evicted);
    }
  }
  cudaStreamDestroy(st);
}

int accel_sync(accel_ctx* ctx, uint64_t request_id) {
  if (!ctx) return ACCEL_EINVAL;
  std::vector<uint64_t> ids;
  // Wait without holding the lock (the RESOLVE monitor keeps re-solving
  // meanwhile); it may add top-up grids to a request while we wait, so repeat
  // until every event of every request is complete.
  for (;;) {
    std::vector<cudaEvent_t> wait;
    {
      std::lock_guard<std::mutex> g(ctx->mu);
      if (ctx->poisoned) return ACCEL_ESTATE;
      CK(ctx, cudaSetDevice(ctx->cfg.device));
      ids.clear();
      if (request_id == ACCEL_ALL) {
        for (auto& kv : ctx->reqs) ids.push_back(kv.first);
      } else {
        if (ctx->reqs.find(request_id) == ctx->reqs.end()) return ctx->fail(ACCEL_EINVAL, "unknown request");
        ids.push_back(request_id);
      }
      for (uint64_t id : ids) {
        Request* r = ctx->reqs[id].get();
        int rc = refresh_done(ctx, r);
        if (rc) return rc;
        if (r->done) continue;
        wait.push_back(r->ev_done);
        for (cudaEvent_t ev : r->ev_topups) wait.push_back(ev);
      }
    }
    if (wait.empty()) break;
    static const double watchdog_s = std::getenv("ACCEL_SYNC_TIMEOUT_S") ? std::atof(std::getenv("ACCEL_SYNC_TIMEOUT_S")) : 0.0;
    const auto t0 = std::chrono::steady_clock::now();
    for (cudaEvent_t ev : wait) {
      cudaError_t e;
      if (watchdog_s > 0.0) {   // debug: poll, and on timeout dump the launches' device state
        while ((e = cudaEventQuery(ev)) == cudaErrorNotReady) {
          if (std::chrono::duration<double>(std::chrono::steady_clock::now() - t0).count() > watchdog_s) {
            std::lock_guard<std::mutex> g(ctx->mu);
            dump_stuck(ctx, ids);
            return ctx->fail(ACCEL_ESTATE, "accel_sync watchdog: requests did not complete (state dumped to stderr)");
          }
          std::this_thread::sleep_for(std::chrono::microseconds(200));
        }
      } else {
        e = cudaEventSynchronize(ev);
      }
      if (e != cudaSuccess) {
        std::lock_guard<std::mutex> g(ctx->mu);
        return ctx->cuda(e, "cudaEventSynchronize");
      }
    }
  }
  std::lock_guard<std::mutex> g(ctx->mu);
  bool cov_bad = false;
  for (uint64_t id : ids) {
    auto it = ctx->reqs.find(id);
    if (it == ctx->reqs.end()) continue;
    Request* r = it->second.get();
    int rc = refresh_done(ctx, r);
    if (rc) return rc;
    if (!r->done) return ctx->fail(ACCEL_ESTATE, "request not complete after sync");
    rc = fetch_result(ctx, r);
    if (rc) return rc;
    if (r->cov_ok == 0) cov_bad = true;
  }
  if (cov_bad) return ctx->fail(ACCEL_ECOVERAGE, "a virtual group did not run exactly once");
  return ACCEL_OK;
}

int accel_epoch(accel_ctx* ctx) {
  if (!ctx) return ACCEL_EINVAL;
  std::lock_guard<std::mutex> g(ctx->mu);
  if (ctx->poisoned) return ACCEL_ESTATE;
  CK(ctx, cudaSetDevice(ctx->cfg.device));
  CK(ctx, cudaEventRecord(ctx->epoch, ctx->ctl));
  ctx->epoch_set = true;
  return ACCEL_OK;
}

int accel_stats(accel_ctx* ctx, uint64_t request_id, accel_req_stats* out) {
  if (!ctx || !out) return ACCEL_EINVAL;
  std::lock_guard<std::mutex> g(ctx->mu);
  if (ctx->poisoned) return ACCEL_ESTATE;
  auto it = ctx->reqs.find(request_id);
  if (it == ctx->reqs.end()) return ctx->fail(ACCEL_EINVAL, "unknown request");
  Request* r = it->second.get();
  int rc = refresh_done(ctx, r);
  if (rc) return rc;
  if (!r->done) return ACCEL_ENOTREADY;
  rc = fetch_result(ctx, r);
  if (rc) return rc;
  std::memset(out, 0, sizeof(*out));
  CK(ctx, cudaEventElapsedTime(&out->elapsed_ms, r->ev_arrival, r->ev_done));
  if (ctx->epoch_set) {
    CK(ctx, cudaEventElapsedTime(&out->arrival_ms, ctx->epoch, r->ev_arrival));
    CK(ctx, cudaEventElapsedTime(&out->done_ms, ctx->epoch, r->ev_done));
  }
  unsigned long long first = ~0ull, last = 0;
  uint32_t max_ctas = 0, launches = 0, vgs = 0;
  for (uint32_t i = 0; i < r->n_desc; ++i) {
    const DescHost* d = reinterpret_cast<const DescHost*>(r->desc_host.data() + (size_t)i * kDescBytes);
    first = std::min(first, d->t_first);
    last = std::max(last, d->t_last);
    max_ctas = std::max(max_ctas, d->max_alive);
    vgs += d->total;
    ++launches;
  }
  out->first_start_ns = first;
  out->last_end_ns = last;
  out->vgs_total = vgs;
  out->launches = launches;
  out->quota_initial = r->quota_initial;
  out->quota_min = r->quota_min;
  out->quota_max = r->quota_max;
  out->resolves = r->resolves;
  out->max_ctas = max_ctas;
  out->coverage_ok = r->cov_ok;
  out->mode = r->mode;
  return ACCEL_OK;
}

int accel_launch_times(accel_ctx* ctx, uint64_t request_id, float* ms_out, uint32_t n, uint32_t* n_out) {
  if (!ctx || (n && !ms_out) || !n_out) return ACCEL_EINVAL;
  std::lock_guard<std::mutex> g(ctx->mu);
  if (ctx->poisoned) return ACCEL_ESTATE;
  auto it = ctx->reqs.find(request_id);
  if (it == ctx->reqs.end()) return ctx->fail(ACCEL_EINVAL, "unknown request");
  Request* r = it->second.get();
  int rc = refresh_done(ctx, r);
  if (rc) return rc;
  if (!r->done) return ACCEL_ENOTREADY;
  if (r->ev_launch.empty()) return ctx->fail(ACCEL_EINVAL, "request had no ACCEL_REQ_LAUNCH_EVENTS");
  const uint32_t m = std::min<uint32_t>(n, r->n_desc);
  for (uint32_t i = 0; i < m; ++i)
    CK(ctx, cudaEventElapsedTime(&ms_out[i], r->ev_launch[i], r->ev_launch[i + 1]));
  *n_out = m;
  return ACCEL_OK;
}

int accel_launch_stats(accel_ctx* ctx, uint64_t request_id, accel_launch_stat* out, uint32_t n,
                       uint32_t* n_out) {
  if (!ctx || (n && !out) || !n_out) return ACCEL_EINVAL;
  std::lock_guard<std::mutex> g(ctx->mu);
  if (ctx->poisoned) return ACCEL_ESTATE;
  auto it = ctx->reqs.find(request_id);
  if (it == ctx->reqs.end()) return ctx->fail(ACCEL_EINVAL, "unknown request");
  Request* r = it->second.get();
  int rc = refresh_done(ctx, r);
  if (rc) return rc;
  if (!r->done) return ACCEL_ENOTREADY;
  rc = fetch_result(ctx, r);
  if (rc) return rc;
  const uint32_t m = std::min<uint32_t>(n, r->n_desc);
  for (uint32_t i = 0; i < m; ++i) {
    const DescHost* d = reinterpret_cast<const DescHost*>(r->desc_host.data() + (size_t)i * kDescBytes);
    out[i].t_first_ns = d->t_first;
    out[i].t_last_ns = d->t_last;
    out[i].ctas_started = d->ctas_started;
    out[i].max_alive = d->max_alive;
    out[i].total = d->total_seen;
    out[i].topped = d->topped;
  }
  *n_out = m;
  return ACCEL_OK;
}

int accel_vg_trace(accel_ctx* ctx, uint64_t request_id, accel_vg_record* out, uint64_t n, uint64_t* n_out) {
  if (!ctx || (n && !out) || !n_out) return ACCEL_EINVAL;
  std::lock_guard<std::mutex> g(ctx->mu);
  if (ctx->poisoned) return ACCEL_ESTATE;
  auto it = ctx->reqs.find(request_id);
  if (it == ctx->reqs.end()) return ctx->fail(ACCEL_EINVAL, "unknown request");
  Request* r = it->second.get();
  if (!r->trace) return ctx->fail(ACCEL_EINVAL, "request was not submitted with ACCEL_REQ_TRACE");
  int rc = refresh_done(ctx, r);
  if (rc) return rc;
  if (!r->done) return ACCEL_ENOTREADY;
  const uint64_t m = std::min<uint64_t>(n, r->trace_elems);
  if (m) CK(ctx, cudaMemcpy(out, r->trace, m * sizeof(accel_vg_record), cudaMemcpyDeviceToHost));
  *n_out = r->trace_elems;
  return ACCEL_OK;
}

int accel_dequeue_order(accel_ctx* ctx, int32_t kernel_id, const accel_dim3* grid, const void* args,
                        uint32_t args_size, uint32_t* order_device) {
  if (!ctx || !grid || !args || !order_device) return ACCEL_EINVAL;
  std::lock_guard<std::mutex> g(ctx->mu);
  if (ctx->poisoned) return ACCEL_ESTATE;
  if (kernel_id < 0 || kernel_id >= (int)ctx->kernels.size()) return ctx->fail(ACCEL_EINVAL, "bad kernel_id");
  const Kernel& k = ctx->kernels[kernel_id];
  if (!k.ofn) return ctx->fail(ACCEL_EINVAL, k.name + " has no cost model");
  if (args_size != k.args_size) return ctx->fail(ACCEL_EINVAL, "args_size mismatch for " + k.name);
  const uint64_t total = (uint64_t)grid->x * grid->y * grid->z;
  if (total == 0 || total > accel::kMaxOrderVGs) return ctx->fail(ACCEL_EINVAL, "grid too large for a cost order");
  CK(ctx, cudaSetDevice(ctx->cfg.device));
  uint32_t gx = grid->x, gy = grid->y, gz = grid->z;
  void* params[5] = {const_cast<void*>(args), &gx, &gy, &gz, &order_device};
  CK(ctx, cudaLaunchKernel(k.ofn, dim3(1), dim3(accel::kOrderThreads), params,
                           accel::kMaxOrderVGs * sizeof(unsigned long long), ctx->ostream));
  CK(ctx, cudaStreamSynchronize(ctx->ostream));
  return ACCEL_OK;
}

int accel_release(accel_ctx* ctx, uint64_t request_id) {
  if (!ctx) return ACCEL_EINVAL;
  std::lock_guard<std::mutex> g(ctx->mu);
  for (auto it = ctx->reqs.begin(); it != ctx->reqs.end();) {
    Request* r = it->second.get();
    if (request_id != ACCEL_ALL && it->first != request_id) {
      ++it;
      continue;
    }
    int rc = refresh_done(ctx, r);
    if (rc) return rc;
    if (!r->done) {
      if (request_id != ACCEL_ALL) return ctx->fail(ACCEL_EINVAL, "request still running");
      ++it;
      continue;
    }
    release_request(ctx, r);
    it = ctx->reqs.erase(it);
  }
  return ACCEL_OK;
}

int accel_tenant_stream(accel_ctx* ctx, int32_t tenant, void** main_stream, void** topup_stream) {
  if (!ctx || tenant < 0 || tenant >= ACCEL_MAX_TENANTS) return ACCEL_EINVAL;
  if (main_stream) *main_stream = ctx->main[tenant];
  if (topup_stream) *topup_stream = ctx->topup[tenant % accel_ctx::kTopupStreams];
  return ACCEL_OK;
}

}  // extern "C"
