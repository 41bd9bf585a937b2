/*
 * accel.h -- C ABI of the B200-native accelOS hot path (libaccel.so).
 *
 * The method: Margiolas & O'Boyle, "Portable and Transparent Software Managed
 * Scheduling on Accelerators for Fair Resource Sharing", CGO'16.
 * A tenant issues *kernel execution requests* -- a kernel plus its NDRange
 * (§5 "Kernel Scheduler", lines 647-655).  In SHARED mode the library
 *   1. sizes the request's persistent CTA quota with the resource-sharing
 *      algorithm of §3 (lines 483-542) over all active requests,
 *   2. builds the Virtual NDRange (descriptor) in device memory (lines 650-652),
 *   3. launches the reduced grid with the block shape unchanged (lines 652-655),
 *      and the persistent CTAs dequeue virtual groups until the original grid
 *      is covered (§2.4, Fig. 8b).
 * In NATIVE mode it launches the original grid on the tenant's stream -- the
 * "standard" hardware FCFS sharing of Fig. 1a / §2.3 (lines 394-438).
 *
 * Conventions (every entry point):
 *   - returns int: ACCEL_OK (0) or a negative ACCEL_E* code; nothing throws or
 *     aborts across the ABI; accel_last_error() gives a message.
 *   - a sticky CUDA error poisons the context: every later call returns
 *     ACCEL_ESTATE (except accel_last_error / accel_finalize).
 *   - all pointers are plain host pointers unless named "device"; device
 *     buffers are owned by the caller (e.g. PyTorch tensors) and must stay
 *     alive until accel_sync() returned for every request that uses them.
 *   - one context per device; all entry points are serialised by a mutex, so
 *     tenants may submit from different host threads.
 */
#ifndef ACCEL_H_
#define ACCEL_H_

#include <stddef.h>
#include <stdint.h>

#ifdef __cplusplus
extern "C" {
#endif

enum {
  ACCEL_OK = 0,
  ACCEL_EINVAL = -1,     /* bad argument                                       */
  ACCEL_ENOFIT = -2,     /* one CTA of the kernel fits on no SM                */
  ACCEL_ECUDA = -3,      /* a CUDA runtime call failed (see accel_last_error)  */
  ACCEL_ESTATE = -4,     /* context poisoned by an earlier CUDA error           */
  ACCEL_ECOVERAGE = -5,  /* verify mode: a virtual group ran != 1 times         */
  ACCEL_ENOMEM = -6,     /* descriptor pool / host allocation exhausted        */
  ACCEL_ENOTREADY = -7   /* accel_stats before the request completed           */
};

typedef enum { ACCEL_MODE_NATIVE = 0, ACCEL_MODE_SHARED = 1 } accel_mode;
/* STATIC: a quota is fixed at launch (§2.5, "bound to
 * the resources initially allocated").  RESOLVE: quotas are recomputed on every
 * arrival and departure (BASELINE.json north star): shrinking lowers a live
 * quota word read at each dequeue, growing launches extra CTAs.
 * (Values 2 and 3 are retired: an SM-granular PARTITION policy and a
 * slowdown-feedback FAIR policy were measured in round 1 -- PARTITION at half
 * the native throughput on C2, FAIR below RESOLVE on the sampled 4-mixes --
 * and removed.) */
typedef enum {
  ACCEL_POLICY_STATIC = 0,
  ACCEL_POLICY_RESOLVE = 1
} accel_policy;

#define ACCEL_ALL UINT64_MAX
#define ACCEL_MAX_TENANTS 16
#define ACCEL_MAX_STEPS 8

typedef struct { uint32_t x, y, z; } accel_dim3;

/* Per-SM device limits the solver works with (§3: T, L, R, plus the
 * CTA-slot limit); a field <= 0 means "query the device" (sms) or the B200
 * default (148 SMs, 2048 threads, 65536 registers, 233472 B shared memory,
 * 32 CTAs per SM). */
typedef struct {
  int32_t sms, thr_per_sm, regs_per_sm, smem_per_sm, ctas_per_sm;
} accel_caps;

typedef struct {
  int32_t device;   /* CUDA ordinal                                          */
  int32_t mode;     /* accel_mode                                            */
  int32_t policy;   /* accel_policy                                          */
  int32_t verify;   /* 1: per-VG coverage counters, checked at accel_sync    */
  accel_caps caps;  /* solver caps (0 = device / B200 default)               */
} accel_config;

typedef struct accel_ctx accel_ctx;

/* Create the context on cfg->device: per-tenant streams (main + top-up, non
 * blocking), the descriptor pool, events.  *out owned by the library; free
 * with accel_finalize. */
int accel_init(const accel_config *cfg, accel_ctx **out);
/* Wait for all requests, release everything.  NULL is a no-op. */
int accel_finalize(accel_ctx *ctx);
/* Switch NATIVE <-> SHARED or the policy; only while no request is running. */
int accel_set_mode(accel_ctx *ctx, int32_t mode, int32_t policy);
/* Last error message of ctx (or of the last failed accel_init when NULL).
 * Valid until the next call on ctx. */
const char *accel_last_error(const accel_ctx *ctx);

/* ---- kernels -------------------------------------------------------------
 * A kernel is a pair of __global__ instantiations compiled into this library
 * (accel_persistent<T> / accel_native<T>, see csrc/device/dispatch.cuh) plus
 * its block shape.  The block shape is never changed. */
typedef struct {
  const char *name;
  const void *persistent_fn;  /* host stub of accel_persistent<T, STATIC>      */
  const void *persistent_resolve_fn; /* accel_persistent<T, RESOLVE>; NULL = persistent_fn */
  const void *native_fn;      /* host stub of accel_native<T>                  */
  const void *topup_fn;       /* host stub of accel_topup<T> (RESOLVE growth)  */
  accel_dim3 block;           /* work-group (CTA) shape                        */
  uint32_t dyn_smem;          /* dynamic shared memory per CTA, bytes          */
  int32_t regs;               /* regs/thread for the solver; 0 = query attrs   */
  uint32_t chunk;             /* VGs per dequeue (§6.4); 0 = default  */
  uint32_t args_size;         /* sizeof the kernel's argument struct           */
  const void *order_fn;       /* host stub of accel_lpt_order<T>: the kernel's
                                 dequeue-order cost model (T::vg_cost); NULL =
                                 none (linear dequeue order)                    */
  uint32_t max_ctas_per_sm;   /* useful occupancy (T::kMaxCtasPerSm): the fewest
                                 resident CTAs per SM at which the kernel alone
                                 reaches >= 90 % of its full-device speed
                                 (measured, scripts/occ_scaling.py).  While the
                                 request shares the device the solver gives it
                                 at most this x SMs -- the paper's greedy fill
                                 "until resource saturation" (PAPER.md lines
                                 538-541) stops at the kernel's own saturation
                                 and the rest goes to its co-runners; alone it
                                 keeps its full share.  0 = no cap.  SHARED
                                 only (DESIGN.md R-solver-10). */
  uint32_t slices;            /* SHARED: run a single launch as this many
                                 sub-launches over consecutive VG ranges
                                 (T::kSlices; 0/1 = none).  The sub-launches
                                 overlap (no dependence between them) and the
                                 last one retires after all of them, so a
                                 long persistent request gets fresh CTAs --
                                 and fresh warp ages -- at every slice
                                 (DESIGN.md R-disp-9). */
} accel_kernel_desc;

/* Fill *out with a built-in tenant kernel: "mop", "stencil", "histo", "bfs",
 * "cutcp", "tpacf", "spmv", "sgemm", "mriq_phimag", "mriq_q".  Pure lookup,
 * no CUDA call.  Returns ACCEL_EINVAL for an unknown name. */
int accel_builtin_kernel(const char *name, accel_kernel_desc *out);
/* Number of built-in kernels and the i-th name (for enumeration). */
int accel_builtin_count(void);
const char *accel_builtin_name(int i);

/* Register a kernel with ctx: queries its attributes, sets the maximum
 * shared-memory carveout (all tenants share one carveout so CTAs of different
 * kernels can co-reside) and computes the per-CTA demand vector.
 * Returns ACCEL_ENOFIT if one CTA cannot fit on an SM. */
int accel_kernel_register(accel_ctx *ctx, const accel_kernel_desc *d, int32_t *kernel_id);

typedef struct {
  uint32_t thr, regs, smem, cta;  /* per-CTA demand (threads, regs, bytes, 1)  */
  int32_t num_regs;               /* regs/thread of the persistent instance    */
  int32_t static_smem;            /* static shared memory of the instance      */
  int32_t occ_persistent;         /* cudaOccupancyMaxActiveBlocksPerMultiprocessor */
  int32_t occ_native;
} accel_kernel_info;
int accel_kernel_info_get(accel_ctx *ctx, int32_t kernel_id, accel_kernel_info *out);

/* ---- requests ------------------------------------------------------------
 * A request is what one tenant enqueues in one go: optional memsets and
 * host->device copies, then a sequence of steps (each: one kernel launched
 * `repeat` times over the same NDRange, e.g. the sweeps of a stencil or the
 * levels of a BFS), then optional device->host copies.  All of it runs in
 * order on the tenant's stream; requests of the same tenant serialise.
 * args are copied at submit.  Launch r of a step sees VirtualBlock::launch_idx
 * = r.  grid = the ORIGINAL number of work-groups (the NDRange / block).    */
typedef struct {
  int32_t kernel_id;
  accel_dim3 grid;       /* original grid of virtual groups                      */
  const void *args;      /* points to the kernel's argument struct (copied)      */
  uint32_t args_size;    /* must equal the registered args_size                  */
  uint32_t repeat;       /* launches of this step, >= 1                          */
  const uint32_t *order_device; /* dequeue order (SHARED mode): the t-th VG handed out
                           is order_device[t], a permutation of 0..G-1 in device
                           memory, caller-owned; NULL = the kernel's own order:
                           most expensive VGs first by its cost model when it has
                           one (order_fn; G <= 8192), computed on the device by
                           the library once per distinct (kernel, grid, args)
                           and cached -- any permutation is correct, so a cached
                           order only affects speed -- else increasing linear
                           order.  Static-grid kernels only.  NATIVE mode ignores
                           it (hardware order).                                    */
} accel_launch;

typedef struct { void *dst_device; int32_t value; uint64_t bytes; } accel_clear;
typedef struct { void *dst; const void *src; uint64_t bytes; } accel_copy; /* host<->device */

/* accel_request.flags */
#define ACCEL_REQ_LAUNCH_EVENTS 1u  /* record a CUDA event around every launch
                                       (per-launch device times via accel_launch_times) */
#define ACCEL_REQ_TRACE 2u          /* record one accel_vg_record per virtual group
                                       (accel_vg_trace); costs one %globaltimer
                                       pair and a 24-B store per VG */
#define ACCEL_REQ_LINEAR_ORDER 4u   /* ignore the kernels' cost models: steps
                                       without order_device dequeue linearly */

typedef struct {
  int32_t tenant;             /* 0..ACCEL_MAX_TENANTS-1: selects the stream pair */
  uint32_t flags;             /* ACCEL_REQ_* */
  uint32_t weight;            /* sharing ratio (§2.2); 0 -> 1          */
  int32_t main_step;          /* step that represents the request in the solver
                                 (its main computation); -1 = the step with the
                                 most virtual groups.  Every other step is solved
                                 against the same active set with its own kernel */
  uint32_t n_steps;           /* 1..ACCEL_MAX_STEPS                             */
  const accel_launch *steps;
  uint32_t n_clear;           /* memsets before the first launch                */
  const accel_clear *clear;
  uint32_t n_h2d;             /* host->device copies (pinned src for async)     */
  const accel_copy *h2d;
  uint32_t n_d2h;             /* device->host copies after the last launch      */
  const accel_copy *d2h;
} accel_request;

/* Submit one request (solver run over the active set incl. this one).
 * Non-blocking; *request_id identifies it for sync/stats. */
int accel_submit(accel_ctx *ctx, const accel_request *r, uint64_t *request_id);
/* Submit n requests that arrive together: ONE solve over all of them.
 * NATIVE mode enqueues them in array order (the mix order decides the FCFS
 * winner); SHARED mode enqueues the largest per-CTA
 * footprint first (DESIGN.md R-place-1).  request_ids[n] out, in array order
 * (ids are the arrival order of later re-solves). */
int accel_submit_group(accel_ctx *ctx, uint32_t n, const accel_request *rs, uint64_t *request_ids);
/* Block until request_id (or every request: ACCEL_ALL) completed.  In verify
 * mode also checks coverage -> ACCEL_ECOVERAGE.  Debug: with the environment
 * variable ACCEL_SYNC_TIMEOUT_S=<seconds> set, a wait longer than that prints
 * every unfinished launch's device state to stderr and returns ACCEL_ESTATE. */
int accel_sync(accel_ctx *ctx, uint64_t request_id);
/* Record the time origin for accel_req_stats.arrival_ms / done_ms on every
 * tenant stream (call between mixes, when idle). */
int accel_epoch(accel_ctx *ctx);

typedef struct {
  uint64_t first_start_ns;   /* device %globaltimer: first CTA of first launch  */
  uint64_t last_end_ns;      /* device %globaltimer: last CTA of last launch    */
  float elapsed_ms;          /* T(s): arrival event -> done event              */
  float arrival_ms;          /* arrival event relative to the epoch            */
  float done_ms;             /* done event relative to the epoch               */
  uint32_t vgs_total;        /* virtual groups over all launches (static grid) */
  uint32_t launches;
  uint32_t quota_initial;    /* persistent CTAs of the main step at launch     */
  uint32_t quota_min, quota_max;
  uint32_t resolves;         /* quota changes after launch (RESOLVE policy)    */
  uint32_t max_ctas;         /* most CTAs that ever dequeued in one launch     */
  int32_t coverage_ok;       /* 1 / 0; -1 when verify is off                   */
  int32_t mode;
} accel_req_stats;
/* Stats of a completed request (ACCEL_ENOTREADY otherwise). */
int accel_stats(accel_ctx *ctx, uint64_t request_id, accel_req_stats *out);
/* Per-launch device durations (ms) of a completed request submitted with
 * ACCEL_REQ_LAUNCH_EVENTS, measured with CUDA events on the tenant stream:
 * ms_out[i] for launch i (steps in order, repeats in order), n = capacity;
 * *n_out = number of launches written. */
int accel_launch_times(accel_ctx *ctx, uint64_t request_id, float *ms_out, uint32_t n, uint32_t *n_out);

/* Per-launch device record of a completed request (from its Virtual NDRange
 * descriptor): %globaltimer of the first CTA start / last CTA end, CTAs that
 * got work, the admission high-water mark, the (dynamic) VG total, and whether
 * a RESOLVE top-up joined.  out[n]; *n_out = launches written. */
typedef struct {
  uint64_t t_first_ns, t_last_ns;
  uint32_t ctas_started, max_alive, total, topped;
} accel_launch_stat;
int accel_launch_stats(accel_ctx *ctx, uint64_t request_id, accel_launch_stat *out, uint32_t n,
                       uint32_t *n_out);
/* Per-VG execution trace of a completed request submitted with
 * ACCEL_REQ_TRACE (the tracing subsystem): record k of launch l
 * of a step is at index (sum of the earlier launches' static VG totals) + k --
 * the coverage layout.  t_start/t_end: %globaltimer around the body, sm =
 * %smid, cta = the CTA (blockIdx.x of the persistent or top-up grid, linear
 * block index of the native grid; top-up CTAs have bit 31 set).  VGs that did
 * not run (bfs past the frontier) keep t_start_ns == 0.  n = capacity in
 * records; *n_out = records of the request. */
typedef struct {
  uint64_t t_start_ns, t_end_ns;
  uint32_t sm, cta;
} accel_vg_record;
int accel_vg_trace(accel_ctx *ctx, uint64_t request_id, accel_vg_record *out, uint64_t n, uint64_t *n_out);
/* The dequeue order the library uses for a step of `kernel_id` over `grid`
 * with `args` (accel_launch.order_device == NULL): VG ids by decreasing
 * T::vg_cost, ties by increasing id (DESIGN.md R-disp-7), written to
 * order_device[G] (DEVICE, caller-owned).  Synchronous.  ACCEL_EINVAL if the
 * kernel has no cost model or G > 8192. */
int accel_dequeue_order(accel_ctx *ctx, int32_t kernel_id, const accel_dim3 *grid, const void *args,
                        uint32_t args_size, uint32_t *order_device);
/* Forget completed requests (frees their descriptors); ACCEL_ALL = all done. */
int accel_release(accel_ctx *ctx, uint64_t request_id);
/* Streams of a tenant (cudaStream_t as void*), for interop (torch.cuda.ExternalStream). */
int accel_tenant_stream(accel_ctx *ctx, int32_t tenant, void **main_stream, void **topup_stream);

/* ---- pure host functions (no GPU needed) ---------------------------------- */
typedef struct { uint32_t thr, regs, smem, cta, grid_vgs, weight; } accel_demand;
/* Per-CTA demand vector of a kernel (SURVEY §8 a1 / DESIGN.md R-solver-2). */
int accel_demand_of(const accel_caps *caps, uint32_t block_threads, uint32_t regs_per_thread,
                    uint32_t smem_bytes, uint32_t grid_vgs, uint32_t weight, accel_demand *out);
/* The share solver of PAPER.md §3 (closed form + per-SM feasibility + greedy),
 * k requests in arrival order -> quota_out[k]. */
int accel_solve(const accel_caps *caps, const accel_demand *d, int32_t k, uint32_t *quota_out);
/* Placement order of k requests (DESIGN.md R-place-1): order_out[k] = request
 * indices, largest per-CTA footprint (max over threads, registers, shared
 * memory, CTA slots of the share of ONE SM) first, ties in arrival order.
 * SHARED mode enqueues a group's grids in this order and the solver's
 * feasibility model F places them in it.  ACCEL_ENOFIT for an invalid demand. */
int accel_placement_order(const accel_caps *caps, const accel_demand *d, int32_t k, int32_t *order_out);
typedef struct {
  double unfairness;  /* max IS / min IS */
  double stp;         /* sum T(a)/T(s)                              */
  double antt;        /* mean T(s)/T(a)                             */
  double is_max, is_min;
} accel_mix_metrics;
/* Sharing metrics of one mix from isolated times ta[k] and shared times ts[k]. */
int accel_metrics(const double *ta, const double *ts, int32_t k, accel_mix_metrics *out);
/* Weighted sharing (DESIGN.md R-metric-5; "changing
 * the sharing ratio"): weighted slowdown WS_i = (ts_i / ta_i) * w_i / mean(w)
 * -- equal for every request when the sharing honours the ratios w -- and the
 * weighted unfairness max WS / min WS (= unfairness for equal weights).
 * ws_out[k] may be NULL. */
int accel_metrics_weighted(const double *ta, const double *ts, const double *w, int32_t k, double *wunfairness,
                           double *ws_out);
/* Profile-guided sharing ratios (DESIGN.md R-solver-11; PAPER.md lines
 * 388-393 "changing the sharing ratio"): k requests, each with its isolated
 * time ms[i*nf + j] when given the device fraction fracs[j] (fracs[0] = 1,
 * strictly decreasing, > 0; scripts/share_profile.py measures them).  Writes
 * the integer ratios w_out[k] (1..scale) that equalise the predicted slowdowns
 * T_i(f_i)/T_i(1) under sum f_i = 1, and (if s_pred != NULL) the predicted
 * slowdown of each request.  Pass w_out as accel_request.weight.  Pure host
 * function.  ACCEL_EINVAL for invalid profiles. */
int accel_guided_weights(int32_t k, int32_t nf, const double *fracs, const double *ms, uint32_t scale,
                         uint32_t *w_out, double *s_pred);
/* Encode a 2-D TMA tensor map (CUtensorMap, 128 B written to out128) for a
 * row-major fp32 matrix: `inner` elements per row (contiguous), `outer` rows,
 * rows row_stride_bytes apart (multiple of 16), box box_inner x box_outer,
 * swizzle 0/32/64/128 (bytes).  Host only (uses the driver through the
 * runtime; needs a driver, not a GPU context).  The tenant kernel reads the
 * map from device memory the caller copies it to (64-B aligned). */
int accel_tma_map_2d(void *out128, const void *gaddr, uint64_t inner, uint64_t outer,
                     uint64_t row_stride_bytes, uint32_t box_inner, uint32_t box_outer, int32_t swizzle);

/* Encode a 3-D TMA tensor map (CUtensorMap) for a dense fp32 volume
 * [d2][d1][d0] (d0 contiguous): row stride d0*4 and plane stride d0*d1*4
 * bytes (both multiples of 16), box box0 x box1 x box2, no swizzle; boxes
 * partly outside the volume read zeros.  Host only, like accel_tma_map_2d. */
int accel_tma_map_3d(void *out128, const void *gaddr, uint64_t d0, uint64_t d1, uint64_t d2, uint32_t box0,
                     uint32_t box1, uint32_t box2);

/* Kernel execution overlap O = T(c)/T(t) of k
 * intervals [start[i], end[i]). */
int accel_overlap(const double *start, const double *end, int32_t k, double *out);

#ifdef __cplusplus
}
#endif
#endif /* ACCEL_H_ */
