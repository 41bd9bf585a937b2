// dispatch.cuh -- device side of accelOS software work-group scheduling on sm_100a.
//
// PAPER.md §2.4 (lines 439-459) and Fig. 8b (lines 748-781): the original
// work-groups of a kernel execution become virtual groups (VGs) in a Virtual
// NDRange in device memory; a reduced set of physical work-groups runs a loop
// in which a master work-item dequeues VG(s) atomically, the group
// synchronises, leaves on RUN_TERMINATE, else runs the kernel body for every
// VG in [wg_base, wg_end).  §6.2 steps 1-3 (lines 719-724): the kernel becomes
// a plain function whose work-item built-ins (get_group_id ...) read the
// virtual id.  §6.4 (lines 824-834): one dequeue may take several VGs.
//
// B200 design: the JIT transformation of §6 is replaced
// by a compile-time C++ template.  A tenant is a struct T with
//     using Args = <plain C struct>;  static constexpr int kThreads, kChunk;
//     static constexpr uint32_t kDynSmem;
//     static __device__ void body(const Args&, const VirtualBlock&, char* smem);
// optionally  static constexpr bool kDynamicTotal = true;
//             static __device__ uint32_t dynamic_total(const Args&, uint32_t launch_idx);
//             static constexpr int kMinBlocks (same __launch_bounds__ both modes)
// The body never reads blockIdx/gridDim (the `mop` test catches that), keeps
// no state across VGs and never waits on another CTA.
//   accel_persistent<T>: the reduced-grid scheduling kernel (Fig. 8b dyn_sched).
//   accel_topup<T>:      RESOLVE growth grids: sticky grids that follow a
//                        step's launches.
//   accel_native<T>:     the same body on the original grid (Fig. 1a baseline).
//
// RESOLVE policy (BASELINE.json north star; not in the paper, whose kernels
// stay "bound to the resources initially allocated", lines 469-475): the
// request's live quota lives in a device control word.  Admission is
// count-based: a CTA works on a launch only while that launch's `alive` count
// is <= live, so shrinking takes effect at the next dequeue of every CTA
// (a VG boundary).  `alive` shares one 64-bit word with the queue head, so
// admission and the first dequeue are ONE atomic (and every dequeue returns a
// fresh alive count for free).  Growing adds CTAs -- sticky top-up grids launched by the
// host monitor on the tenant's second stream, which serve the current launch
// and then follow the request's later launches.
//
// Completion accounting (who waits for whom).  Launch l+1's main grid follows
// launch l's main grid in stream order (griddepcontrol.wait / the kernel
// boundary), and so does whatever follows the request's LAST main grid, whose
// CTAs retire only after that launch's top-ups (kCfgLast: the request's join).
// So the main grids only need launch l's
// TOP-UP CTAs to be done: a top-up CTA counts itself in `tu_alive` before it
// joins a launch and leaves it with a release fence + decrement
// (wait_topups).  A top-up CTA is in no stream order with the main grids:
// before it serves launch l+1 it needs launch l complete (wait_hybrid).  Once
// the monitor grows a request it sets ctl->grown (with the live quota, before
// the first top-up grid); a main CTA that saw `grown` at its last dequeue
// retires with a release fence and the `alive` decrement, so such a launch
// completes as soon as its last CTA leaves (alive == 0).  A request that was
// never grown -- always, alone -- retires its main CTAs with no fence and no
// atomic.  For the launch that was running when the request grew, whose main
// CTAs may not account, a top-up falls back to waiting until launch l+1's
// main grid has STARTED (ctl->cur, a release by the CTA holding l+1's first
// ticket after its griddepcontrol.wait: l's main grid is then complete) and
// l's top-ups are done; that wait needs a free slot for l+1's CTA 0, so it is
// bounded (kGiveUpNs) and a top-up that gives up leaves the request (always
// safe: top-up CTAs are optional capacity).  An early main grid (R-place-3,
// launched ahead on a side stream) waits for its predecessor's main CTAs too:
// that request's launches carry kCfgAccount (every main CTA accounts).
#pragma once

#include <cstdint>
#include <type_traits>
#include <utility>

#include "accel.h"
#include "../host/internal.h"

namespace accel {

// measurement-only compile-time switches (A/B builds; all 0 in the product)
#ifndef ACCEL_XP_NOTOPPED
#define ACCEL_XP_NOTOPPED 0
#endif
#ifndef ACCEL_XP_NOCUR
#define ACCEL_XP_NOCUR 0
#endif
#ifndef ACCEL_XP_NOCTL
#define ACCEL_XP_NOCTL 0
#endif
#ifndef ACCEL_XP_STRONGCTL
#define ACCEL_XP_STRONGCTL 0
#endif
#ifndef ACCEL_XP_PDL
#define ACCEL_XP_PDL 1   // 0: release at CTA start, 1: at the last chunk, 2: at half the queue
#endif
#ifndef ACCEL_XP_SAMPLECTL
#define ACCEL_XP_SAMPLECTL 0
#endif


// Per-request control block (device memory), two 128-B lines: line 0 is
// read at every admission and dequeue (the live quota), line 1 takes the
// reductions.  Measured: with `cur` on the live quota's line, the per-CTA
// red.max on it queued every CTA's live-quota load behind it in the L2 slice
// (RESOLVE single-tenant overhead 16-21 % -> 10-11 % without it).
struct alignas(128) Ctl {
  // ---- line 0 (live and grown are read together, one 64-bit load)
  uint32_t live;      // live quota (RESOLVE)
  uint32_t grown;     // the monitor has launched a top-up grid for this request
                      // (written with `live`, before the grid): main CTAs account
  uint32_t lost;      // top-up CTAs that gave up waiting for a launch (diagnostic)
  uint32_t pad1[29];
  // ---- line 1
  uint32_t cur;       // highest request-relative launch index started (one red per launch)
  uint32_t pad2[31];
};
static_assert(sizeof(Ctl) == 256, "Ctl layout");

// Virtual NDRange of ONE launch ("Virtual Kernel Execution
// Range which is copied to the accelerator memory").  384 B = three 128-B
// lines so that the three access patterns never share a line (an L2 line that
// takes atomics serialises every other access to it; measured):
//   line 0  read-only during the launch (written by the init kernel) -> L1 hits
//   line 1  the software queue head (one atomicAdd per dequeue)
//   line 2  statistics and RESOLVE admission (reductions, rare atomics)
struct alignas(128) Desc {
  // ---- line 0
  uint32_t total;        // VGs in the original grid (static upper bound)
  uint32_t gx, gy, gz;   // original grid shape (decode, R-disp-2)
  uint32_t chunk;        // VGs per dequeue (§6.4)
  uint32_t launch_idx;   // index of this launch inside its step
  uint32_t flags;        // kFlag*
  uint32_t req_idx;      // launch index inside the request
  Ctl* ctl;              // RESOLVE control block, nullptr otherwise
  uint32_t* coverage;    // verify: coverage[vg] += 1
  uint32_t has_prev;     // this - 1 is the request's previous launch
  uint32_t vg_base;      // sliced step (R-disp-9): first VG of this launch's range
  accel_vg_record* trace;  // ACCEL_REQ_TRACE: trace[vg], nullptr otherwise
  uint32_t governed;       // RESOLVE: this launch belongs to the request's main
                           // step, whose CTA count the live quota governs (the
                           // other steps keep their own solved grid)
  uint32_t slice;          // sliced step: index of this launch's range (0 = first)
  const uint32_t* order;   // dequeue order (ticket t -> VG order[t]), nullptr = linear
  uint32_t pad0[12];
  // ---- line 1: the software queue head (RUN_TERMINATE when >= total) in the
  // low 32 bits, the admitted CTA count (`alive`, RESOLVE) in the high 32
  unsigned long long qa;
  uint32_t pad1[30];
  // ---- line 2
  unsigned long long t_first;  // min %globaltimer over CTA starts
  unsigned long long t_last;   // max %globaltimer over CTA ends
  uint32_t total_seen;   // total as read by the CTAs (dynamic for bfs)
  uint32_t ctas_started; // CTAs admitted with work
  uint32_t tu_alive;     // RESOLVE: top-up CTAs in this launch (wait_topups)
  uint32_t max_alive;    // high-water mark of `alive` (RESOLVE)
  uint32_t topped;       // a top-up CTA joined this launch (RESOLVE)
  uint32_t admit_fail;   // RESOLVE: CTAs admitted over the live quota (ran one chunk, left)
  uint32_t evicted;      // RESOLVE: CTAs that left at a dequeue (shrink)
  uint32_t last_live;    // RESOLVE: live quota seen by the last refused CTA
  uint32_t pad_adm;
  uint32_t draining;     // RESOLVE: evicted CTAs still finishing their last VG
  uint32_t pad2[18];
};
static_assert(sizeof(Desc) == 384, "Desc layout");

// Fire-and-forget reductions (no return value, no round trip).
__device__ __forceinline__ void red_min_u64(unsigned long long* p, unsigned long long v) {
  asm volatile("red.relaxed.gpu.global.min.u64 [%0], %1;" ::"l"(p), "l"(v) : "memory");
}
__device__ __forceinline__ void red_max_u64(unsigned long long* p, unsigned long long v) {
  asm volatile("red.relaxed.gpu.global.max.u64 [%0], %1;" ::"l"(p), "l"(v) : "memory");
}
__device__ __forceinline__ void red_add_u32(uint32_t* p, uint32_t v) {
  asm volatile("red.relaxed.gpu.global.add.u32 [%0], %1;" ::"l"(p), "r"(v) : "memory");
}

enum : uint32_t { kFlagStamps = 1u, kFlagAlive = 2u };

// Desc::qa = alive << 32 | next
constexpr unsigned long long kAlive1 = 1ull << 32;
constexpr unsigned long long kAliveNeg = ~0ull << 32;   // adds -1 to the alive half
__device__ __forceinline__ uint32_t qa_next(unsigned long long v) { return (uint32_t)v; }
__device__ __forceinline__ uint32_t qa_alive(unsigned long long v) { return (uint32_t)(v >> 32); }

// Replacement of the OpenCL work-item built-ins (get_group_id / get_num_groups,
// PAPER.md §6.3): what a body sees instead of blockIdx/gridDim.
struct VirtualBlock {
  uint32_t x, y, z;        // get_group_id(0..2)
  uint32_t gx, gy, gz;     // get_num_groups(0..2)
  uint32_t linear;         // x + gx*(y + gy*z)
  uint32_t launch_idx;     // launch index inside the request step
};

__device__ __forceinline__ unsigned long long globaltimer() {
  unsigned long long t;
  asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(t));
  return t;
}
// A persistent grid lets its successor launch only when its CTAs reach their
// last VG (serve): a successor released at CTA start holds SM slots for the
// whole launch -- waiting in griddepcontrol.wait -- and takes every slot a
// co-runner frees in the meantime (measured: bfs's level grids waited 100-240
// us each for slots behind the stencil's pre-launched sweeps in C2).
__device__ __forceinline__ void pdl_wait() { asm volatile("griddepcontrol.wait;" ::: "memory"); }
__device__ __forceinline__ void pdl_release() { asm volatile("griddepcontrol.launch_dependents;" ::: "memory"); }
__device__ __forceinline__ uint32_t smid() {
  uint32_t v;
  asm volatile("mov.u32 %0, %%smid;" : "=r"(v));
  return v;
}
// ACCEL_REQ_TRACE: one record per VG, written by the master thread.
__device__ __forceinline__ void trace_vg(accel_vg_record* t, uint32_t vg, unsigned long long t0, uint32_t cta) {
  accel_vg_record r;
  r.t_start_ns = t0;
  r.t_end_ns = globaltimer();
  r.sm = smid();
  r.cta = cta;
  t[vg] = r;
}

__device__ __forceinline__ uint32_t ld_relaxed(const uint32_t* p) {
  uint32_t v;
  asm volatile("ld.relaxed.gpu.global.u32 %0, [%1];" : "=r"(v) : "l"(p) : "memory");
  return v;
}

// {live, grown} of a Ctl line 0 in one load (live in the low half).  A weak
// L2 load (.cg: no L1 copy that could go stale), not a strong one: a strong
// load right behind the dequeue atomic measured 0.5 us per stencil launch
// and 1.6 us per lbm launch; a view a few hundred ns old is all the
// protocol needs (shrink at a later dequeue, accounting from `grown`, which
// the host writes before any top-up CTA can run).
__device__ __forceinline__ unsigned long long ld_ctl(const void* p) {
#if ACCEL_XP_STRONGCTL
  unsigned long long v;
  asm volatile("ld.relaxed.gpu.global.u64 %0, [%1];" : "=l"(v) : "l"(p) : "memory");
  return v;
#else
  return __ldcg(reinterpret_cast<const unsigned long long*>(p));
#endif
}

__device__ __forceinline__ uint32_t ld_volatile(const uint32_t* p) {
  uint32_t v;
  asm volatile("ld.volatile.global.u32 %0, [%1];" : "=r"(v) : "l"(p));
  return v;
}
// Release/acquire fence at GPU scope (message passing between CTAs); lighter
// than __threadfence() (fence.sc.gpu).
__device__ __forceinline__ void fence_acq_rel() { asm volatile("fence.acq_rel.gpu;" ::: "memory"); }

__device__ __forceinline__ unsigned long long ld_volatile_u64(const unsigned long long* p) {
  unsigned long long v;
  asm volatile("ld.volatile.global.u64 %0, [%1];" : "=l"(v) : "l"(p));
  return v;
}

// Optional T::kMinBlocks: minimum resident CTAs per SM for __launch_bounds__,
// applied to BOTH instantiations so native and persistent get the same
// register budget (§6.5: the transformation must not
// add register pressure).
template <class T, class = void>
struct min_blocks : std::integral_constant<int, 1> {};
template <class T>
struct min_blocks<T, std::void_t<decltype(T::kMinBlocks)>> : std::integral_constant<int, T::kMinBlocks> {};

// Optional T::kMaxCtasPerSm: the kernel's useful occupancy (accel_kernel_desc
// max_ctas_per_sm); 0 = none.
template <class T, class = void>
struct max_ctas_per_sm : std::integral_constant<uint32_t, 0> {};
template <class T>
struct max_ctas_per_sm<T, std::void_t<decltype(T::kMaxCtasPerSm)>>
    : std::integral_constant<uint32_t, (uint32_t)T::kMaxCtasPerSm> {};

// Optional T::kSlices (R-disp-9): SHARED runs of a single launch are split
// into this many sub-launches over consecutive VG ranges; 0/1 = none.
template <class T, class = void>
struct slices_of : std::integral_constant<uint32_t, 1> {};
template <class T>
struct slices_of<T, std::void_t<decltype(T::kSlices)>> : std::integral_constant<uint32_t, (uint32_t)T::kSlices> {};

template <class T, class = void>
struct has_dynamic_total : std::false_type {};
template <class T>
struct has_dynamic_total<T, std::void_t<decltype(T::kDynamicTotal)>>
    : std::integral_constant<bool, T::kDynamicTotal> {};

// kSpread: the kernel's VG cost varies smoothly in space (cutcp's atom
// density, tpacf's pair blocks).  The CTAs of one SM reach the queue together,
// so linear tickets hand each SM a run of adjacent -- equally heavy -- VGs and
// the heavy runs pile up on a few SMs (issue-bound kernels then run 20 % long).
// Spread kernels map ticket t -> VG t * p mod total (gcd(p, total) = 1,
// p ~ total / golden ratio): consecutive tickets land far apart.
template <class T, class = void>
struct has_spread : std::false_type {};
template <class T>
struct has_spread<T, std::void_t<decltype(T::kSpread)>> : std::integral_constant<bool, T::kSpread> {};

__device__ __forceinline__ uint32_t spread_factor(uint32_t total) {
  if (total <= 2) return 1;
  uint32_t p = (uint32_t)(0.6180339887 * total);
  for (;; ++p) {
    uint32_t a = p, b = total;
    while (b) { const uint32_t r = a % b; a = b; b = r; }
    if (a == 1) return p;
  }
}

template <class T>
__device__ __forceinline__ uint32_t vg_total(const typename T::Args& a, const Desc* d,
                                             uint32_t launch_idx) {
  if constexpr (has_dynamic_total<T>::value) {
    uint32_t t = T::dynamic_total(a, launch_idx);
    return t < d->total ? t : d->total;
  } else {
    return d->total;
  }
}

__device__ __forceinline__ VirtualBlock decode(uint32_t vg, uint32_t gx, uint32_t gy,
                                               uint32_t gz, uint32_t launch_idx) {
  VirtualBlock b;
  b.gx = gx; b.gy = gy; b.gz = gz;
  b.linear = vg;
  b.launch_idx = launch_idx;
  if (gy == 1 && gz == 1) {   // 1-D grids: no division
    b.x = vg; b.y = 0; b.z = 0;
  } else {
    const uint32_t q = vg / gx;
    b.x = vg - q * gx;
    b.y = q % gy;
    b.z = q / gy;
  }
  return b;
}

constexpr uint32_t kTerminate = 0xffffffffu;

// A launch is complete when its queue is exhausted and no CTA is admitted
// (a CTA is admitted before its first dequeue and leaves after its last VG).
// Used only where every CTA of the launch accounts (kCfgAccount requests).
__device__ __forceinline__ void wait_complete(const Desc* p) {
  for (;;) {
    const uint32_t tot = ld_volatile(&p->total_seen);
    const unsigned long long v = ld_volatile_u64(&p->qa);
    if (tot != kTerminate && qa_next(v) >= tot && qa_alive(v) == 0) {
      fence_acq_rel();
      if (ld_volatile(&p->draining) == 0) break;
    }
    __nanosleep(256);
  }
  fence_acq_rel();
  // the launch's results were written through the generic proxy by other CTAs;
  // this CTA may read them with TMA (async proxy)
  asm volatile("fence.proxy.async.global;" ::: "memory");
}

// Top-up CTA: wait until launch p (the predecessor of request launch
// `next_idx`) is complete -- every admitted CTA left (alive == 0: all of p's
// main CTAs accounted), or p's successor main grid has started (p's main grid
// done) and p's own top-ups are done.  False if neither happened within
// kGiveUpNs (the successor's CTA 0 found no slot): the caller leaves.
constexpr unsigned long long kGiveUpNs = 500000;
__device__ __forceinline__ bool wait_hybrid(const Desc* p, uint32_t next_idx) {
  const unsigned long long t0 = globaltimer();
  for (;;) {
    const uint32_t tot = ld_volatile(&p->total_seen);
    const unsigned long long v = ld_volatile_u64(&p->qa);
    if (tot != kTerminate && qa_next(v) >= tot) {
      if (qa_alive(v) == 0) {
        fence_acq_rel();
        if (ld_volatile(&p->draining) == 0) break;
      }
      if (ld_volatile(&p->ctl->cur) >= next_idx) {
        fence_acq_rel();
        if (ld_volatile(&p->tu_alive) == 0 && ld_volatile(&p->draining) == 0) break;
      }
    }
    if (globaltimer() - t0 > kGiveUpNs) return false;
    __nanosleep(256);
  }
  fence_acq_rel();
  asm volatile("fence.proxy.async.global;" ::: "memory");
  return true;
}

// Launch p's main grid is known complete (stream order, or ctl->cur past it):
// wait until its top-up CTAs are done too.  The queue word is read first: a
// top-up that joined before the queue ran dry counted itself in tu_alive
// before its admission atomic (release fence in between), so it is visible
// here; one that joins later gets no VG.
__device__ __forceinline__ void wait_topups(const Desc* p) {
  for (;;) {
    const uint32_t tot = ld_volatile(&p->total_seen);
    const unsigned long long v = ld_volatile_u64(&p->qa);
    if (tot != kTerminate && qa_next(v) >= tot) {
      fence_acq_rel();
      if (ld_volatile(&p->tu_alive) == 0 && ld_volatile(&p->draining) == 0) break;
    }
    __nanosleep(256);
  }
  fence_acq_rel();
  asm volatile("fence.proxy.async.global;" ::: "memory");
}

// Launch configuration word, a kernel parameter (no descriptor load on the
// critical path of a CTA's first dequeue): bits 0-15 chunk, then flags.  The
// policy itself is a template parameter, so the STATIC kernel carries no
// RESOLVE state in its registers.
enum : uint32_t {
  kCfgChunkMask = 0xffffu,
  kCfgResolve = 1u << 16,
  kCfgStamps = 1u << 17,
  kCfgHasPrev = 1u << 18,  // the request ran a launch before this one (RESOLVE
                           // persistent grids check its `topped` word)
  kCfgWaitPrev = 1u << 20,     // wait for the predecessor launch on the device whether or not
                               // it was topped up (R-place-3: this grid was launched ahead
                               // on a side stream, not behind its predecessor)
  kCfgStaticFirst = 1u << 19,  // main grid: CTA b's first chunk is [b*chunk, (b+1)*chunk)
                               // with no atomic (desc_init starts the queue head at
                           // grid*chunk and, under RESOLVE, `alive` at grid)
  kCfgAccount = 1u << 21,  // RESOLVE main grid whose CTAs retire with the fenced `alive`
                           // decrement (a request with an early main grid, R-place-3)
  kCfgTopup = 1u << 22,    // a top-up CTA (accel_topup): always accounts
  kCfgLast = 1u << 23,     // RESOLVE: the request's last launch -- its main CTAs retire only
                           // after the launch's top-ups (the request's join, in stream order)
  kCfgIndep = 1u << 29,    // a later slice of a sliced step: independent of its stream
                           // predecessor (no griddepcontrol.wait, no predecessor check)
  kCfgSliceJoin = 1u << 30, // the last slice: its CTAs retire after every earlier slice
  // measurement-only ablations (env ACCEL_ABLATE on the host; scripts/isolated.py)
  kAblNoFence = 1u << 24,  // retire without the release fence (UNSAFE with top-ups)
  kAblNoLive = 1u << 25,   // never load the live quota (no shrink)
  kAblNoStats = 1u << 26,  // no max_alive reduction at admission
  kAblNoDec = 1u << 27,    // no alive decrement at retire (UNSAFE with top-ups)
  kAblNoTop = 1u << 28     // no predecessor `topped` check (UNSAFE with top-ups)
};

// Scheduling state of one CTA in shared memory (the paper's `local struct SD`,
// Fig. 8b).  Everything the master thread keeps between
// dequeues lives here, not in registers, so the body keeps the register budget
// it has in the native kernel: only the buffer parity k lives across the body.
// The VG to run next is double-buffered: thread 0 publishes VG k+1 into
// cur[(k+1)&1] while slower warps may still be loading cur[k&1] (a body
// need not contain a barrier); the barrier closing iteration k orders both.
struct SchedState {
  struct Cur {
    uint32_t vg;         // queue position to run next (sd.wg_base)
    uint32_t id;         // the VG at that position (vg, or spread)
    uint32_t x, y, z;    // its decode, by thread 0 (the warps only load it)
  } cur[2];
  uint32_t end;        // end of the current chunk (sd.wg_end)
  uint32_t total;      // VGs of this launch (RUN_TERMINATE when vg >= total)
  uint32_t gx, gy, gz, launch_idx;
  uint32_t spread;     // 0: linear, else the kSpread factor
  uint32_t chunk;
  uint32_t prefetch_window;
  uint32_t nxt;        // prefetched chunk (valid if have_nxt)
  uint32_t* coverage;
  accel_vg_record* trace;
  const uint32_t* order;   // dequeue order of the launch (nullptr: linear / spread)
  Ctl* ctl;                // RESOLVE: the request's control block (d->ctl)
  uint32_t vg_base;        // sliced step: first VG of this launch's range
  uint32_t governed;       // RESOLVE: the live quota governs this launch
  unsigned long long t0;   // trace: start of the current VG
  // RESOLVE, thread 0: view of the live quota and the admitted count, loaded
  // right after each dequeue and used at the next one, so the check adds no
  // latency in front of the queue atomic
  uint8_t have_nxt, admitted, draining;
  uint8_t released;    // griddepcontrol.launch_dependents issued
  uint8_t ndq;         // RESOLVE: dequeues so far (ACCEL_XP_SAMPLECTL)
  // RESOLVE: read the control line at this dequeue?  Always in the product;
  // ACCEL_XP_SAMPLECTL (measurement): every 4th dequeue, every dequeue of a
  // CTA whose VGs run long, and every dequeue in the launch's last two waves.
  __device__ __forceinline__ bool ctl_due() {
#if ACCEL_XP_SAMPLECTL
    return long_vg || (ndq++ & 3u) == 0u || total - end <= 2u * chunk * gridDim.x;
#else
    return true;
#endif
  }
  uint8_t over;        // RESOLVE: admitted over the live quota -> leave at the next dequeue
  uint8_t long_vg;     // the last VG ran longer than kLongVgNs
  template <bool kSpread>
  __device__ __forceinline__ void set_cur(uint32_t k, uint32_t vg) {
    cur[k].vg = vg;
    if (vg < total) {
      // ticket vg of this launch's range -> VG (vg_base: the range of a slice)
      uint32_t id = vg_base + vg;
      if (order != nullptr) {
        id = __ldg(order + vg_base + vg);
      } else if constexpr (kSpread) {
        id = vg_base + (uint32_t)(((uint64_t)vg * spread) % total);
      }
      cur[k].id = id;
      const VirtualBlock b = decode(id, gx, gy, gz, launch_idx);
      cur[k].x = b.x; cur[k].y = b.y; cur[k].z = b.z;
    }
  }
};

// One dequeue (Fig. 8b line 26, rt_sched_wgroup): one 64-bit
// atomicAdd of `chunk` on the queue word, which also returns the admitted
// count.  Under RESOLVE a CTA first leaves if its last view says the launch
// holds more CTAs than the live quota (shrink at a VG boundary; a CAS on the
// alive half so exactly alive - live CTAs leave), or if it was admitted over
// the quota.  A dequeue may be a prefetch issued while the CTA's current VG is
// still running, so an evicted CTA is `draining` (counted by wait_complete)
// until retire(), after that VG's results are written.  Returns the raw queue
// word (kEvicted when the CTA left).
constexpr unsigned long long kEvicted = ~0ull;
// RESOLVE slow path of a dequeue: leave the launch (over-admitted) or try to
// be evicted (alive > live).  Returns true if the CTA left.
// No loops here: a CAS retry loop in this thread-0 branch made the compiler
// treat the tenant body as possibly divergent and drop the uniform datapath
// (stencil RESOLVE: 0 vs 38 uniform compares, +6 % instructions executed;
// ncu source page + cuobjdump), even when moved out of line.
__device__ __forceinline__ bool try_leave(Desc* d, SchedState* S) {
  atomicAdd(&d->draining, 1u);
  fence_acq_rel();   // draining visible before alive drops
  bool left = false;
  if (S->over) {
    atomicAdd(&d->qa, kAliveNeg);
    left = true;
  } else {
    // one CAS attempt (a loop here, even out of line, cost the body its
    // uniform datapath): a CTA that loses the race keeps working and retries
    // at its next dequeue
    const uint32_t live = ld_relaxed(&d->ctl->live);
    const unsigned long long v = ld_volatile_u64(&d->qa);
    if (qa_alive(v) > live) left = atomicCAS(&d->qa, v, v + kAliveNeg) == v;
  }
  if (left) {
    red_add_u32(&d->evicted, 1u);
    S->admitted = 0;
    S->draining = 1;
    return true;
  }
  red_add_u32(&d->draining, 0xffffffffu);   // not evicted after all
  return false;
}

// hint_alive / hint_live: this CTA's view from its previous dequeue (the
// admitted count it returned, the live quota read beside it), in registers.
template <bool kResolve>
__device__ __forceinline__ unsigned long long dequeue(Desc* d, SchedState* S, uint32_t hint_alive,
                                                      uint32_t hint_live) {
  if (kResolve && (S->over || hint_alive > hint_live) && try_leave(d, S))
    return kEvicted;
  return atomicAdd(&d->qa, (unsigned long long)S->chunk);
}

// ctl_view: {live, grown} as read beside this CTA's last dequeue (~0 if it
// never dequeued: it then accounts, conservatively)
template <bool kResolve>
__device__ __forceinline__ void retire(Desc* d, uint32_t cfg, const SchedState* S, unsigned long long ctl_view) {
  if (kResolve) {
    // a main-grid CTA that ran until the queue was dry retires silently: its
    // results reach its waiters through stream order (see the header); once
    // the request was grown, it accounts for the top-ups' sake
    const bool grown = (ctl_view >> 32) != 0u;
    if (S->admitted && ((cfg & (kCfgAccount | kCfgTopup)) || grown)) {
      if (!(cfg & kAblNoFence)) fence_acq_rel();  // this CTA's VG results before the alive decrement
      if (!(cfg & kAblNoDec)) atomicAdd(&d->qa, kAliveNeg);
    }
    if (S->draining) {
      fence_acq_rel();  // the last VG's results before the draining decrement
      atomicSub(&d->draining, 1u);
    }
    if (cfg & kCfgTopup) {
      fence_acq_rel();
      atomicSub(&d->tu_alive, 1u);
    } else if (cfg & kCfgLast) {
      // the request's join: its last main grid completes only after any
      // top-up CTAs of that launch (what follows on the tenant stream -- copies
      // back, the next request -- sees their results).  A top-up that joins
      // after this check finds the queue dry and writes nothing.
      fence_acq_rel();
      if (ld_volatile(&d->topped)) wait_topups(d);
    }
  } else if (cfg & kCfgAccount) {   // STATIC, sliced step: every main CTA accounts
    fence_acq_rel();
    atomicAdd(&d->qa, kAliveNeg);
  }
  if (cfg & kCfgSliceJoin) {
    // the last slice completes only after every earlier slice of its step:
    // they run without a stream dependence (kCfgIndep), and what follows the
    // step on the stream waits only for this grid.  Their CTAs have all
    // started (each slice's successor launches once all of them released it),
    // so this waits on resident CTAs only.
    const uint32_t n = d->slice;
    for (uint32_t j = 1; j <= n; ++j) wait_complete(d - j);
  }
  if (cfg & kCfgStamps) red_max_u64(&d->t_last, globaltimer());
}

constexpr unsigned long long kLongVgNs = 40000;   // 40 us: ~20 queue round trips

// Serve one launch: admission, dequeue loop, retire.  All threads call it.
template <class T, bool kResolve>
__device__ __forceinline__ void serve(const typename T::Args& args, Desc* d, char* smem,
                                      SchedState* S, uint32_t cfg, uint32_t cta_tag) {
  if (threadIdx.x == 0) {    // master work-item: environment init (rt_env_init)
    const uint32_t chunk = cfg & kCfgChunkMask;
    uint32_t b;
    S->admitted = 1;
    S->draining = 0;
    S->over = 0;
    S->released = 0;
    S->ndq = 0;
    // Static first chunk (main grids): measured, the first dequeue of 740
    // CTAs on one queue word serialised in L2 and spread the CTAs' first VG
    // starts over 6 us of a 30-us stencil launch (scripts/vg_trace.py)
    const bool stat = (cfg & kCfgStaticFirst) != 0u;
    uint32_t topped_prev = 0;
    if (!kResolve) {
      b = stat ? blockIdx.x * chunk : qa_next(atomicAdd(&d->qa, (unsigned long long)chunk));
    } else {
      // a predecessor launch that was topped up may still be running on its
      // top-up CTAs: this grid's body must wait for it.  The flag load, the
      // admission, the first dequeue and the scheduling-state set-up are all
      // issued before the flag is tested, so a launch that was never topped
      // pays no serial round trip for it
      topped_prev =
          (cfg & kCfgWaitPrev) ? 1u
          : ((cfg & kCfgHasPrev) && !(cfg & kAblNoTop) && !ACCEL_XP_NOTOPPED) ? ld_volatile(&(d - 1)->topped) : 0u;
      // admission and first dequeue in one atomic; an arrival over the live
      // quota runs the chunk it got and leaves at its next dequeue
      // (a static-first CTA reads the live quota after its first dynamic
      // dequeue: a shrink that precedes the launch evicts one chunk later,
      // and the launch start carries no load of the control line)
      const uint32_t live = (d->governed && !stat && !(cfg & kAblNoLive)) ? ld_relaxed(&d->ctl->live) : 0xffffffffu;
      uint32_t a;
      if (stat) {
        // admitted from the start (alive = grid); a shrink that came first
        // evicts at the next dequeue
        b = blockIdx.x * chunk;
        a = gridDim.x;
        // CTA 0 holds the launch's first ticket: it announces the launch to
        // top-up grids, a release after griddepcontrol.wait (the previous
        // launch's main grid is complete and its results visible to whoever
        // acquires this).  Issued before this thread's first store or
        // reduction, so the release waits for nothing outstanding
        if (blockIdx.x == 0 && !ACCEL_XP_NOCUR)
          asm volatile("red.release.gpu.global.max.u32 [%0], %1;" ::"l"(&d->ctl->cur), "r"(d->req_idx) : "memory");
        if (blockIdx.x == 0 && !(cfg & kAblNoStats))
          asm volatile("red.relaxed.gpu.global.max.u32 [%0], %1;" ::"l"(&d->max_alive), "r"(a) : "memory");
      } else {
        const unsigned long long v = atomicAdd(&d->qa, kAlive1 | chunk);
        b = qa_next(v);
        a = qa_alive(v) + 1u;
        if (!(cfg & kAblNoStats))
          asm volatile("red.relaxed.gpu.global.max.u32 [%0], %1;" ::"l"(&d->max_alive), "r"(a) : "memory");
        if (a > live) {
          S->over = 1;
          red_add_u32(&d->admit_fail, 1u);
          d->last_live = live;
        }
      }
      // (a queue-admitted CTA never holds ticket 0 under static first chunks;
      // without them the CTA that does announces the launch, as above)
      if (!stat && b == 0)
        asm volatile("red.release.gpu.global.max.u32 [%0], %1;" ::"l"(&d->ctl->cur), "r"(d->req_idx) : "memory");
    }
    const uint32_t launch_idx = d->launch_idx;
    // a dynamic total is the predecessor's output: read it after the wait
    auto wait_prev = [&] {
      if (cfg & kCfgWaitPrev) wait_complete(d - 1);   // not in stream order with it
      else wait_topups(d - 1);                         // its main grid completed
    };
    if constexpr (has_dynamic_total<T>::value) {
      if (topped_prev) {
        wait_prev();
        topped_prev = 0;
      }
    }
    const uint32_t total = vg_total<T>(args, d, launch_idx);
    // Publish the total.  A static total: CTA 0 of either grid (the waiters
    // of wait_topups follow the main grid, so its CTA 0 has run).  A dynamic
    // total under RESOLVE: every CTA (the same value: it is final once the
    // predecessor launch completed; an early grid's waiter must not depend on
    // one particular CTA)
    if ((kResolve && has_dynamic_total<T>::value) || blockIdx.x == 0) d->total_seen = total;
    S->chunk = chunk;
    S->have_nxt = 0;
    S->long_vg = 0;
    if (b < total) red_add_u32(&d->ctas_started, 1u);
    S->end = b < total ? min(b + chunk, total) : b;
    S->total = total;
    S->gx = d->gx;
    S->gy = d->gy;
    S->gz = d->gz;
    S->launch_idx = launch_idx;
    S->coverage = d->coverage;
    S->trace = d->trace;
    S->order = d->order;
    S->vg_base = d->vg_base;
    // descriptor fields the dequeue loop needs, kept in shared memory: a
    // descriptor load there is an L1 miss (and an L2 round trip in front of
    // the dequeue atomic) whenever the tenant's body evicted the line --
    // measured ~0.8 us per stencil launch under RESOLVE
    if (kResolve) {
      S->ctl = d->ctl;
      S->governed = d->governed && !(cfg & kAblNoLive);
    }
    S->spread = has_spread<T>::value ? spread_factor(total) : 0u;
    S->prefetch_window = 2u * chunk * gridDim.x;
    S->template set_cur<has_spread<T>::value>(0, b);
    if (topped_prev) wait_prev();
    if (cfg & kCfgStamps) red_min_u64(&d->t_first, globaltimer());
  }
  __syncthreads();
  // thread 0: the prefetched queue word and live quota stay in registers
  // across the body (a shared-memory store would wait for the atomic)
  // thread 0's view for the RESOLVE checks: the last queue word and control
  // line {live, grown} (~0 until read: live = max, grown = conservative)
  unsigned long long r_v = 0, r_ctl = ~0ull;
  // RESOLVE hints from the previous dequeue (evaluated before r_v / r_ctl are
  // overwritten; the live quota governs the request's main step only)
  auto hints = [&](uint32_t* ha, uint32_t* hl) {
    *ha = qa_alive(r_v);
    *hl = S->governed ? (uint32_t)r_ctl : 0xffffffffu;
  };
  for (uint32_t k = 0;; k ^= 1u) {
    const SchedState::Cur c = S->cur[k];
    if (c.vg >= S->total) break;                 // RUN_TERMINATE
    if (threadIdx.x == 0) {
      if (!S->have_nxt && (!S->long_vg || S->total - S->end > S->prefetch_window)) {
        // prefetch the next chunk id once per chunk, early (hidden behind the
        // body).  A prefetched id is a reservation: in the last waves,
        // reservations held by busy CTAs leave finished CTAs (whole SMs) idle
        // for up to one VG duration.  So kernels whose VGs run long (where
        // that idle time dwarfs one queue round trip) dequeue just in time
        // once fewer than two waves of VGs remain
        // the control line ({live, grown}) is read beside every dequeue
        uint32_t ha = 0, hl = 0xffffffffu;
        if (kResolve) hints(&ha, &hl);
        if (kResolve && !ACCEL_XP_NOCTL && S->ctl_due()) r_ctl = ld_ctl(&S->ctl->live);
        r_v = dequeue<kResolve>(d, S, ha, hl);
        S->have_nxt = 1;
      }
      S->t0 = globaltimer();
    }
    VirtualBlock vb;
    vb.x = c.x; vb.y = c.y; vb.z = c.z;
    vb.gx = S->gx; vb.gy = S->gy; vb.gz = S->gz;
    vb.linear = c.id;
    vb.launch_idx = S->launch_idx;
    T::body(args, vb, smem);
    if (threadIdx.x == 0) {
      const uint32_t vg = S->cur[k].vg, id = S->cur[k].id;
      if (S->coverage != nullptr) atomicAdd(&S->coverage[id], 1u);
      if (S->trace != nullptr) trace_vg(S->trace, id, S->t0, cta_tag);
      S->long_vg = globaltimer() - S->t0 > kLongVgNs;
      if (vg + 1 < S->end) {
        S->template set_cur<has_spread<T>::value>(k ^ 1u, vg + 1);
      } else {                                   // publish the prefetched chunk
        if (!S->have_nxt) {                      // tail: just in time
          uint32_t ha = 0, hl = 0xffffffffu;
          if (kResolve) hints(&ha, &hl);
          if (kResolve && !ACCEL_XP_NOCTL && S->ctl_due()) r_ctl = ld_ctl(&S->ctl->live);
          r_v = dequeue<kResolve>(d, S, ha, hl);
        }
        const uint32_t nxt = r_v != kEvicted ? qa_next(r_v) : kTerminate;
        S->end = nxt < S->total ? min(nxt + S->chunk, S->total) : nxt;
        // this CTA's last chunk (the queue will be dry at its next dequeue,
        // or is already): let the request's next launch be scheduled
        if (ACCEL_XP_PDL != 0 && !S->released &&
            (nxt >= S->total ||
             (ACCEL_XP_PDL == 1 ? S->total - nxt <= S->chunk * gridDim.x : 2u * nxt >= S->total))) {
          pdl_release();
          S->released = 1;
        }
        S->template set_cur<has_spread<T>::value>(k ^ 1u, nxt);
        S->have_nxt = 0;
      }
    }
    __syncthreads();
  }
  if (threadIdx.x == 0) retire<kResolve>(d, cfg, S, r_ctl);
}

// Programmatic dependent launch (sm_90+): a request's launch l+1 is launched
// with programmatic stream serialization after launch l (runtime.cpp).  Every
// CTA lets the next grid launch as soon as it has started (once ALL CTAs of
// this grid are resident, the next grid's CTAs may take the SM slots its
// retiring CTAs free), then waits until the previous grid completed and its
// writes are visible -- before it reads anything the previous launch wrote.
// Launched without the attribute, both instructions are no-ops.
__device__ __forceinline__ void pdl_enter() {
  asm volatile("griddepcontrol.launch_dependents;" ::: "memory");
  asm volatile("griddepcontrol.wait;" ::: "memory");
}


// -------------------------------------------------------------------------
// The scheduling kernel: grid = quota (1-D), block = the original block;
// serves launch d.  cfg = chunk | kCfg* flags.  kResolve = RESOLVE policy.
template <class T, bool kResolve>
__global__ void __launch_bounds__(T::kThreads, min_blocks<T>::value)
    accel_persistent(const __grid_constant__ typename T::Args args, Desc* __restrict__ d, uint32_t cfg) {
  extern __shared__ __align__(128) char smem[];
  __shared__ SchedState S;
#if ACCEL_XP_PDL == 0
  pdl_release();
#endif
  if (!(cfg & kCfgIndep)) pdl_wait();   // a later slice depends on nothing before it
  serve<T, kResolve>(args, d, smem, &S, cfg, blockIdx.x);
}

// RESOLVE top-up grid: d = first launch of the request step, `sticky` =
// launches in the step; starts at the request's current launch and follows
// the step's later launches (each only once its predecessor completed).
template <class T>
__global__ void __launch_bounds__(T::kThreads, min_blocks<T>::value)
    accel_topup(const __grid_constant__ typename T::Args args, Desc* __restrict__ d, uint32_t sticky_word) {
  extern __shared__ __align__(128) char smem[];
  __shared__ SchedState S;
  __shared__ uint32_t s_l, s_go;
  // kStickyMain: this grid IS the request's main step (ACCEL_STICKY_MAIN,
  // experiment): one long-lived grid serves every launch of the step, so its
  // warps age like a single-launch kernel's instead of being the youngest on
  // their SM at every launch
  constexpr uint32_t kStickyMain = 1u << 31;
  const bool main_grid = (sticky_word & kStickyMain) != 0u;
  const uint32_t sticky = sticky_word & ~kStickyMain;
  if (threadIdx.x == 0) {
    const uint32_t cur = ld_volatile(&d->ctl->cur);
    s_l = main_grid ? 0u : (cur > d->req_idx ? cur - d->req_idx : 0u);
  }
  __syncthreads();
  for (uint32_t l = s_l; l < sticky; ++l) {
    Desc* dl = d + l;
    if (threadIdx.x == 0) {
      s_go = 1u;
      // launch l's inputs are complete (or the wait gave up: leave)
      if (dl->has_prev && !wait_hybrid(dl - 1, dl->req_idx)) {
        s_go = 0u;
        red_add_u32(&dl->ctl->lost, 1u);
      } else {
        atomicExch(&dl->topped, 1u);
        atomicAdd(&dl->tu_alive, 1u);   // before the admission atomic (wait_topups)
        fence_acq_rel();
        // the main grid announces the launch it serves (after launch l-1
        // completed, so `cur >= l` still implies that for wait_hybrid)
        if (main_grid)
          asm volatile("red.release.gpu.global.max.u32 [%0], %1;" ::"l"(&dl->ctl->cur), "r"(dl->req_idx) : "memory");
      }
    }
    __syncthreads();
    if (!s_go) return;
    // (the predecessor wait above already ran: no kCfgHasPrev)
    const uint32_t cfg = dl->chunk | kCfgResolve | kCfgTopup | ((dl->flags & kFlagStamps) ? kCfgStamps : 0u);
    serve<T, true>(args, dl, smem, &S, cfg, blockIdx.x | 0x80000000u);
    __syncthreads();
    // a top-up CTA that was evicted (shrink) or admitted over the live quota
    // is surplus: it leaves the request instead of following the later
    // launches (the monitor tops up afresh on a later growth, apply_quota)
    if (S.over || S.draining) return;
  }
  // the main grid completes only after every CTA (its own and growth grids')
  // left the step's last launch: what follows on the stream sees all results
  if (main_grid && threadIdx.x == 0) wait_topups(d + sticky - 1);
}

// ---------------------------------------------------------------------------
// Dequeue order from the tenant's cost model (DESIGN.md R-disp-7).  The
// software queue may hand out VGs in any order; a
// tenant with an optional
//     static __device__ float vg_cost(const Args&, const VirtualBlock&);
// (an estimate of a VG's work, e.g. the atoms a cutcp VG streams) gets its VGs
// dealt most expensive first -- longest-processing-time-first list
// scheduling over the persistent CTAs, so the tail after the queue runs dry
// is short.  One CTA computes every cost and bitonic-sorts the keys
// (~cost << 32 | vg: decreasing cost, ties by increasing id) in shared memory.
template <class T, class = void>
struct has_vg_cost : std::false_type {};
template <class T>
struct has_vg_cost<T, std::void_t<decltype(T::vg_cost(std::declval<const typename T::Args&>(),
                                                      std::declval<const VirtualBlock&>()))>> : std::true_type {};


template <class T>
__global__ void __launch_bounds__(kOrderThreads) accel_lpt_order(const __grid_constant__ typename T::Args args, uint32_t gx,
                                                                  uint32_t gy, uint32_t gz, uint32_t* order) {
  extern __shared__ unsigned long long key[];
  const uint32_t total = gx * gy * gz;
  uint32_t n = 1;
  while (n < total) n <<= 1;
  for (uint32_t v = threadIdx.x; v < n; v += kOrderThreads) {
    unsigned long long k = ~0ull;
    if (v < total) {
      const float c = fmaxf(T::vg_cost(args, decode(v, gx, gy, gz, 0)), 0.f);   // >= 0: bits are monotone
      k = ((unsigned long long)(0xffffffffu - __float_as_uint(c)) << 32) | v;
    }
    key[v] = k;
  }
  __syncthreads();
  for (uint32_t k = 2; k <= n; k <<= 1)
    for (uint32_t j = k >> 1; j > 0; j >>= 1) {
      for (uint32_t i = threadIdx.x; i < n; i += kOrderThreads) {
        const uint32_t l = i ^ j;
        if (l > i) {
          const unsigned long long x = key[i], y = key[l];
          if ((x > y) == ((i & k) == 0)) {
            key[i] = y;
            key[l] = x;
          }
        }
      }
      __syncthreads();
    }
  for (uint32_t v = threadIdx.x; v < total; v += kOrderThreads) order[v] = (uint32_t)key[v];
}

// The original kernel: one CTA per VG, hardware block scheduler (Fig. 1a).
// (Every kernel takes the tenant's Args as a __grid_constant__ parameter: a
// body may hand the address of a field to the TMA unit -- a CUtensorMap in
// the argument struct, as stencil_tma does.)
template <class T>
__global__ void __launch_bounds__(T::kThreads, min_blocks<T>::value)
    accel_native(const __grid_constant__ typename T::Args args, Desc* __restrict__ d, uint32_t /*unused*/) {
  extern __shared__ __align__(128) char smem[];
  pdl_enter();
  const uint32_t flags = d->flags;
  if (threadIdx.x == 0 && (flags & kFlagStamps)) red_min_u64(&d->t_first, globaltimer());
  VirtualBlock vb;
  vb.x = blockIdx.x; vb.y = blockIdx.y; vb.z = blockIdx.z;
  vb.gx = gridDim.x; vb.gy = gridDim.y; vb.gz = gridDim.z;
  vb.linear = blockIdx.x + gridDim.x * (blockIdx.y + gridDim.y * blockIdx.z);
  vb.launch_idx = d->launch_idx;
  bool run = true;
  uint32_t total = d->total;
  if constexpr (has_dynamic_total<T>::value) {
    total = vg_total<T>(args, d, vb.launch_idx);
    run = vb.linear < total;
  }
  if (vb.linear == 0 && threadIdx.x == 0) d->total_seen = total;
  if (run) {
    __shared__ unsigned long long s_t0;   // trace: thread 0's VG start (not a register across the body)
    if (threadIdx.x == 0 && d->trace != nullptr) s_t0 = globaltimer();
    T::body(args, vb, smem);
    if (threadIdx.x == 0) {
      if (d->coverage != nullptr) atomicAdd(&d->coverage[vb.linear], 1u);
      if (d->trace != nullptr) trace_vg(d->trace, vb.linear, s_t0, vb.linear);
    }
  }
  if (threadIdx.x == 0 && (flags & kFlagStamps)) red_max_u64(&d->t_last, globaltimer());
}

}  // namespace accel
