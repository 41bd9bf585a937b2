"""Reference share solver (TEST INFRASTRUCTURE ONLY -- see oracle/__init__.py).

Follows PAPER.md §3 "Accelerator Resource Sharing Control" (lines 483-542)
step by step, in the paper's notation, with the readings listed in DESIGN.md
§Readings (R-solver-*).  Every tie is broken explicitly so that the C++ solver
of the product path must match this module exactly.

Paper, restated (not pasted): K kernels run concurrently.  Kernel i has
work-group size w_i, local memory m_i and register usage r_i per work-group.
With device totals T (threads), L (local memory) and R (registers) the number
of work-groups x_i, y_i, z_i allowed by each resource is T/(K w_i), L/(K m_i),
R/(K r_i) (lines 525-535); the quota is min(x_i, y_i, z_i) (lines 536-537);
because these are Diophantine the result may be conservative, so a greedy
heuristic increments work-groups across the kernels until saturation
(lines 537-542).

Readings:
  R-solver-1  floor() for the garbled fractions of lines 526-535.
  R-solver-2  B200 resources: besides threads, registers and shared memory the
              per-SM CTA-slot limit (32) is a fourth resource; registers are
              allocated per warp in 256-register units and per SM
              sub-partition (SMSP); shared memory per CTA is rounded to 128 B
              after adding 1 KiB reserved (cuda_occupancy.h).
  R-solver-3  The closed form runs on device totals; a per-SM feasibility
              model F (below) then checks that the quotas actually pack.
              F simulates the placement the library causes (R-place-1):
              kernels in placement order (largest per-CTA footprint first,
              ties by arrival), each kernel's CTAs dealt round-robin over the
              SMs, skipping SMs where the CTA does not fit, from a pointer
              that carries over between kernels -- the B200 block scheduler's
              breadth-first fill.  (The first version dealt ceil/floor counts
              on rotating offsets regardless of room: it claimed that 127
              small CTAs occupy 127 SMs and gave a one-CTA-per-SM GEMM 21 SMs.)
  R-solver-4  A quota never exceeds the request's virtual-group count G_i;
              a request with G_i = 0 gets 0.
  R-solver-5  Requests with identical (demand, G, weight) form a class; the
              decrement (when F fails) and the greedy increment act on whole
              classes, so identical kernels always receive identical quotas.
  R-solver-6  Greedy: passes over classes in order of first arrival, +1 CTA
              per member of a class if F still holds; stop after a pass that
              accepted nothing.
  R-solver-7  Weights w (§2.2, "changing the sharing
              ratio") scale each request's share of every total; default 1.
  R-solver-8  A request with several kernels (mri-q, sgemm split + GEMM) is
              represented by its main step; every other step is solved against
              the same active set with its own kernel in the request's place.
"""
from __future__ import annotations

from dataclasses import dataclass, field
from fractions import Fraction
from typing import Sequence


@dataclass(frozen=True)
class Caps:
    """Per-SM limits of the device (B200 defaults, cuda_occupancy.h for sm_100)."""
    sms: int = 148
    thr_per_sm: int = 2048
    regs_per_sm: int = 65536
    smem_per_sm: int = 233472          # 228 KiB, maximum carveout
    ctas_per_sm: int = 32
    smsp_per_sm: int = 4
    max_smem_per_cta: int = 232448    # 227 KiB usable by one CTA (optin)
    smem_reserved: int = 1024         # reserved per CTA
    smem_gran: int = 128
    reg_gran: int = 256
    max_regs_per_thread: int = 255

    @property
    def regs_per_smsp(self) -> int:
        return self.regs_per_sm // self.smsp_per_sm


class NoFit(Exception):
    """A CTA of this kernel fits on no SM (ACCEL_ENOFIT)."""


@dataclass(frozen=True)
class Demand:
    """Per-CTA demand vector d = (thr, regs, smem, cta) plus G and weight."""
    thr: int
    regs: int
    smem: int
    cta: int
    grid_vgs: int
    weight: int = 1

    @property
    def warps(self) -> int:
        return self.thr // 32

    @property
    def rpw(self) -> int:
        return self.regs // self.warps if self.warps else 0

    def key(self):
        return (self.thr, self.regs, self.smem, self.cta, self.grid_vgs, self.weight)


def ceil_div(a: int, b: int) -> int:
    return -(-a // b)


def demand_of(block: int, regs_per_thread: int, smem_bytes: int, grid_vgs: int,
              weight: int = 1, caps: Caps = Caps()) -> Demand:
    """Step 1: a kernel's per-CTA demand vector (R-solver-2).

    warps = ceil(b/32); thr = 32 warps; rpw = ceil(32 rho / 256) * 256;
    regs = rpw * warps; smem = ceil((sigma + 1024)/128) * 128; cta = 1.
    """
    warps = ceil_div(block, 32)
    thr = 32 * warps
    rpw = ceil_div(32 * regs_per_thread, caps.reg_gran) * caps.reg_gran
    regs = rpw * warps
    smem = ceil_div(smem_bytes + caps.smem_reserved, caps.smem_gran) * caps.smem_gran
    if (thr > caps.thr_per_sm or smem_bytes > caps.max_smem_per_cta
            or regs_per_thread > caps.max_regs_per_thread
            or ceil_div(warps, caps.smsp_per_sm) * rpw > caps.regs_per_smsp
            or smem > caps.smem_per_sm):
        raise NoFit((block, regs_per_thread, smem_bytes))
    return Demand(thr, regs, smem, 1, grid_vgs, weight)


def check_demand(d: Demand, caps: Caps = Caps()) -> None:
    if (d.thr <= 0 or d.thr % 32 or d.thr > caps.thr_per_sm or d.cta != 1
            or d.regs % d.warps or d.rpw % caps.reg_gran
            or ceil_div(d.warps, caps.smsp_per_sm) * d.rpw > caps.regs_per_smsp
            or d.smem > caps.smem_per_sm or d.smem <= 0 or d.weight <= 0):
        raise NoFit(d)


def closed_form(ds: Sequence[Demand], caps: Caps = Caps()) -> list[int]:
    """Step 2 (PAPER.md 525-537): n_i = min(x_i, y_i, z_i, slot term, G_i)."""
    S = caps.sms
    active = [d for d in ds if d.grid_vgs > 0]
    W = sum(d.weight for d in active)
    out = []
    for d in ds:
        if d.grid_vgs == 0:
            out.append(0)
            continue
        x = (S * caps.thr_per_sm * d.weight) // (W * d.thr)      # threads
        z = (S * caps.regs_per_sm * d.weight) // (W * d.regs)    # registers
        y = (S * caps.smem_per_sm * d.weight) // (W * d.smem)    # local memory
        c = (S * caps.ctas_per_sm * d.weight) // (W * d.cta)     # CTA slots
        n = min(x, y, z, c, d.grid_vgs)
        out.append(max(n, 1))
    return out


def footprint(d: Demand, caps: Caps = Caps()) -> Fraction:
    """Per-CTA footprint: the largest share of ONE SM's resources a CTA takes."""
    return max(Fraction(d.thr, caps.thr_per_sm), Fraction(d.regs, caps.regs_per_sm),
               Fraction(d.smem, caps.smem_per_sm), Fraction(d.cta, caps.ctas_per_sm))


def placement_order(ds: Sequence[Demand], caps: Caps = Caps()) -> list[int]:
    """R-place-1: request indices, largest per-CTA footprint first, ties in
    arrival order (the order the library enqueues a group's grids in)."""
    return sorted(range(len(ds)), key=lambda i: (-footprint(ds[i], caps), i))


def feasible(ds: Sequence[Demand], n: Sequence[int], caps: Caps = Caps()) -> bool:
    """Step 3: per-SM feasibility F(n) (R-solver-3): the placement below
    exists."""
    return placement(ds, n, caps) is not None


def placement(ds: Sequence[Demand], n: Sequence[int], caps: Caps = Caps()):
    """The per-SM placement model behind F(n) (R-solver-3): returns
    counts[sm][i] = CTAs of request i on SM sm, or None when a CTA fits nowhere.

    Kernels in placement order; kernel i's n_i CTAs are dealt round-robin over
    the SMs from a pointer p (carried over between kernels, starting at SM 0),
    each CTA going to the next SM where it fits: thread, CTA-slot and
    shared-memory sums within the SM's limits, and its warps packed into the
    sub-partitions -- round-robin from the least-loaded SMSP (lowest index on
    ties), no SMSP above regs_per_sm/4.  F fails when a CTA fits on no SM.
    Dealt in rounds: every SM that fits at the start of a round takes one CTA
    (an SM is revisited only after a full cycle), the last round the first
    SMs from p.
    """
    S = caps.sms
    P = caps.smsp_per_sm
    # per-SM state (threads, CTA slots, shared memory, registers per SMSP);
    # SMs in the same state answer alike, so the step is memoised per state
    st = [(0, 0, 0, (0,) * P)] * S
    memo: dict = {}

    def place(state, d: Demand):
        """The SM state after adding one CTA of d, or None if it does not fit."""
        key = (state, d.thr, d.cta, d.smem, d.warps, d.rpw)
        if key in memo:
            return memo[key]
        t, c, m, sp = state
        out = None
        if t + d.thr <= caps.thr_per_sm and c + d.cta <= caps.ctas_per_sm and m + d.smem <= caps.smem_per_sm:
            start = min(range(P), key=lambda s: (sp[s], s))
            nsp = list(sp)
            for w in range(d.warps):
                nsp[(start + w) % P] += d.rpw
            if max(nsp) <= caps.regs_per_smsp:
                out = (t + d.thr, c + d.cta, m + d.smem, tuple(nsp))
        memo[key] = out
        return out

    counts = [[0] * len(ds) for _ in range(S)]
    p = 0
    for i in placement_order(ds, caps):
        d, left = ds[i], n[i]
        while left > 0:
            fit = []
            for j in range(S):
                sm = (p + j) % S
                nxt = place(st[sm], d)
                if nxt is not None:
                    fit.append((sm, nxt))
                    if len(fit) == left:
                        break
            if not fit:
                return None
            for sm, nxt in fit:
                st[sm] = nxt
                counts[sm][i] += 1
            left -= len(fit)
            p = (fit[-1][0] + 1) % S
    return counts


def dominant_share(d: Demand, n: int, caps: Caps = Caps()) -> Fraction:
    """max over resources of n*d_r / (S * cap_r), exact."""
    S = caps.sms
    return max(Fraction(n * d.thr, S * caps.thr_per_sm),
               Fraction(n * d.regs, S * caps.regs_per_sm),
               Fraction(n * d.smem, S * caps.smem_per_sm),
               Fraction(n * d.cta, S * caps.ctas_per_sm))


def classes(ds: Sequence[Demand]) -> list[list[int]]:
    """R-solver-5: request indices grouped by identical key, in first-arrival order."""
    order: list[list[int]] = []
    seen: dict = {}
    for i, d in enumerate(ds):
        k = d.key()
        if k not in seen:
            seen[k] = len(order)
            order.append([])
        order[seen[k]].append(i)
    return order


def solve(ds: Sequence[Demand], caps: Caps = Caps()) -> list[int]:
    """Quota n_i (persistent CTAs) for each active request, in arrival order."""
    for d in ds:
        check_demand(d, caps)
    n = closed_form(ds, caps)
    cls = classes(ds)
    # Step 3: decrement whole classes until F holds.
    while not feasible(ds, n, caps):
        best = None
        for ci, members in enumerate(cls):
            i = members[0]
            if n[i] <= 1:
                continue
            s = dominant_share(ds[i], n[i], caps)
            # ties -> the class whose first member arrived latest
            if best is None or s >= best[0]:
                best = (s, ci)
        if best is None:
            # R-solver-9: even one CTA per request does not pack; keep the
            # 1-CTA quotas (the hardware queues the excess) -- only possible
            # on devices with fewer SMs than concurrent requests.
            break
        for i in cls[best[1]]:
            n[i] -= 1
    # Step 4: class-symmetric greedy fill (R-solver-6).
    while True:
        accepted = False
        for members in cls:
            if any(n[i] + 1 > ds[i].grid_vgs for i in members):
                continue
            for i in members:
                n[i] += 1
            if feasible(ds, n, caps):
                accepted = True
            else:
                for i in members:
                    n[i] -= 1
        if not accepted:
            break
    return n


def step_quota(ds: Sequence[Demand], i: int, step: Demand, caps: Caps = Caps()) -> int:
    """Quota of a secondary kernel of request i (R-solver-8): the same active
    set solved again with request i represented by that step's own kernel."""
    dj = list(ds)
    dj[i] = step
    return solve(dj, caps)[i]
