#!/usr/bin/env python
"""accelOS-on-B200 bench: fair space sharing of one GPU by concurrent tenants.

    python bench.py [--gpus N] [--steps K] [--warmup W] [--config c2] [--impl accel|reference]

One STEP = one mix of tenant kernel-execution requests (BASELINE.json config,
default config 2 = the paper's Fig. 2 mix bfs + cutcp + stencil + tpacf,
PAPER.md lines 289-299) submitted together through the C ABI and run to
completion: solver quotas + persistent dispatch (SHARED mode).  The same mix
is also run in NATIVE mode (standard concurrent streams, Fig. 1a) for the
"vs native streams" comparison, and every tenant alone (NATIVE) for T(a).

Headline metric (BASELINE.json): unfairness (max/min slowdown), STP and ANTT
vs native streams -> reported under "sharing".  `value` is whole-job
throughput in mixes/s (all GPUs), device-timed with CUDA events.

Multi-GPU: one process per GPU -- under torchrun, or self-spawned by
`--gpus N` when WORLD_SIZE is unset.  Every rank runs its own independent mix
on its own GPU (no collective on the data path: PAPER.md has one accelerator
per platform, lines 844-852; BASELINE config 5).  The control plane is gloo on
the host (barrier + gather of per-rank timings; no NCCL); value = all mixes /
max over ranks of the device time.
"""
from __future__ import annotations

import argparse
import json
import math
import os
import statistics
import sys
import threading
import time

os.environ.setdefault("CUDA_DEVICE_MAX_CONNECTIONS", "32")
ROOT = os.path.dirname(os.path.abspath(__file__))
if ROOT not in sys.path:
    sys.path.insert(0, ROOT)

import numpy as np  # noqa: E402

import synth  # noqa: E402

METRIC = "unfairness (max/min slowdown), STP and ANTT vs native streams, 1–8 B200"
UNIT = "mixes/s"

# BASELINE.json configs -> (tenants in arrival order, preset size, seeds)
CONFIGS = {
    "c1": dict(tenants=["stencil", "histo"], size="small", seeds=[1, 2],
               desc="2 tenants on 1 GPU: stencil 64^3 fp32 + histo 256K uint8"),
    "c2": dict(tenants=["bfs", "cutcp", "stencil", "tpacf"], size="default", seeds=[3, 4, 5, 6],
               desc="Paper Fig.2 mix: bfs + cutcp + stencil + tpacf concurrently on 1xB200"),
}
ALL_TENANTS = ["bfs", "cutcp", "stencil", "tpacf", "histo", "spmv", "sgemm", "mriq"]


def c5_mix(rank: int) -> list[str]:
    """BASELINE config 5: an ordered 4-tuple of distinct tenants per GPU, seed 100+g."""
    r = np.random.Generator(np.random.PCG64(100 + rank))
    return [ALL_TENANTS[i] for i in r.permutation(len(ALL_TENANTS))[:4]]


def env_rank():
    return (int(os.environ.get("RANK", 0)), int(os.environ.get("WORLD_SIZE", 1)),
            int(os.environ.get("LOCAL_RANK", 0)))


# ----------------------------------------------------------------- clocks
class ClockSampler:
    """NVML sampling of SM clock and throttle reasons during the timed region."""

    REASONS = {0x1: "gpu_idle", 0x2: "applications_clocks_setting", 0x4: "sw_power_cap",
               0x8: "hw_slowdown", 0x10: "sync_boost", 0x20: "sw_thermal_slowdown",
               0x40: "hw_thermal_slowdown", 0x80: "hw_power_brake_slowdown",
               0x100: "display_clock_setting"}

    def __init__(self, device: int, period: float = 0.1):
        self.device, self.period = device, period
        self.samples: list[int] = []
        self.reasons: set[str] = set()
        self.max_mhz = None
        self._stop = threading.Event()
        self._t = None
        try:
            import pynvml
            pynvml.nvmlInit()
            self.nv = pynvml
            self.h = pynvml.nvmlDeviceGetHandleByIndex(device)
            self.max_mhz = pynvml.nvmlDeviceGetMaxClockInfo(self.h, pynvml.NVML_CLOCK_SM)
        except Exception as e:  # noqa: BLE001
            self.nv = None
            self.err = str(e)

    def _run(self):
        while not self._stop.is_set():
            try:
                self.samples.append(self.nv.nvmlDeviceGetClockInfo(self.h, self.nv.NVML_CLOCK_SM))
                mask = self.nv.nvmlDeviceGetCurrentClocksEventReasons(self.h)
                for bit, name in self.REASONS.items():
                    if mask & bit and name != "gpu_idle":
                        self.reasons.add(name)
            except Exception:  # noqa: BLE001
                pass
            time.sleep(self.period)

    def __enter__(self):
        if self.nv:
            self._t = threading.Thread(target=self._run, daemon=True)
            self._t.start()
        return self

    def __exit__(self, *exc):
        self._stop.set()
        if self._t:
            self._t.join()

    def summary(self):
        if not self.nv:
            return {"sm_mhz": None, "sm_max_mhz": None, "reasons": [], "error": self.err}
        return {"sm_mhz": statistics.median(self.samples) if self.samples else None,
                "sm_max_mhz": self.max_mhz, "reasons": sorted(self.reasons),
                "samples": len(self.samples)}


# ----------------------------------------------------------------- oracle leg
def oracle_sample(name: str, d: dict, budget: float) -> tuple[float, str]:
    """Time the CPU oracle on a bounded sample of one tenant request and
    extrapolate to the whole request.  Returns (seconds for the full request,
    description of the sample)."""
    from oracle import tenants as O
    t0 = time.perf_counter()
    if name == "stencil":
        s = max(1, min(d["sweeps"], int(budget / 0.2) or 1))
        O.stencil(dict(d, sweeps=s))
        dt = time.perf_counter() - t0
        return dt * d["sweeps"] / s, f"stencil {s}/{d['sweeps']} sweeps at full size"
    if name == "histo":
        O.histo(d)
        dt = time.perf_counter() - t0
        return dt * d["iters"], f"histo 1/{d['iters']} iterations"
    if name == "bfs":
        O.bfs(d)
        return time.perf_counter() - t0, "bfs full"
    if name == "cutcp":
        npts = d["nx"] * d["ny"] * d["nz"]
        m = int(min(npts, max(256, budget * 2e8 / max(d["natoms"], 1))))
        r = np.random.Generator(np.random.PCG64(0))
        flat = r.choice(npts, m, replace=False)
        ijk = np.stack([flat % d["nx"], (flat // d["nx"]) % d["ny"], flat // (d["nx"] * d["ny"])], 1)
        t0 = time.perf_counter()
        O.cutcp_points(d, ijk)
        dt = time.perf_counter() - t0
        return dt * npts / m, f"cutcp {m}/{npts} lattice points"
    if name == "tpacf":
        sub = dict(d, nsets=1, rand=np.ascontiguousarray(d["rand"][:1]))
        O.tpacf(sub)
        dt = time.perf_counter() - t0
        # DD once + per set (RR + DR); the sample did DD + 1 set
        return dt * (1 + 3 * d["nsets"]) / 4, f"tpacf DD + 1/{d['nsets']} random sets"
    if name == "spmv":
        O.spmv(d)
        dt = time.perf_counter() - t0
        return dt * d["iters"], f"spmv 1/{d['iters']} iterations"
    if name == "sgemm":
        m = min(d["m"], 64)
        ij = np.stack(np.meshgrid(np.arange(m), np.arange(min(d["n"], 64)), indexing="ij"), -1).reshape(-1, 2)
        t0 = time.perf_counter()
        O.sgemm_entries(d, ij)
        dt = time.perf_counter() - t0
        return dt * d["m"] * d["n"] / len(ij), f"sgemm {len(ij)}/{d['m'] * d['n']} entries"
    if name == "mriq":
        m = min(d["numx"], 2048)
        idx = np.arange(m) * (d["numx"] // m)
        t0 = time.perf_counter()
        O.mriq_points(d, idx)
        dt = time.perf_counter() - t0
        return dt * d["numx"] / m, f"mri-q {m}/{d['numx']} voxels"
    raise KeyError(name)


def cpu_mix_seconds(tenants, inputs, budget_per_tenant):
    tot = 0.0
    desc = []
    for name in tenants:
        s, what = oracle_sample(name, inputs[name], budget_per_tenant)
        tot += s
        desc.append(what)
    return tot, "; ".join(desc)


def make_inputs(cfg_name: str, rank: int, gen: bool = True):
    """(tenants in arrival order, preset size, generated inputs).  Config 5:
    rank g runs its own ordered 4-tuple (seed 100 + g); the others run the
    same mix on every GPU (the weak-scaling run of SURVEY §8(d).1)."""
    if cfg_name == "c5":
        tenants = c5_mix(rank)
        size = "default"
        seeds = [100 + rank + 7 * i for i in range(4)]
    else:
        c = CONFIGS[cfg_name]
        tenants, size, seeds = c["tenants"], c["size"], c["seeds"]
    inputs = {t: synth.preset(t, size, seed=s) for t, s in zip(tenants, seeds)} if gen else None
    return tenants, size, inputs


def run_reference(args):
    """--impl reference: the CPU oracle as it stands (this tier's reference
    arm), on bounded samples of the same workload, on the host cores."""
    rank, world, _ = env_rank()
    if rank != 0:
        return
    tenants, size, inputs = make_inputs(args.config, 0)
    from oracle import tenants as O
    O.build()
    # samples sized so that the timed steps take ~2 minutes in all (larger
    # samples extrapolate better: tiny ones are dominated by thread start-up)
    budget = min(3.0, max(0.3, 120.0 / max(1, args.steps) / len(tenants)))
    for _ in range(args.warmup):
        cpu_mix_seconds(tenants, inputs, 0.3)
    secs = []
    desc = ""
    for _ in range(args.steps):
        s, desc = cpu_mix_seconds(tenants, inputs, budget)
        secs.append(s)
    ms = 1e3 * statistics.mean(secs)
    value = 1e3 / ms
    cores = os.cpu_count()
    line = {"impl": "reference", "metric": METRIC, "value": value, "unit": UNIT, "n_gpus": args.gpus,
            "steps": args.steps, "warmup": args.warmup, "ms_per_step": ms, "higher_is_better": True,
            "scaling": "weak", "vs_baseline": None, "dtype": "f64", "data": "synthetic",
            "config": {"workload": CONFIGS.get(args.config, {}).get("desc", args.config),
                       "tenants": tenants, "size": size},
            "cpu_baseline": {"value": value, "unit": UNIT, "cores": cores, "kind": "oracle",
                             "sample": desc + " (extrapolated to the full requests, run serially "
                                              "with OpenMP on all host cores)"},
            "e2e": {"value": value, "unit": UNIT, "h2d_bytes_per_step": 0, "d2h_bytes_per_step": 0}}
    print(json.dumps(line), flush=True)


def aggregate(allres: list[dict], world: int, steps: int, policy: str) -> dict:
    """Whole-job figures from the per-rank results: device times are the max
    over ranks (the job ends when the slowest GPU ends); value = all mixes
    completed on all GPUs / that time (weak scaling: each GPU runs its own
    mix); sharing metrics are geometric (U) / arithmetic (STP, ANTT) means
    over every rank's steps."""
    gm = lambda xs: math.exp(statistics.mean(math.log(x) for x in xs))  # noqa: E731
    tmax = max(r["dev_ms"] for r in allres)
    emax = max(r["e2e_ms"] for r in allres)
    nmax = max(r["nat_ms"] for r in allres)
    return {
        "tmax": tmax, "emax": emax, "nmax": nmax,
        "value": world * steps / (tmax / 1e3),
        "U_sh": gm([u for r in allres for u in r["sh"]["U"]]),
        "U_na": gm([u for r in allres for u in r["na"]["U"]]),
        "stp_sh": statistics.mean(u for r in allres for u in r["sh"]["STP"]),
        "stp_na": statistics.mean(u for r in allres for u in r["na"]["STP"]),
        "antt_sh": statistics.mean(u for r in allres for u in r["sh"]["ANTT"]),
        "antt_na": statistics.mean(u for r in allres for u in r["na"]["ANTT"]),
        "other": {
            name: {
                "unfairness": gm([u for r in allres for u in r["ot"][name]["U"]]),
                "stp": statistics.mean(u for r in allres for u in r["ot"][name]["STP"]),
                "antt": statistics.mean(u for r in allres for u in r["ot"][name]["ANTT"]),
                "mixes_per_s": world * steps / (max(r["oth_ms"][name] for r in allres) / 1e3),
                "throughput_speedup": nmax / max(r["oth_ms"][name] for r in allres),
            } for name in allres[0]["ot"]
        },
    }


# ----------------------------------------------------------------- host / ranks
def host_cpu() -> dict:
    """The host the oracle ran on: core count and /proc/cpuinfo model."""
    model = None
    try:
        with open("/proc/cpuinfo") as f:
            for ln in f:
                if ln.startswith("model name"):
                    model = ln.split(":", 1)[1].strip()
                    break
    except OSError:
        pass
    threads = int(os.environ.get("OMP_NUM_THREADS", 0)) or os.cpu_count()
    return {"cores": os.cpu_count(), "omp_threads": threads, "model": model}


def cpu_baseline(tenants, inputs) -> dict:
    """The oracle as it stands (never tuned), on a bounded sample of the same
    mix on this host's cores, extrapolated to the whole mix (rank 0 only)."""
    from oracle import tenants as O
    O.build()
    s, desc = cpu_mix_seconds(tenants, inputs, 3.0)
    h = host_cpu()
    return {"value": 1.0 / s, "unit": UNIT, "cores": h["omp_threads"], "kind": "oracle",
            "sample": desc + " (extrapolated to the full requests, run serially with OpenMP "
                             "on all host cores)", "host": h}


def spawn_ranks(args, argv) -> int:
    """--gpus N without torchrun: start N copies of this script, one per GPU,
    with the torchrun environment (RANK, WORLD_SIZE, LOCAL_RANK, MASTER_*)."""
    import socket
    import subprocess
    sk = socket.socket()
    sk.bind(("127.0.0.1", 0))
    port = sk.getsockname()[1]
    sk.close()
    procs = []
    for r in range(args.gpus):
        env = dict(os.environ, RANK=str(r), WORLD_SIZE=str(args.gpus), LOCAL_RANK=str(r),
                   LOCAL_WORLD_SIZE=str(args.gpus), MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
        procs.append(subprocess.Popen([sys.executable, os.path.abspath(__file__), *argv], env=env))
    rcs = [p.wait() for p in procs]
    return max(abs(rc) for rc in rcs)


class Ranks:
    """Control plane of the N-GPU run: gloo on the host (barrier, gather of
    per-rank results).  Nothing of the data path crosses ranks."""

    def __init__(self, rank: int, world: int):
        self.rank, self.world = rank, world
        if world > 1:
            import datetime

            import torch.distributed as dist
            os.environ.setdefault("MASTER_ADDR", "127.0.0.1")
            dist.init_process_group("gloo", rank=rank, world_size=world,
                                    timeout=datetime.timedelta(seconds=1800))
            self.dist = dist

    def barrier(self):
        if self.world > 1:
            self.dist.barrier()

    def gather(self, obj) -> list:
        if self.world == 1:
            return [obj]
        out = [None] * self.world
        self.dist.all_gather_object(out, obj)
        return out

    def close(self):
        if self.world > 1:
            self.dist.destroy_process_group()


def stub_rank(args, rank, world, ranks: Ranks) -> dict:
    """ACCEL_BENCH_STUB=1 (CPU tests of the N-rank plumbing): the per-rank
    result the GPU leg would produce, with fabricated device times, after the
    same barriers."""
    tenants, size, _ = make_inputs(args.config, rank, gen=False)
    ranks.barrier()
    dev_ms = 10.0 * args.steps + rank
    ranks.barrier()
    st = {"U": [1.2 + 0.1 * rank] * args.steps, "STP": [2.5] * args.steps, "ANTT": [1.8] * args.steps,
          "O": [0.9] * args.steps, "makespan_ms": [dev_ms / args.steps] * args.steps,
          "ts_ms": [[1.0] * len(tenants)] * args.steps}
    na = dict(st, U=[4.0] * args.steps, STP=[2.0] * args.steps, ANTT=[2.2] * args.steps)
    return {"rank": rank, "dev_ms": dev_ms, "e2e_ms": dev_ms * 1.5, "nat_ms": 12.0 * args.steps,
            "oth_ms": {"static": 11.0 * args.steps}, "tenants": tenants, "size": size, "sh": st, "na": na,
            "ot": {"static": st}, "quotas": [[1, 1, 1, 0]] * len(tenants), "clk": {"sm_mhz": None},
            "ta": [1.0] * len(tenants), "iso_persist": [1.0] * len(tenants), "roof": {}, "dom": None,
            "h2d": 0, "d2h": 0, "launches_per_step": 0, "parity": {"shared_equals_native": True}}


# ----------------------------------------------------------------- GPU leg
def size_matched_copy(nbytes: float, roof: dict, reps: int = 20) -> dict:
    """Context for an HBM-bound kernel's frac: the bandwidth a plain device
    copy reaches on the SAME bytes per launch (nbytes/2 read + nbytes/2
    written, back to back, CUDA events).  At ~30 us per launch a copy itself
    stays well below the large-copy peak (ramp-up and tail of every launch);
    scripts/stencil_size.py shows the stencil kernel at 0.87 of peak on
    volumes 8x the default.  Outside the timed region; torch's copy kernel is
    the yardstick, not part of the path."""
    import torch
    n = max(1, int(nbytes // 8))
    x = torch.ones(n, dtype=torch.float32, device="cuda")
    y = torch.empty_like(x)
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    for _ in range(3):
        y.copy_(x)
    e0.record()
    for _ in range(reps):
        y.copy_(x)
        x, y = y, x
    e1.record()
    torch.cuda.synchronize()
    gbs = 8.0 * n / (e0.elapsed_time(e1) * 1e-3 / reps) / 1e9
    return {"copy_gbs": gbs, "copy_frac_of_peak": gbs / roof["peak"],
            "frac": roof["achieved"] / gbs, "isolated_frac": roof["isolated"]["achieved"] / gbs}


def run_rank(args, rank, world, local, ranks: Ranks) -> dict:
    """Everything one GPU does: correctness pass, T(a) calibration, the timed
    SHARED steps (barrier + synchronize on both sides), NATIVE and the other
    policies, the end-to-end steps.  Returns the rank's raw results."""
    # a stalled request turns into an error with a device-state dump
    # (accel_sync watchdog) instead of a hung bench
    os.environ.setdefault("ACCEL_SYNC_TIMEOUT_S", "120")
    import torch

    from paper_conf_cgo_margiolaso16_b200 import abi
    from paper_conf_cgo_margiolaso16_b200.jobs import make_job
    from paper_conf_cgo_margiolaso16_b200.runtime import Accel

    torch.cuda.set_device(local)
    tenants, size, inputs = make_inputs(args.config, rank)
    dev = torch.device("cuda", local)
    jobs = [make_job(t, inputs[t], dev) for t in tenants]
    acc = Accel(device=local, mode=abi.MODE_SHARED)
    # bfs: launch levels until the frontier is empty (depth + 1 launches,
    # learned by one untimed probe run)
    for j in jobs:
        if hasattr(j, "fit_levels"):
            j.fit_levels(acc)
    flush_buf = torch.empty(256 * 1024 * 1024 // 4, dtype=torch.float32, device=dev)  # > L2 (126 MB)

    def flush():
        flush_buf.fill_(1.0)
        torch.cuda.synchronize()

    POL = {"resolve": abi.POLICY_RESOLVE, "static": abi.POLICY_STATIC}
    head_pol = POL[args.policy]
    # reported beside the headline: STATIC (the paper's policy) and RESOLVE,
    # and "guided" -- RESOLVE with profile-guided sharing ratios (DESIGN.md
    # R-solver-11) from the committed share profiles, when every tenant has one
    other_pols = [p for p in POL if p != args.policy]
    WEIGHTS = {p: None for p in POL}
    prof_path = os.path.join(ROOT, "profiles", "r2", "share_profile.json")
    if os.path.exists(prof_path):
        prof = json.load(open(prof_path))
        if all(t in prof["profile"] for t in tenants):
            POL["guided"] = abi.POLICY_RESOLVE
            WEIGHTS["guided"] = abi.accel_guided_weights(prof["fracs"],
                                                         [prof["profile"][t]["ms"] for t in tenants])[0]
            other_pols.append("guided")

    def run_group(js, mode, e2e=False, launch_events=False, policy=None, weights=None):
        policy = head_pol if policy is None else policy
        if acc.mode != mode or acc.policy != policy:
            acc.set_mode(mode, policy)
        flush()
        acc.epoch()
        ids = acc.submit(js, e2e=e2e, launch_events=launch_events, weights=weights)
        acc.sync()
        st = [acc.stats(i) for i in ids]
        lt = [acc.launch_times(i, j.launches()) for i, j in zip(ids, js)] if launch_events else None
        acc.release()
        return st, lt

    # -- correctness pass (untimed): coverage of every VG in every mode, and
    # output transparency -- every SHARED policy's outputs bit-identical to
    # the NATIVE run of the same mix (every original
    # work-group runs exactly once with its own id).  Parity against the CPU
    # oracle at these exact sizes is tests/test_gpu_bench_workload.py.
    parity = {}
    with Accel(device=local, mode=abi.MODE_SHARED, verify=True) as vacc:
        ref = None
        for name, mode, pol in [("native", abi.MODE_NATIVE, abi.POLICY_STATIC)] + \
                [(p, abi.MODE_SHARED, POL[p]) for p in (args.policy, *other_pols)]:
            vacc.set_mode(mode, pol)
            st = vacc.run(jobs, weights=WEIGHTS.get(name))
            assert all(s.coverage_ok == 1 for s in st), f"coverage check failed ({name})"
            res = [j.result() for j in jobs]
            if ref is None:
                ref = res
            else:
                ok = all(np.array_equal(a[k], b[k]) for a, b in zip(ref, res) for k in a)
                parity[name] = ok
                assert ok, f"{name} outputs differ from NATIVE"
    del ref

    # -- calibration: T(a) = native isolated (median), persistent isolated
    # (and, when the bench policy is RESOLVE, persistent isolated under
    # STATIC: the paper's own mechanism, without the re-solve bookkeeping)
    iso_native, iso_persist, iso_static, iso_launch = {}, {}, {}, {}
    for j in jobs:
        runs = [(abi.MODE_NATIVE, iso_native, None), (abi.MODE_SHARED, iso_persist, None)]
        if head_pol != abi.POLICY_STATIC:
            runs.append((abi.MODE_SHARED, iso_static, abi.POLICY_STATIC))
        for mode, store, pol in runs:
            ts, lts = [], []
            for _ in range(args.calib_reps):
                st, lt = run_group([j], mode, launch_events=True, policy=pol)
                ts.append(st[0].elapsed_ms)
                lts.append(lt[0])
            store[j.name] = statistics.median(ts)
            if mode == abi.MODE_SHARED and pol is None:
                iso_launch[j.name] = lts
    ta = [iso_native[t] for t in tenants]

    def steps_loop(mode, k, e2e=False, policy=None, weights=None):
        return [run_group(jobs, mode, e2e=e2e, launch_events=True, policy=policy, weights=weights)
                for _ in range(k)]

    steps_loop(abi.MODE_SHARED, args.warmup)
    ranks.barrier()
    torch.cuda.synchronize()
    with ClockSampler(local) as clk:
        shared = steps_loop(abi.MODE_SHARED, args.steps)
    torch.cuda.synchronize()
    ranks.barrier()
    steps_loop(abi.MODE_NATIVE, args.warmup)
    native = steps_loop(abi.MODE_NATIVE, args.steps)
    other = {}
    for p in other_pols:
        steps_loop(abi.MODE_SHARED, 1, policy=POL[p], weights=WEIGHTS[p])
        other[p] = steps_loop(abi.MODE_SHARED, args.steps, policy=POL[p], weights=WEIGHTS[p])
    steps_loop(abi.MODE_SHARED, 1, e2e=True)
    e2e = steps_loop(abi.MODE_SHARED, args.steps, e2e=True)

    def summarize(runs):
        mk, U, STP, ANTT, OV = [], [], [], [], []
        for st, _ in runs:
            mk.append(max(s.done_ms for s in st) - min(s.arrival_ms for s in st))
            ts = [s.elapsed_ms for s in st]
            m = abi.accel_metrics(ta, ts)
            U.append(m.unfairness)
            STP.append(m.stp)
            ANTT.append(m.antt)
            OV.append(abi.accel_overlap([float(s.first_start_ns) for s in st],
                                        [float(s.last_end_ns) for s in st]))
        return {"makespan_ms": mk, "U": U, "STP": STP, "ANTT": ANTT, "O": OV,
                "ts_ms": [[s.elapsed_ms for s in st] for st, _ in runs]}

    sh, na, ee = summarize(shared), summarize(native), summarize(e2e)
    ot = {p: summarize(v) for p, v in other.items()}

    # roofline of the dominant kernel: the tenant with the largest device time
    # in the shared step; per-launch CUDA-event durations on its stream
    works = {j.name: j.work() for j in jobs}
    tot = {t: statistics.mean(ts[i] for ts in sh["ts_ms"]) for i, t in enumerate(tenants)}
    roof = {}
    ppath = os.path.join(ROOT, "MEASURED_PEAKS.json")
    peaks = json.load(open(ppath)) if os.path.exists(ppath) else {"hbm_gbs": 6650.0, "bf16_tflops": 1590.0}
    for i, t in enumerate(tenants):
        w = works[t]
        if "bytes_per_launch" not in w and "bytes" not in w and "flops" not in w:
            continue
        skip = w.get("skip_launches", 0)
        per_launch = [x for _, lt in shared for x in lt[i][skip:]]
        iso = [x for lt in iso_launch[t] for x in lt[skip:]]
        avg = statistics.mean(per_launch)
        avg_iso = statistics.mean(iso)
        if w["bound"] == "hbm":
            b = w.get("bytes_per_launch", w.get("bytes"))
            ach, ach_iso, peak, unit = b / avg / 1e6, b / avg_iso / 1e6, peaks["hbm_gbs"], "GB/s"
        else:
            f = w.get("flops_per_launch", w.get("flops"))
            ach, ach_iso, unit = f / avg / 1e9, f / avg_iso / 1e9, "TFLOP/s"
            peak = w.get("peak_tflops", peaks.get("bf16_tflops"))
        roof[t] = {"bound": w["bound"], "achieved": ach, "peak": peak, "unit": unit, "frac": ach / peak,
                   "traffic": None, "avg_launch_ms": avg,
                   "isolated": {"achieved": ach_iso, "frac": ach_iso / peak, "avg_launch_ms": avg_iso}}
    dom = max(roof, key=lambda t: tot[t]) if roof else None
    # DRAM traffic per launch of the dominant kernel from the committed
    # `ncu --set full` capture (scripts/ncu_traffic.py -> profiles/ncu_traffic.json)
    tpath = os.path.join(ROOT, "profiles", "ncu_traffic.json")
    if dom is not None and os.path.exists(tpath):
        tr = json.load(open(tpath)).get(dom)
        if tr:
            roof[dom]["traffic"] = tr["dram_bytes_per_launch"]
            roof[dom]["traffic_source"] = tr.get("source")
    if dom is not None and roof[dom]["bound"] == "hbm":
        roof[dom]["size_matched_copy"] = size_matched_copy(works[dom].get("bytes_per_launch", works[dom].get("bytes")),
                                                           roof[dom])

    # our kernels per step: descriptor init + every launch (RESOLVE's join is
    # folded into the last launch); growth grids come on top (counted from the
    # requests' stats)
    launches_per_step = sum(1 + j.launches() for j in jobs)
    res = {"rank": rank, "dev_ms": sum(sh["makespan_ms"]), "e2e_ms": sum(ee["makespan_ms"]),
           "nat_ms": sum(na["makespan_ms"]), "oth_ms": {p: sum(v["makespan_ms"]) for p, v in ot.items()},
           "weights": {p: w for p, w in WEIGHTS.items() if w is not None},
           "tenants": tenants, "size": size, "sh": sh, "na": na, "ot": ot,
           "quotas": [[s.quota_initial, s.quota_min, s.quota_max, s.resolves] for s in shared[-1][0]],
           "clk": clk.summary(), "ta": ta, "iso_persist": [iso_persist[t] for t in tenants],
           "iso_static": [iso_static[t] for t in tenants] if iso_static else None,
           "roof": roof, "dom": dom, "h2d": sum(j.h2d_bytes() for j in jobs),
           "d2h": sum(j.d2h_bytes() for j in jobs), "launches_per_step": launches_per_step,
           "parity": {"shared_equals_native": all(parity.values()), "policies": sorted(parity)}}
    acc.close()
    return res, inputs


# ----------------------------------------------------------------- main
def main(argv=None):
    argv = sys.argv[1:] if argv is None else list(argv)
    ap = argparse.ArgumentParser()
    ap.add_argument("--gpus", type=int, default=1)
    ap.add_argument("--steps", type=int, default=10)
    ap.add_argument("--warmup", type=int, default=3)
    ap.add_argument("--config", default="c2", choices=["c1", "c2", "c5"])
    ap.add_argument("--impl", default="accel", choices=["accel", "reference"])
    ap.add_argument("--calib-reps", type=int, default=20)
    ap.add_argument("--policy", default="resolve", choices=["resolve", "static"],
                    help="SHARED-mode policy of the timed (headline) run; the others are reported too")
    ap.add_argument("--no-cpu-baseline", action="store_true")
    ap.add_argument("--out", default=None, help="also write the JSON line here")
    ap.add_argument("--hang-dump-s", type=float, default=0.0,
                    help="debug: dump every thread's Python stack after this many seconds")
    args = ap.parse_args(argv)
    if args.hang_dump_s > 0:
        import faulthandler
        faulthandler.dump_traceback_later(args.hang_dump_s, repeat=True)
    if args.impl == "reference":
        run_reference(args)
        return 0
    if "WORLD_SIZE" not in os.environ and args.gpus > 1:
        return spawn_ranks(args, argv)

    rank, world, local = env_rank()
    ranks = Ranks(rank, world)
    if os.environ.get("ACCEL_BENCH_STUB"):
        local_res, inputs = stub_rank(args, rank, world, ranks), None
    else:
        local_res, inputs = run_rank(args, rank, world, local, ranks)
    allres = ranks.gather(local_res)

    if rank == 0:
        cpu = None
        if not args.no_cpu_baseline:
            if inputs is None:
                cpu = {"value": None, "unit": UNIT, "cores": os.cpu_count(), "kind": "oracle", "sample": "stub"}
            else:
                cpu = cpu_baseline(local_res["tenants"], inputs)
        line = json.dumps(result_line(args, allres, world, cpu))
        print(line, flush=True)
        if args.out:
            with open(args.out, "w") as f:
                f.write(line + "\n")
    ranks.barrier()
    ranks.close()
    return 0


def result_line(args, allres, world, cpu) -> dict:
    r0 = allres[0]
    tenants, size = r0["tenants"], r0["size"]
    agg = aggregate(allres, world, args.steps, args.policy)
    tmax, emax, nmax, value = agg["tmax"], agg["emax"], agg["nmax"], agg["value"]
    U_sh, U_na, stp_sh, stp_na = agg["U_sh"], agg["U_na"], agg["stp_sh"], agg["stp_na"]
    antt_sh, antt_na, other_sum = agg["antt_sh"], agg["antt_na"], agg["other"]
    for p in other_sum:
        other_sum[p]["T_s_ms"] = dict(zip(tenants, np.mean(r0["ot"][p]["ts_ms"], 0).tolist()))
        if p in r0.get("weights", {}):
            other_sum[p]["weights"] = dict(zip(tenants, r0["weights"][p]))
    clocks = r0["clk"]
    dom = r0["dom"]
    roof = r0["roof"]
    overhead = {t: p / a - 1 for t, p, a in zip(tenants, r0["iso_persist"], r0["ta"])}
    overhead_st = ({t: p / a - 1 for t, p, a in zip(tenants, r0["iso_static"], r0["ta"])}
                   if r0.get("iso_static") else overhead)
    line = {
        "metric": METRIC, "value": value, "unit": UNIT, "n_gpus": world, "steps": args.steps,
        "warmup": args.warmup, "ms_per_step": tmax / args.steps, "higher_is_better": True,
        "scaling": "weak", "vs_baseline": None, "dtype": "f32+i32", "data": "synthetic",
        "config": {"workload": CONFIGS.get(args.config, {}).get("desc", "config 5 mix per GPU"),
                   "config": args.config, "tenants": [r["tenants"] for r in allres] if world > 1 else tenants,
                   "size": size, "mode": f"SHARED (accelOS persistent CTAs, {args.policy} quotas)",
                   "l2": "flushed before every step (256 MiB write)",
                   "parallelism": f"independent mix per GPU x{world} (gloo control plane, no data-path collective)"},
        "sharing": {
            "unfairness_shared": U_sh, "unfairness_native": U_na,
            "fairness_improvement": U_na / U_sh,
            "stp_shared": stp_sh, "stp_native": stp_na, "stp_ratio": stp_sh / stp_na,
            "antt_shared": antt_sh, "antt_native": antt_na,
            "throughput_speedup": nmax / tmax,
            "overlap_shared": statistics.mean(o for r in allres for o in r["sh"]["O"]),
            "overlap_native": statistics.mean(o for r in allres for o in r["na"]["O"]),
            "T_a_ms": dict(zip(tenants, r0["ta"])),
            "T_s_ms_shared": dict(zip(tenants, np.mean(r0["sh"]["ts_ms"], 0).tolist())),
            "T_s_ms_native": dict(zip(tenants, np.mean(r0["na"]["ts_ms"], 0).tolist())),
            "dispatch_overhead": overhead,
            "dispatch_overhead_static": overhead_st,
            "native_mixes_per_s": world * args.steps / (nmax / 1e3),
            "quotas_last_step": dict(zip(tenants, r0["quotas"])),
            "other_policies": other_sum,
            "per_rank": [{"rank": r["rank"], "U": statistics.mean(r["sh"]["U"]),
                          "STP": statistics.mean(r["sh"]["STP"]), "dev_ms": r["dev_ms"]} for r in allres]
            if world > 1 else None,
        },
        "parity": {"shared_equals_native": all(r["parity"]["shared_equals_native"] for r in allres),
                   "policies": r0["parity"].get("policies")},
        "e2e": {"value": world * args.steps / (emax / 1e3), "unit": UNIT,
                "h2d_bytes_per_step": sum(r["h2d"] for r in allres),
                "d2h_bytes_per_step": sum(r["d2h"] for r in allres)},
        "gpu_launches": sum(r["launches_per_step"] for r in allres) * args.steps,
        "roofline": dict(roof[dom], kernel=dom) if dom else None,
        "rooflines": roof,
        "cpu_baseline": cpu,
        "clocks": {"sm_mhz": clocks.get("sm_mhz"), "sm_max_mhz": clocks.get("sm_max_mhz"),
                   "reasons": clocks.get("reasons")},
    }
    # LAST (the driver keeps the tail of the line): the headline sharing
    # numbers against the BASELINE.json targets in a compact form
    line["headline"] = {
        "U_shared": round(U_sh, 3), "U_native": round(U_na, 3), "FI": round(U_na / U_sh, 3),
        "STP_ratio": round(stp_sh / stp_na, 4), "ANTT_ratio": round(antt_sh / antt_na, 4),
        "throughput_vs_native": round(nmax / tmax, 4),
        "max_dispatch_overhead": round(max(overhead.values()), 4) if overhead else None,
        "max_dispatch_overhead_static": round(max(overhead_st.values()), 4) if overhead_st else None,
        "targets": {"U<=1.5": U_sh <= 1.5, "STP>=native": stp_sh >= stp_na,
                    "overhead<=5%": bool(overhead) and max(overhead.values()) <= 0.05,
                    "overhead_static<=5%": bool(overhead_st) and max(overhead_st.values()) <= 0.05},
    }
    return line


if __name__ == "__main__":
    sys.exit(main())
