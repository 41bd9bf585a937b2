"""BASELINE configs 3 and 4 on one B200:

  c3  all 64 ordered pairs of the 8 tenants at default sizes (self-pairs test
      "equal shares for identical kernels"), NATIVE vs SHARED-resolve vs
      SHARED-static; per mix U, STP, ANTT, makespan; per config the geometric
      means of the fairness improvement FI = U_native / U_shared, of the STP
      ratio and of the throughput speedup, their min / max, and the share of
      mixes with FI < 1 (the paper's E3 / E7 analogues, PAPER.md lines 958-962,
      1061-1064).
  c4  all 8 tenants, staggered arrivals t_i = i * D with D = 0.25 x the median
      isolated T(a), seeded arrival order (seed 7); quotas re-solved on every
      arrival and departure under RESOLVE; U, STP, ANTT and W.ANTT (the worst
      normalised turnaround, Tables 1-2) per mode.

    python scripts/mixes.py --config c3 [--reps 3] [--out gpurun_out/c3.json]
    python scripts/mixes.py --config c4 [--reps 5]

Device-timed with CUDA events (accel_req_stats), L2 flushed before every run,
inputs resident in HBM; T(a) = NATIVE isolated median.  Metric definitions:
oracle/metrics_ref.py, computed here with the library's accel_metrics."""
from __future__ import annotations

import argparse
import itertools
import json
import math
import os
import statistics
import sys
import time

os.environ.setdefault("CUDA_DEVICE_MAX_CONNECTIONS", "32")
ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import numpy as np  # noqa: E402
import torch  # noqa: E402

import synth  # noqa: E402
from paper_conf_cgo_margiolaso16_b200 import abi  # noqa: E402
from paper_conf_cgo_margiolaso16_b200.jobs import make_job  # noqa: E402
from paper_conf_cgo_margiolaso16_b200.runtime import Accel  # noqa: E402

TENANTS = ["bfs", "cutcp", "stencil", "tpacf", "histo", "spmv", "sgemm", "mriq"]
ALPHA = 0.0   # --alpha: SHARED-mode weights ~ T(a)^alpha (0 = equal shares, the paper's policy)
MODES = [("native", abi.MODE_NATIVE, abi.POLICY_STATIC), ("resolve", abi.MODE_SHARED, abi.POLICY_RESOLVE),
         ("static", abi.MODE_SHARED, abi.POLICY_STATIC), ("guided", abi.MODE_SHARED, abi.POLICY_RESOLVE)]
SHARED = ["resolve", "static", "guided"]
# "guided": RESOLVE with profile-guided sharing ratios (DESIGN.md R-solver-11)
# from the measured share profiles (scripts/share_profile.py)
PROFILE = os.path.join(ROOT, "profiles", "r2", "share_profile.json")
_prof = None


def guided_weights(names):
    global _prof
    if _prof is None:
        _prof = json.load(open(PROFILE))
    ms = [_prof["profile"][t]["ms"] for t in names]
    return abi.accel_guided_weights(_prof["fracs"], ms)[0]


def gm(xs):
    xs = [x for x in xs if x > 0]
    return math.exp(statistics.mean(math.log(x) for x in xs)) if xs else float("nan")


class Runner:
    def __init__(self, tenants, size, dev):
        self.dev = dev
        self.acc = Accel(device=dev.index or 0, mode=abi.MODE_SHARED)
        # two instances per tenant (self-pairs need distinct buffers)
        self.inputs = {t: synth.preset(t, size, seed=11) for t in tenants}
        self.jobs = {t: [make_job(t, self.inputs[t], dev), make_job(t, synth.preset(t, size, seed=12), dev)]
                     for t in tenants}
        for js in self.jobs.values():   # bfs: depth + 1 level launches (one probe run)
            for j in js:
                if hasattr(j, "fit_levels"):
                    j.fit_levels(self.acc)
        self.flush_buf = torch.empty(256 * 1024 * 1024 // 4, dtype=torch.float32, device=dev)

    def set(self, mode, policy):
        if self.acc.mode != mode or self.acc.policy != policy:
            self.acc.set_mode(mode, policy)

    def run(self, jobs, mode, policy, delays_s=None, weights=None):
        """Submit `jobs` (arrival order); delays_s[i] = host-side arrival offset;
        weights = sharing ratios, None = equal."""
        self.set(mode, policy)
        self.flush_buf.fill_(1.0)
        torch.cuda.synchronize()
        self.acc.epoch()
        ids = []
        if delays_s is None:
            ids = self.acc.submit(jobs, tenants=list(range(len(jobs))), weights=weights)
        else:
            t0 = time.perf_counter()
            for i, (j, dl) in enumerate(zip(jobs, delays_s)):
                while time.perf_counter() - t0 < dl:
                    pass
                ids += self.acc.submit([j], tenants=[i], weights=None if weights is None else [weights[i]])
        self.acc.sync()
        st = [self.acc.stats(i) for i in ids]
        self.acc.release()
        return st

    def instance(self, t: str, i: int):
        """The i-th instance of tenant t (its own buffers; mixes with repeated
        tenants need one per occurrence).  Instances >= 2 reuse the inputs of
        instance 0."""
        while len(self.jobs[t]) <= i:
            j = make_job(t, self.inputs[t], self.dev)
            if hasattr(j, "fit_levels"):
                j.fit_levels(self.acc)
            self.jobs[t].append(j)
        return self.jobs[t][i]

    def isolated(self, reps):
        ta = {}
        for t, (j, _) in self.jobs.items():
            xs = [self.run([j], abi.MODE_NATIVE, abi.POLICY_STATIC)[0].elapsed_ms for _ in range(reps + 1)][1:]
            ta[t] = statistics.median(xs)
        return ta


def mix_metrics(st, ta_list):
    ts = [s.elapsed_ms for s in st]
    m = abi.accel_metrics(ta_list, ts)
    mk = max(s.done_ms for s in st) - min(s.arrival_ms for s in st)
    ov = abi.accel_overlap([float(s.first_start_ns) for s in st], [float(s.last_end_ns) for s in st])
    return {"U": m.unfairness, "STP": m.stp, "ANTT": m.antt, "makespan_ms": mk, "O": ov,
            "WANTT": max(t / a for t, a in zip(ts, ta_list)), "ts_ms": ts}


def config3(r: Runner, ta, reps, only=None):
    mixes = []
    for a, b in (only or itertools.product(TENANTS, TENANTS)):
        ja = r.jobs[a][0]
        jb = r.jobs[b][1] if a == b else r.jobs[b][0]
        res = {"mix": [a, b]}
        for name, mode, pol in MODES:
            w = guided_weights([a, b]) if name == "guided" else None
            runs = [mix_metrics(r.run([ja, jb], mode, pol, weights=w), [ta[a], ta[b]]) for _ in range(reps)]
            res[name] = {k: statistics.mean(x[k] for x in runs) for k in ("U", "STP", "ANTT", "makespan_ms", "WANTT")}
        mixes.append(res)
        print(json.dumps({"mix": res["mix"], **{n: {k: round(v, 3) for k, v in res[n].items()} for n, _, _ in MODES}}),
              flush=True)
    out = {}
    for name in SHARED:
        fi = [m["native"]["U"] / m[name]["U"] for m in mixes]
        stp = [m[name]["STP"] / m["native"]["STP"] for m in mixes]
        thr = [m["native"]["makespan_ms"] / m[name]["makespan_ms"] for m in mixes]
        out[name] = {"U_gmean": gm([m[name]["U"] for m in mixes]),
                     "FI_gmean": gm(fi), "FI_min": min(fi), "FI_max": max(fi),
                     "FI_below_1_pct": 100.0 * sum(f < 1 for f in fi) / len(fi),
                     "STP_ratio_gmean": gm(stp), "throughput_speedup_gmean": gm(thr),
                     "throughput_speedup_min": min(thr), "throughput_speedup_max": max(thr),
                     "self_pairs_U_gmean": gm([m[name]["U"] for m in mixes if m["mix"][0] == m["mix"][1]])}
    out["native"] = {"U_gmean": gm([m["native"]["U"] for m in mixes])}
    return mixes, out


def config4(r: Runner, ta, reps):
    perm = np.random.Generator(np.random.PCG64(7)).permutation(len(TENANTS))
    order = [TENANTS[i] for i in perm]
    delta = 0.25 * statistics.median(ta.values()) / 1e3
    delays = [i * delta for i in range(len(order))]
    jobs = [r.jobs[t][0] for t in order]
    tal = [ta[t] for t in order]
    out = {"order": order, "delta_ms": delta * 1e3}
    for name, mode, pol in MODES:
        w = guided_weights(order) if name == "guided" else None
        runs = [mix_metrics(r.run(jobs, mode, pol, delays, weights=w), tal) for _ in range(reps)]
        out[name] = {k: statistics.mean(x[k] for x in runs) for k in ("U", "STP", "ANTT", "WANTT", "makespan_ms")}
        out[name]["slowdowns"] = dict(zip(order, [statistics.mean(x["ts_ms"][i] for x in runs) / tal[i]
                                                  for i in range(len(order))]))
        print(name, json.dumps({k: (round(v, 3) if isinstance(v, float) else v) for k, v in out[name].items()}),
              flush=True)
    for name in SHARED:
        out[name]["FI"] = out["native"]["U"] / out[name]["U"]
        out[name]["STP_ratio"] = out[name]["STP"] / out["native"]["STP"]
        out[name]["throughput_speedup"] = out["native"]["makespan_ms"] / out[name]["makespan_ms"]
    return out


def sampled(r: Runner, ta, reps, k, n, seed, repeat=False):
    """n seeded random ordered k-tuples of the tenants,
    submitted together -- distinct tenants, or (repeat=True, the paper's
    sampling space: ordered tuples with repetition)
    any tenant any number of times, each occurrence its own instance;
    geometric means as in c3."""
    g = np.random.Generator(np.random.PCG64(seed))
    mixes = []
    keys = ("U", "STP", "ANTT", "makespan_ms", "WANTT", "O")
    for _ in range(n):
        if repeat:
            names = [TENANTS[i] for i in g.integers(0, len(TENANTS), k)]
        else:
            names = [TENANTS[i] for i in g.permutation(len(TENANTS))[:k]]
        seen: dict[str, int] = {}
        jobs = []
        for t in names:
            jobs.append(r.instance(t, seen.get(t, 0)))
            seen[t] = seen.get(t, 0) + 1
        res = {"mix": names}
        for name, mode, pol in MODES:
            w = guided_weights(names) if name == "guided" else None
            if ALPHA and mode == abi.MODE_SHARED and name != "guided":
                # profile-guided sharing ratio: w ~ T(a)^alpha (alpha < 0: the
                # shorter requests get the larger shares)
                tmax = max(ta[t] for t in names)
                w = [max(1, round(16 * (ta[t] / tmax) ** ALPHA)) for t in names]
            runs = [mix_metrics(r.run(jobs, mode, pol, weights=w), [ta[t] for t in names]) for _ in range(reps)]
            res[name] = {kk: statistics.mean(x[kk] for x in runs) for kk in keys}
            # per-tenant slowdowns T(s)/T(a) (which tenant sets U)
            res[name]["s"] = [statistics.mean(x["ts_ms"][i] for x in runs) / ta[t] for i, t in enumerate(names)]
        mixes.append(res)
        print(json.dumps({"mix": names, **{nm: {kk: (round(v, 3) if kk != "s" else [round(x, 3) for x in v])
                                                 for kk, v in res[nm].items()} for nm, _, _ in MODES}}),
              flush=True)
    out = {}
    for name in SHARED:
        fi = [m["native"]["U"] / m[name]["U"] for m in mixes]
        out[name] = {"U_gmean": gm([m[name]["U"] for m in mixes]), "FI_gmean": gm(fi),
                     "FI_min": min(fi), "FI_max": max(fi),
                     "FI_below_1_pct": 100.0 * sum(f < 1 for f in fi) / len(fi),
                     "STP_ratio_gmean": gm([m[name]["STP"] / m["native"]["STP"] for m in mixes]),
                     "throughput_speedup_gmean": gm([m["native"]["makespan_ms"] / m[name]["makespan_ms"]
                                                     for m in mixes]),
                     "WANTT_max": max(m[name]["WANTT"] for m in mixes),
                     "ANTT_gmean": gm([m[name]["ANTT"] for m in mixes]),
                     "O_mean": statistics.mean(m[name]["O"] for m in mixes),
                     # BASELINE.json target for 4-tenant mixes: U <= 1.5 and STP >= native
                     "target_met_pct": 100.0 * sum(m[name]["U"] <= 1.5 and m[name]["STP"] >= m["native"]["STP"]
                                                   for m in mixes) / len(mixes),
                     "U_le_1.5_pct": 100.0 * sum(m[name]["U"] <= 1.5 for m in mixes) / len(mixes),
                     "STP_ge_native_pct": 100.0 * sum(m[name]["STP"] >= m["native"]["STP"] for m in mixes) / len(mixes)}
    out["native"] = {"U_gmean": gm([m["native"]["U"] for m in mixes]),
                     "WANTT_max": max(m["native"]["WANTT"] for m in mixes),
                     "ANTT_gmean": gm([m["native"]["ANTT"] for m in mixes]),
                     "O_mean": statistics.mean(m["native"]["O"] for m in mixes)}
    return mixes, out


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--config", default="c3", choices=["c3", "c4", "f2"])
    ap.add_argument("--k", type=int, default=4, help="f2: tenants per mix")
    ap.add_argument("--n", type=int, default=32, help="f2: number of sampled mixes")
    ap.add_argument("--seed", type=int, default=2024)
    ap.add_argument("--repeat", action="store_true", help="f2: tuples with repetition (the paper's space)")
    ap.add_argument("--alpha", type=float, default=0.0, help="f2: SHARED weights ~ T(a)^alpha (0 = equal)")
    ap.add_argument("--reps", type=int, default=3)
    ap.add_argument("--size", default="default")
    ap.add_argument("--out", default=None)
    ap.add_argument("--only", default=None, help="c3: comma-separated a:b pairs, e.g. mriq:mriq,cutcp:sgemm")
    ap.add_argument("--tenants", default=None, help="restrict the tenants loaded (comma-separated)")
    ap.add_argument("--modes", default=None, help="restrict the modes (comma-separated; native is always run)")
    a = ap.parse_args()
    global ALPHA
    ALPHA = a.alpha
    dev = torch.device("cuda", 0)
    if a.tenants:
        TENANTS[:] = a.tenants.split(",")
    if a.modes:
        keep = set(a.modes.split(",")) | {"native"}
        MODES[:] = [m for m in MODES if m[0] in keep]
        SHARED[:] = [n for n in SHARED if n in keep]
    r = Runner(TENANTS, a.size, dev)
    # warm every tenant in every mode once (module load, first touch)
    for t, (j, _) in r.jobs.items():
        for _, mode, pol in MODES:
            r.run([j], mode, pol)
    ta = r.isolated(max(3, a.reps))
    print("T(a) ms", json.dumps({k: round(v, 3) for k, v in ta.items()}), flush=True)
    res = {"config": a.config, "size": a.size, "reps": a.reps, "T_a_ms": ta}
    if a.config == "c3":
        only = [tuple(p.split(":")) for p in a.only.split(",")] if a.only else None
        mixes, summ = config3(r, ta, a.reps, only)
        res.update({"mixes": mixes, "summary": summ})
        print("SUMMARY", json.dumps(summ), flush=True)
    elif a.config == "f2":
        mixes, summ = sampled(r, ta, a.reps, a.k, a.n, a.seed, a.repeat)
        res.update({"mixes": mixes, "summary": summ, "k": a.k, "n": a.n, "seed": a.seed, "repeat": a.repeat})
        print("SUMMARY", json.dumps(summ), flush=True)
    else:
        res["summary"] = config4(r, ta, a.reps)
        print("SUMMARY", json.dumps(res["summary"]), flush=True)
    if a.out:
        json.dump(res, open(a.out, "w"), indent=1)
    r.acc.close()


if __name__ == "__main__":
    main()
