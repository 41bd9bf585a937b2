"""f1: the sharing-ratio lever of PAPER.md §2.2 lines
388-393 ("changing the sharing ratio") on one B200.

Runs a 4-tenant mix (default: BASELINE config 2, bfs + cutcp + stencil +
tpacf at default sizes, the bench's seeds) under SHARED-resolve with request
weights omega (accel_request.weight -> the solver's closed form, R-solver-7)
and reports U, STP and ANTT per weight vector, beside NATIVE and the
unweighted run.  Two families:

  rule   omega_i ~ T(a)_i ** alpha (a profile-guided rule, one alpha for every
         mix: alpha = 0 is the paper's equal share, alpha < 0 favours the
         shorter requests)
  grid   every vector in {1, 2, 3, 4}^K with min 1 (exhaustive: the best U
         reachable by static weights on this mix -- an upper bound on what a
         weight rule can do, NOT a policy)

    python scripts/weights.py [--config c2] [--reps 5] [--out gpurun_out/w.json]

Device-timed (accel_req_stats, CUDA events), L2 flushed before every run,
T(a) = NATIVE isolated median."""
from __future__ import annotations

import argparse
import itertools
import json
import os
import statistics
import sys

os.environ.setdefault("CUDA_DEVICE_MAX_CONNECTIONS", "32")
ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import torch  # noqa: E402

from bench import make_inputs  # noqa: E402
from paper_conf_cgo_margiolaso16_b200 import abi  # noqa: E402
from paper_conf_cgo_margiolaso16_b200.jobs import make_job  # noqa: E402
from paper_conf_cgo_margiolaso16_b200.runtime import Accel  # noqa: E402


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--config", default="c2")
    ap.add_argument("--reps", type=int, default=5)
    ap.add_argument("--grid", type=int, default=4, help="grid: weights 1..G per tenant (0 = no grid)")
    ap.add_argument("--out", default=None)
    args = ap.parse_args()
    dev = torch.device("cuda", 0)
    tenants, _, inputs = make_inputs(args.config, 0)
    jobs = [make_job(t, inputs[t], dev) for t in tenants]
    acc = Accel(device=0, mode=abi.MODE_SHARED)
    for j in jobs:
        if hasattr(j, "fit_levels"):
            j.fit_levels(acc)
    flush_buf = torch.empty(256 * 1024 * 1024 // 4, dtype=torch.float32, device=dev)

    def run(js, mode, weights=None):
        acc.set_mode(mode, abi.POLICY_RESOLVE)
        flush_buf.fill_(1.0)
        torch.cuda.synchronize()
        return [s.elapsed_ms for s in acc.run(js, weights=weights)]

    ta = []
    for j in jobs:
        run([j], abi.MODE_NATIVE)
        ta.append(statistics.median(run([j], abi.MODE_NATIVE)[0] for _ in range(args.reps)))

    def measure(mode, weights=None):
        run(jobs, mode, weights)   # warm-up
        U, STP, ANTT, TS = [], [], [], []
        for _ in range(args.reps):
            ts = run(jobs, mode, weights)
            m = abi.accel_metrics(ta, ts)
            U.append(m.unfairness)
            STP.append(m.stp)
            ANTT.append(m.antt)
            TS.append(ts)
        return {"U": statistics.median(U), "STP": statistics.median(STP), "ANTT": statistics.median(ANTT),
                "slowdown": [statistics.median(t[i] for t in TS) / ta[i] for i in range(len(ta))]}

    res = {"tenants": tenants, "T_a_ms": ta, "native": measure(abi.MODE_NATIVE),
           "equal": measure(abi.MODE_SHARED), "rule": {}, "grid": []}
    print("native", res["native"])
    print("equal ", res["equal"])
    # alpha < 0: shorter requests get larger shares (shortest-first within the
    # sharing); alpha > 0: longer ones do
    for alpha in (-1.0, -0.75, -0.5, -0.25, 0.25, 0.5, 1.0):
        w = [max(1, round(16 * (t / (min(ta) if alpha > 0 else max(ta))) ** alpha)) for t in ta]
        r = measure(abi.MODE_SHARED, w)
        r["weights"] = w
        res["rule"][str(alpha)] = r
        print(f"rule alpha={alpha} w={w}", {k: (round(v, 3) if isinstance(v, float) else [round(x, 2) for x in v])
                                            for k, v in r.items() if k != "weights"})
    if args.grid:
        for w in itertools.product(range(1, args.grid + 1), repeat=len(jobs)):
            if min(w) != 1:
                continue
            r = measure(abi.MODE_SHARED, list(w))
            r["weights"] = list(w)
            res["grid"].append(r)
        res["grid"].sort(key=lambda r: r["U"])
        for r in res["grid"][:8]:
            print("grid", r["weights"], round(r["U"], 3), round(r["STP"], 3), [round(x, 2) for x in r["slowdown"]])
    acc.close()
    if args.out:
        with open(args.out, "w") as f:
            json.dump(res, f, indent=1)


if __name__ == "__main__":
    main()
