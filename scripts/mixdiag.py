"""Per-tenant view of a few mixes (slowdown, quotas, start/end on the device
clock): which tenant sets U.

    python scripts/mixdiag.py mriq,bfs,cutcp,mriq mriq,bfs [--reps 3]
"""
import argparse
import json
import os
import statistics
import sys

os.environ.setdefault("CUDA_DEVICE_MAX_CONNECTIONS", "32")
sys.path.insert(0, os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import mixes as M  # noqa: E402
from paper_conf_cgo_margiolaso16_b200 import abi  # noqa: E402


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("mixes", nargs="+")
    ap.add_argument("--reps", type=int, default=3)
    ap.add_argument("--weights", default=None, help="SHARED weights per mix position, e.g. 1,4")
    a = ap.parse_args()
    mixes = [m.split(",") for m in a.mixes]
    tenants = sorted({t for m in mixes for t in m})
    r = M.Runner(tenants, "default", torch.device("cuda", 0))
    for t, (j, _) in r.jobs.items():
        for _, mode, pol in M.MODES:
            r.run([j], mode, pol)
    ta = r.isolated(3)
    print("T(a) ms", json.dumps({k: round(v, 3) for k, v in ta.items()}))
    for names in mixes:
        seen = {}
        jobs = []
        for t in names:
            jobs.append(r.instance(t, seen.get(t, 0)))
            seen[t] = seen.get(t, 0) + 1
        for name, mode, pol in M.MODES:
            rows = []
            for _ in range(a.reps):
                w = [int(x) for x in a.weights.split(",")] if a.weights and mode == abi.MODE_SHARED else None
                st = r.run(jobs, mode, pol, weights=w)
                t0 = min(s.first_start_ns for s in st)
                rows.append([(s.elapsed_ms, (s.first_start_ns - t0) / 1e6, (s.last_end_ns - t0) / 1e6,
                              s.quota_initial, s.quota_min, s.quota_max, s.launches) for s in st])
            print(f"== {names} {name}")
            sl = []
            for i, t in enumerate(names):
                el = statistics.median(x[i][0] for x in rows)
                x = rows[-1][i]
                sl.append(el / ta[t])
                print(f"  {t:8s} T_s {el:8.3f} ms  slowdown {el / ta[t]:6.2f}  start {x[1]:7.3f} end {x[2]:7.3f}"
                      f"  quota init/min/max {x[3]}/{x[4]}/{x[5]}  launches {x[6]}")
            print(f"  U {max(sl) / min(sl):.2f}")


if __name__ == "__main__":
    main()
