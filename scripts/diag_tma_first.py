"""First sweep count at which the TMA stencil next to bfs differs from the
cp.async reference, and what the wrong values look like (got vs the
reference after T, T-1 and T-2 sweeps at the same points).
    python scripts/diag_tma_first.py [--max-sweeps 12] [--mode resolve]"""
import argparse
import os
import sys

os.environ.setdefault("CUDA_DEVICE_MAX_CONNECTIONS", "32")
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np  # noqa: E402

import bench  # noqa: E402
from paper_conf_cgo_margiolaso16_b200 import abi  # noqa: E402
from paper_conf_cgo_margiolaso16_b200.jobs import StencilJob, make_job  # noqa: E402
from paper_conf_cgo_margiolaso16_b200.runtime import Accel  # noqa: E402

ap = argparse.ArgumentParser()
ap.add_argument("--max-sweeps", type=int, default=12)
ap.add_argument("--mode", default="resolve")
ap.add_argument("--reps", type=int, default=6)
ap.add_argument("--kernel", default="stencil_tma")
a = ap.parse_args()
_, _, inp = bench.make_inputs("c2", 0)
acc = Accel(0)
acc.set_mode(abi.MODE_NATIVE, abi.POLICY_STATIC)
ref = {}
for t in range(1, a.max_sweeps + 1):
    j = StencilJob(dict(inp["stencil"], sweeps=t), kernel="stencil")
    acc.run([j])
    ref[t] = j.result()["a"]
ref[0] = inp["stencil"]["a0"]
bfs = make_job("bfs", inp["bfs"])
bfs.fit_levels(acc)
m = {"native": (abi.MODE_NATIVE, abi.POLICY_STATIC), "static": (abi.MODE_SHARED, abi.POLICY_STATIC),
     "resolve": (abi.MODE_SHARED, abi.POLICY_RESOLVE)}[a.mode]
acc.set_mode(*m)
for t in range(1, a.max_sweeps + 1):
    bad_reps = 0
    for rep in range(a.reps):
        sj = StencilJob(dict(inp["stencil"], sweeps=t), kernel=a.kernel)
        acc.run([bfs, sj])
        got = sj.result()["a"]
        bad = np.argwhere(got != ref[t])
        if len(bad):
            bad_reps += 1
            if bad_reps == 1:
                zs = sorted(set(int(z) for z in bad[:, 0]))
                print(f"sweeps {t} rep {rep}: {len(bad)} points differ, z planes {zs[:12]}", flush=True)
                for z, y, x in bad[:6]:
                    print(f"    ({z},{y},{x}) got {got[z, y, x]:.9g} want {ref[t][z, y, x]:.9g} "
                          f"T-1 {ref[t - 1][z, y, x]:.9g} T-2 {ref[max(t - 2, 0)][z, y, x]:.9g}", flush=True)
    print(f"sweeps {t}: {bad_reps}/{a.reps} reps differ", flush=True)
