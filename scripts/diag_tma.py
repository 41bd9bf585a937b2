"""Diagnose SHARED != NATIVE for the TMA stencil in mixes: which co-runners
trigger it, how many elements differ, and whether the wrong values are those
of an earlier sweep (a stale read) or something else.

    python scripts/diag_tma.py [--sweeps 100] [--reps 3]
"""
import argparse
import os
import sys

os.environ.setdefault("CUDA_DEVICE_MAX_CONNECTIONS", "32")
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np  # noqa: E402
import torch  # noqa: E402

import bench  # noqa: E402
import synth  # noqa: E402
from paper_conf_cgo_margiolaso16_b200 import abi  # noqa: E402
from paper_conf_cgo_margiolaso16_b200.jobs import StencilJob, make_job  # noqa: E402
from paper_conf_cgo_margiolaso16_b200.runtime import Accel  # noqa: E402


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--sweeps", type=int, default=100)
    ap.add_argument("--reps", type=int, default=3)
    ap.add_argument("--kernel", default="stencil_tma")
    ap.add_argument("--global-maps", action="store_true")
    ap.add_argument("--combos", default="-,bfs,bfs+cutcp+tpacf")
    a = ap.parse_args()
    _, _, inp = bench.make_inputs("c2", 0)
    ds = dict(inp["stencil"], sweeps=a.sweeps, tma_global_maps=a.global_maps)
    acc = Accel(0)
    # reference: stencil alone, NATIVE, for T and T-1, T-2 sweeps
    acc.set_mode(abi.MODE_NATIVE, abi.POLICY_STATIC)
    ref = {}
    for t in (a.sweeps, a.sweeps - 1, a.sweeps - 2):
        j = StencilJob(dict(ds, sweeps=t), kernel="stencil")
        acc.run([j])
        ref[t] = j.result()["a"]
    others = {n: make_job(n, inp[n]) for n in ("bfs", "cutcp", "tpacf")}
    others["bfs"].fit_levels(acc)
    combos = [[] if c == "-" else c.split("+") for c in a.combos.split(",")]
    for pol_name, mode, pol in [("native", abi.MODE_NATIVE, abi.POLICY_STATIC), ("static", abi.MODE_SHARED, abi.POLICY_STATIC),
                                ("resolve", abi.MODE_SHARED, abi.POLICY_RESOLVE)]:
        acc.set_mode(mode, pol)
        for co in combos:
            for rep in range(a.reps):
                sj = StencilJob(ds, kernel=a.kernel)
                jobs = [others[n] for n in co[:1]] + [sj] + [others[n] for n in co[1:]]
                acc.run(jobs)
                got = sj.result()["a"]
                bad = got != ref[a.sweeps]
                msg = f"{pol_name:8s} co={'+'.join(co) or '-':18s} rep {rep}: differ {int(bad.sum())}"
                if bad.any():
                    z, y, x = np.nonzero(bad)
                    msg += (f" z[{z.min()},{z.max()}] y[{y.min()},{y.max()}] x[{x.min()},{x.max()}]"
                            f" maxdiff {float(np.abs(got - ref[a.sweeps])[bad].max()):.3g}")
                    for t in (a.sweeps - 1, a.sweeps - 2):
                        msg += f" eq_T-{a.sweeps - t}: {int((got[bad] == ref[t][bad]).sum())}"
                    tiles = {(int(zz) // 8, int(yy) // 8, int(xx) // 128) for zz, yy, xx in zip(z, y, x)}
                    msg += f" tiles {len(tiles)}"
                print(msg, flush=True)


if __name__ == "__main__":
    main()
