"""The paper's tiny-kernel case (E10): bfs, spmv and
tpacf with 2, 4 or 8 work-groups, NATIVE vs persistent STATIC / RESOLVE;
median request time (arrival -> done) over many repetitions.
    python scripts/tiny_grids.py [--reps 40]"""
import argparse
import json
import os
import statistics
import sys

os.environ.setdefault("CUDA_DEVICE_MAX_CONNECTIONS", "32")
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import synth  # noqa: E402
from paper_conf_cgo_margiolaso16_b200 import abi  # noqa: E402
from paper_conf_cgo_margiolaso16_b200.jobs import make_job  # noqa: E402
from paper_conf_cgo_margiolaso16_b200.runtime import Accel  # noqa: E402

# input sizes giving 2 / 4 / 8 VGs (bfs: per level at most; spmv: rows / 64;
# tpacf: ceil(npts/256) x (2 S + 1) x qsplit with S = 0 is not allowed, so
# npts = 256, S = 1, qsplit 1 -> 3 ... the nearest shapes are used and the
# actual VG count is printed)
CASES = {
    "bfs": [dict(nv=512), dict(nv=1024), dict(nv=2048)],
    "spmv": [dict(grid=11, iters=1), dict(grid=16, iters=1), dict(grid=22, iters=1)],
    "tpacf": [dict(npts=256, nsets=1, qsplit=1), dict(npts=256, nsets=1, qsplit=2),   # 3, 6 VGs
              dict(npts=512, nsets=1, qsplit=1)],                                      # 6 ... see vgs
}


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--reps", type=int, default=40)
    a = ap.parse_args()
    acc = Accel(0)
    out = []
    for t, cases in CASES.items():
        for over in cases:
            d = synth.preset(t, "tiny", **{k: v for k, v in over.items() if k != "qsplit"})
            if "qsplit" in over:
                d["qsplit"] = over["qsplit"]
            job = make_job(t, d)
            if hasattr(job, "fit_levels"):
                job.fit_levels(acc)
            st = job.steps[job.main_step if job.main_step >= 0 else 0]
            vgs = st.grid[0] * st.grid[1] * st.grid[2]
            res = {"tenant": t, "vgs": vgs, "launches": job.launches()}
            for name, mode, pol in [("native", abi.MODE_NATIVE, abi.POLICY_STATIC),
                                    ("static", abi.MODE_SHARED, abi.POLICY_STATIC),
                                    ("resolve", abi.MODE_SHARED, abi.POLICY_RESOLVE)]:
                acc.set_mode(mode, pol)
                el = []
                for _ in range(a.reps + 2):
                    torch.cuda.synchronize()
                    el.append(acc.run([job])[0].elapsed_ms)
                res[name + "_us"] = 1e3 * statistics.median(el[2:])
            res["static_vs_native"] = res["static_us"] / res["native_us"] - 1
            res["resolve_vs_native"] = res["resolve_us"] / res["native_us"] - 1
            out.append(res)
            print(json.dumps({k: (round(v, 4) if isinstance(v, float) else v) for k, v in res.items()}), flush=True)
    acc.close()


if __name__ == "__main__":
    main()
