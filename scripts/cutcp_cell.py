"""cutcp: isolated time vs the atom-binning cell edge (an input layout: the
body walks the cell rows within the cutoff, so smaller cells test fewer
out-of-cutoff pairs but visit more rows).  Outputs of every cell size are
compared with the 4-A layout (R-tol-1 tolerance: only the summation order
differs).

    python scripts/cutcp_cell.py [--cells 4,3,2] [--reps 5]
"""
import argparse
import os
import statistics
import sys

os.environ.setdefault("CUDA_DEVICE_MAX_CONNECTIONS", "32")
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np  # noqa: E402
import torch  # noqa: E402

import synth  # noqa: E402
from paper_conf_cgo_margiolaso16_b200 import abi  # noqa: E402
from paper_conf_cgo_margiolaso16_b200.jobs import make_job  # noqa: E402
from paper_conf_cgo_margiolaso16_b200.runtime import Accel  # noqa: E402


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--cells", default="4,3,2")
    ap.add_argument("--reps", type=int, default=5)
    a = ap.parse_args()
    acc = Accel(0)
    flush = torch.empty(64 * 1024 * 1024, dtype=torch.float32, device="cuda")
    ref = None
    for cell in [float(c) for c in a.cells.split(",")]:
        d = synth.preset("cutcp", "default", seed=1, cell=cell)
        job = make_job("cutcp", d)
        line = f"cell {cell:3.1f}"
        for name, mode, pol in [("native", abi.MODE_NATIVE, abi.POLICY_STATIC), ("static", abi.MODE_SHARED, abi.POLICY_STATIC),
                                ("resolve", abi.MODE_SHARED, abi.POLICY_RESOLVE)]:
            acc.set_mode(mode, pol)
            el = []
            for _ in range(a.reps + 1):
                flush.fill_(1)
                torch.cuda.synchronize()
                ids = acc.submit([job])
                acc.sync()
                el.append(acc.stats(ids[0]).elapsed_ms)
                acc.release()
            line += f"  {name} {statistics.median(el[1:]):.3f} ms"
        v = job.result()["v"].astype(np.float64)
        if ref is None:
            ref = v
        else:
            tol = 1e-4 * np.maximum(np.abs(ref), 1e-2 * np.abs(ref).max())
            line += f"  max|d|/tol vs 4A {float((np.abs(v - ref) / tol).max()):.3f}"
        print(line, flush=True)


if __name__ == "__main__":
    main()
