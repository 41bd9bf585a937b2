"""Stencil bandwidth vs volume: the same kernel on larger volumes, to
separate its streaming rate from the fixed per-launch cost (ramp-up, tail
of the last VG wave, launch gap) that a ~30 us launch of the default
512 x 512 x 64 volume pays.  Algorithmic bytes = 8 B per point per sweep.

    python scripts/stencil_size.py [--sizes 512x512x64,1024x1024x64,...] [--sweeps 20]
"""
import argparse
import os
import statistics
import sys

os.environ.setdefault("CUDA_DEVICE_MAX_CONNECTIONS", "32")
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import json  # noqa: E402

import torch  # noqa: E402

import synth  # noqa: E402
from paper_conf_cgo_margiolaso16_b200 import abi  # noqa: E402
from paper_conf_cgo_margiolaso16_b200.jobs import make_job  # noqa: E402
from paper_conf_cgo_margiolaso16_b200.runtime import Accel  # noqa: E402


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--sizes", default="512x512x64,1024x512x64,1024x1024x64,1024x1024x128")
    ap.add_argument("--sweeps", type=int, default=20)
    ap.add_argument("--reps", type=int, default=5)
    a = ap.parse_args()
    peak = json.load(open(os.path.join(os.path.dirname(os.path.dirname(os.path.abspath(__file__))), "MEASURED_PEAKS.json")))["hbm_gbs"]
    acc = Accel(0)
    flush = torch.empty(64 * 1024 * 1024, dtype=torch.float32, device="cuda")
    for s in a.sizes.split(","):
        nx, ny, nz = (int(v) for v in s.split("x"))
        d = synth.preset("stencil", "default", seed=1, nx=nx, ny=ny, nz=nz, sweeps=a.sweeps)
        job = make_job("stencil", d)
        line = f"{s:14s}"
        for name, mode, pol in [("native", abi.MODE_NATIVE, abi.POLICY_STATIC), ("static", abi.MODE_SHARED, abi.POLICY_STATIC),
                                ("resolve", abi.MODE_SHARED, abi.POLICY_RESOLVE)]:
            acc.set_mode(mode, pol)
            lt = []
            for _ in range(a.reps + 1):
                flush.fill_(1)
                torch.cuda.synchronize()
                ids = acc.submit([job], launch_events=True)
                acc.sync()
                lt.append(acc.launch_times(ids[0], job.launches()))
                acc.release()
            us = statistics.median([statistics.mean(x) for x in lt[1:]]) * 1e3
            gbs = 8.0 * nx * ny * nz / (us * 1e-6) / 1e9
            line += f"  {name} {us:7.1f} us/launch {gbs:6.0f} GB/s ({gbs / peak:.2f})"
        # a plain device copy of one volume (read + write = the same 8 B per
        # point), back to back, for the size-matched bandwidth ceiling
        x = torch.ones(nx * ny * nz, device="cuda")
        y = torch.empty_like(x)
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        for _ in range(3):
            y.copy_(x)
        e0.record()
        for _ in range(a.sweeps):
            y.copy_(x)
            x, y = y, x
        e1.record()
        torch.cuda.synchronize()
        us = e0.elapsed_time(e1) * 1e3 / a.sweeps
        gbs = 8.0 * nx * ny * nz / (us * 1e-6) / 1e9
        line += f"  torch-copy {us:7.1f} us {gbs:6.0f} GB/s ({gbs / peak:.2f})"
        print(line, flush=True)


if __name__ == "__main__":
    main()
