"""Does a persistent compute-bound co-runner that arrived first starve a later
one's warps?  mri-q (or another tenant) first, the second tenant `delay_ms`
later; per-VG trace of the second: VG duration distribution.
    python scripts/starve.py [first] [second] [delay_ms]"""
import os
import sys
import time

os.environ.setdefault("CUDA_DEVICE_MAX_CONNECTIONS", "32")
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np  # noqa: E402
import torch  # noqa: E402

import synth  # noqa: E402
from paper_conf_cgo_margiolaso16_b200 import abi  # noqa: E402
from paper_conf_cgo_margiolaso16_b200.jobs import make_job  # noqa: E402
from paper_conf_cgo_margiolaso16_b200.runtime import Accel  # noqa: E402

first = sys.argv[1] if len(sys.argv) > 1 else "mriq"
second = sys.argv[2] if len(sys.argv) > 2 else "cutcp"
delay = float(sys.argv[3]) if len(sys.argv) > 3 else 1.0
a = make_job(first, synth.preset(first, "default", seed=3))
b = make_job(second, synth.preset(second, "default", seed=4))
acc = Accel(0)
for name, mode, pol in [("native", abi.MODE_NATIVE, abi.POLICY_STATIC), ("static", abi.MODE_SHARED, abi.POLICY_STATIC),
                        ("resolve", abi.MODE_SHARED, abi.POLICY_RESOLVE)]:
    acc.set_mode(mode, pol)
    for rep in range(4):
        torch.cuda.synchronize()
        t0 = time.perf_counter()
        ids = acc.submit([a], tenants=[0], trace=True)
        while time.perf_counter() - t0 < delay / 1e3:
            pass
        ids += acc.submit([b], tenants=[1], trace=True)
        acc.sync()
        st = [acc.stats(i) for i in ids]
        tr = acc.vg_trace(ids[1])
        acc.release()
        ran = tr[tr["t_start_ns"] > 0]
        d = (ran["t_end_ns"] - ran["t_start_ns"]) / 1e6
        g0 = min(s.first_start_ns for s in st)
        print(f"{name:8s} rep {rep}: {first} {(st[0].first_start_ns - g0) / 1e6:.2f}..{(st[0].last_end_ns - g0) / 1e6:.2f} ms "
              f"q {st[0].quota_initial}; {second} {(st[1].first_start_ns - g0) / 1e6:.2f}..{(st[1].last_end_ns - g0) / 1e6:.2f} ms "
              f"q {st[1].quota_initial}; VG ms p50 {np.median(d):.3f} p99 {np.percentile(d, 99):.3f} max {d.max():.3f}, "
              f"VGs > 2 ms: {int((d > 2).sum())}", flush=True)
acc.close()
