"""C4 (8 staggered arrivals, RESOLVE) with per-VG traces: for every request,
VGs running per 0.5-ms bin and the mean VG duration per bin (where a
request's time goes in the staggered mix).
    python scripts/c4_trace.py [--reps 2]"""
import os
import statistics
import sys
import time

os.environ.setdefault("CUDA_DEVICE_MAX_CONNECTIONS", "32")
sys.path.insert(0, os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np  # noqa: E402
import torch  # noqa: E402

import mixes as M  # noqa: E402
from paper_conf_cgo_margiolaso16_b200 import abi  # noqa: E402

r = M.Runner(M.TENANTS, "default", torch.device("cuda", 0))
ta = r.isolated(2)
perm = np.random.Generator(np.random.PCG64(7)).permutation(len(M.TENANTS))
order = [M.TENANTS[i] for i in perm]
delta = 0.25 * statistics.median(ta.values()) / 1e3
jobs = [r.jobs[t][0] for t in order]
acc = r.acc
for rep in range(int(os.environ.get("REPS", 2))):
    r.set(abi.MODE_SHARED, abi.POLICY_RESOLVE)
    r.flush_buf.fill_(1.0)
    torch.cuda.synchronize()
    acc.epoch()
    ids = []
    t0 = time.perf_counter()
    for i, j in enumerate(jobs):
        while time.perf_counter() - t0 < i * delta:
            pass
        ids += acc.submit([j], tenants=[i], trace=True)
    acc.sync()
    st = [acc.stats(i) for i in ids]
    trs = [acc.vg_trace(i) for i in ids]
    acc.release()
    g0 = min(s.first_start_ns for s in st)
    print(f"===== rep {rep}")
    for t, s, tr in zip(order, st, trs):
        ran = tr[tr["t_start_ns"] > 0]
        a = (ran["t_start_ns"] - g0) / 1e6
        b = (ran["t_end_ns"] - g0) / 1e6
        end = float(b.max())
        bins = np.arange(0, end + 0.5, 0.5)
        conc = []
        for lo in bins:
            hi = lo + 0.5
            ov = np.clip(np.minimum(b, hi) - np.maximum(a, lo), 0, None).sum() / 0.5
            conc.append(ov)
        print(f"{t:8s} sd {s.elapsed_ms / ta[t]:5.2f} start {(s.first_start_ns - g0) / 1e6:6.2f} end {end:6.2f} ms "
              f"q0 {s.quota_initial} qmax {s.quota_max} vgs {len(ran)} vg_ms_med {float(np.median(b - a)):.3f}")
        print("    VGs running per 0.5 ms: " + " ".join(f"{c:.0f}" for c in conc))
