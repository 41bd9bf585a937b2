"""C4 RESOLVE/STATIC repeated; for reps whose U exceeds a threshold, print
every request's device start/end, quotas and per-launch stats (which request
stalls, and how many CTAs it had)."""
import os
import statistics
import sys

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
TRACE = bool(os.environ.get("TRACE"))
pol = abi.POLICY_STATIC if os.environ.get("POL") == "static" else abi.POLICY_RESOLVE
shown = 0
for rep in range(int(os.environ.get("REPS", 40))):
    r.set(abi.MODE_SHARED, pol)
    r.flush_buf.fill_(1.0)
    torch.cuda.synchronize()
    r.acc.epoch()
    ids = []
    import time
    t0 = time.perf_counter()
    for i, j in enumerate(jobs):
        while time.perf_counter() - t0 < i * delta:
            pass
        ids += r.acc.submit([j], tenants=[i], trace=TRACE)
    r.acc.sync()
    st = [r.acc.stats(i) for i in ids]
    ls = [r.acc.launch_stats(i, j.launches()) for i, j in zip(ids, jobs)]
    trs = {t: r.acc.vg_trace(i) for t, i in zip(order, ids) if TRACE and t in ("cutcp", "mriq")}
    r.acc.release()
    sd = [s.elapsed_ms / ta[t] for s, t in zip(st, order)]
    U = max(sd) / min(sd)
    print(f"rep {rep} U {U:.2f}", flush=True)
    if U > 9 and shown < 2:
        shown += 1
        g0 = min(s.first_start_ns for s in st)
        for t, s, l, x in zip(order, st, ls, sd):
            print(f"   {t:8s} sd {x:6.2f} arr {s.arrival_ms:7.3f} start {(s.first_start_ns - g0) / 1e6:7.3f} end {(s.last_end_ns - g0) / 1e6:7.3f}"
                  f" q0 {s.quota_initial} qmin {s.quota_min} qmax {s.quota_max} res {s.resolves} launches {len(l)}")
            if t in trs:
                tr = trs[t]
                ran = tr[tr["t_start_ns"] > 0]
                a = (ran["t_start_ns"] - g0) / 1e6
                b = (ran["t_end_ns"] - g0) / 1e6
                first = {}
                for c, x in zip(ran["cta"], a):
                    first[int(c)] = min(first.get(int(c), 1e9), float(x))
                fs = np.array(sorted(first.values()))
                k = int(np.argmax(b))
                print(f"      trace: {len(ran)} VGs, {len(first)} CTAs; CTA first-VG start p50 {np.median(fs):.3f} p90 {fs[int(.9*len(fs))]:.3f} max {fs.max():.3f} ms;"
                      f" VG ms p50 {float(np.median(b - a)):.3f} max {float((b - a).max()):.3f}; last VG {int(ran['cta'][k])} cta start {float(a[k]):.3f} end {float(b[k]):.3f}"
                      f" (that CTA's first VG at {first[int(ran['cta'][k])]:.3f}); VGs ending after 14 ms: {int((b > 14).sum())}")
            if t in ("cutcp", "mriq", "tpacf"):
                for k, y in enumerate(l):
                    print(f"      launch {k}: {(y.t_first_ns - g0) / 1e6:7.3f} .. {(y.t_last_ns - g0) / 1e6:7.3f} ctas {y.ctas_started} max_alive {y.max_alive} total {y.total} topped {y.topped}")
