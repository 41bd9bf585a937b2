"""Timeline of one mix: per request, per launch device stamps (us from the
first start), admitted-CTA high-water mark and top-up flag.
    python scripts/timeline.py [native|static|resolve] [config]"""
import os
import sys

os.environ.setdefault("CUDA_DEVICE_MAX_CONNECTIONS", "32")
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import bench  # noqa: E402
from paper_conf_cgo_margiolaso16_b200 import abi  # noqa: E402
from paper_conf_cgo_margiolaso16_b200.jobs import make_job  # noqa: E402
from paper_conf_cgo_margiolaso16_b200.runtime import Accel  # noqa: E402

mode = sys.argv[1] if len(sys.argv) > 1 else "resolve"
cfg = sys.argv[2] if len(sys.argv) > 2 else "c2"
if "," in cfg:   # an ad-hoc mix of default-size tenants, e.g. sgemm,spmv
    import synth  # noqa: E402
    tenants = cfg.split(",")
    inputs = {t: synth.preset(t, "default", seed=11 + i) for i, t in enumerate(tenants)}
else:
    tenants, size, inputs = bench.make_inputs(cfg, 0)
jobs = [make_job(t, inputs[t]) for t in tenants]
m, p = {"native": (abi.MODE_NATIVE, abi.POLICY_STATIC), "static": (abi.MODE_SHARED, abi.POLICY_STATIC),
        "resolve": (abi.MODE_SHARED, abi.POLICY_RESOLVE)}[mode]
acc = Accel(0, mode=m, policy=p)
for j in jobs:
    if hasattr(j, "fit_levels"):
        j.fit_levels(acc)
for rep in range(3):
    ids = acc.submit(jobs)
    acc.sync()
    st = [acc.stats(i) for i in ids]
    ls = [acc.launch_stats(i, j.launches()) for i, j in zip(ids, jobs)]
    acc.release()
t0 = min(s.first_start_ns for s in st)
for t, s, l in zip(tenants, st, ls):
    print(f"{t:8s} T(s)={s.elapsed_ms:7.3f} ms start={(s.first_start_ns - t0) / 1e3:8.1f} "
          f"end={(s.last_end_ns - t0) / 1e3:8.1f} us q0={s.quota_initial} qmin={s.quota_min} "
          f"qmax={s.quota_max} resolves={s.resolves}")
    step = max(1, len(l) // int(os.environ.get("TL_LINES", "12")))
    for i in range(0, len(l), step):
        x = l[i]
        print(f"    launch {i:3d}: {(x.t_first_ns - t0) / 1e3:8.1f} .. {(x.t_last_ns - t0) / 1e3:8.1f} us "
              f"ctas={x.ctas_started:4d} max_alive={x.max_alive:4d} total={x.total} topped={x.topped}")
acc.close()
