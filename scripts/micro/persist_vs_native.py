"""Persistent kernel with quota = G (one VG per CTA) vs quota = occupancy vs native."""
import os, sys, statistics
os.environ.setdefault("CUDA_DEVICE_MAX_CONNECTIONS", "32")
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.dirname(os.path.abspath(__file__)))))
import torch, synth
from paper_conf_cgo_margiolaso16_b200 import abi
from paper_conf_cgo_margiolaso16_b200.jobs import make_job
from paper_conf_cgo_margiolaso16_b200.runtime import Accel
t = sys.argv[1] if len(sys.argv) > 1 else "spmv"
d = synth.preset(t, "default", seed=1)
for label, caps, mode in [("native", None, abi.MODE_NATIVE), ("persist_occ", None, abi.MODE_SHARED),
                          ("persist_G", abi.accel_caps(4000, 0, 0, 0, 0), abi.MODE_SHARED),
                          ("persist_half", abi.accel_caps(74, 0, 0, 0, 0), abi.MODE_SHARED),
                          ("persist_2x", abi.accel_caps(296, 0, 0, 0, 0), abi.MODE_SHARED)]:
    acc = Accel(0, mode=mode, caps=caps)
    job = make_job(t, d)
    ts = []
    for _ in range(4):
        ids = acc.submit([job], launch_events=True)
        acc.sync()
        s = acc.stats(ids[0])
        lt = acc.launch_times(ids[0], job.launches())
        acc.release()
        ts.append(statistics.mean(lt))
    print(f"{t} {label:12s} quota={s.quota_initial:6d} launch={1e3*statistics.median(ts[1:]):8.1f} us")
    acc.close()
