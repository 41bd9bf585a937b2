"""Isolated per-launch timing of the stencil kernels (NATIVE, STATIC,
RESOLVE; default size, 100 sweeps): CUDA events around every launch on the
tenant stream, L2 flushed before each request; algorithmic 8 B/point."""
import os
import statistics
import sys

os.environ.setdefault("CUDA_DEVICE_MAX_CONNECTIONS", "32")
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import synth  # noqa: E402
from paper_conf_cgo_margiolaso16_b200 import abi  # noqa: E402
from paper_conf_cgo_margiolaso16_b200.jobs import StencilJob  # noqa: E402
from paper_conf_cgo_margiolaso16_b200.runtime import Accel  # noqa: E402

kernels = sys.argv[1:] or ["stencil_tma", "stencil"]
d = synth.preset("stencil", "default", seed=1)
acc = Accel(0)
flush = torch.empty(64 << 20, dtype=torch.float32, device="cuda")
b = 8 * d["nx"] * d["ny"] * d["nz"]
for kern in kernels:
    job = StencilJob(d, kernel=kern)
    for mode, pol, nm in [(abi.MODE_NATIVE, abi.POLICY_STATIC, "native"), (abi.MODE_SHARED, abi.POLICY_STATIC, "static"),
                          (abi.MODE_SHARED, abi.POLICY_RESOLVE, "resolve")]:
        acc.set_mode(mode, pol)
        ts = []
        for _ in range(8):
            flush.fill_(1)
            torch.cuda.synchronize()
            ids = acc.submit([job], launch_events=True)
            acc.sync()
            lt = acc.launch_times(ids[0], job.launches())
            s = acc.stats(ids[0])
            acc.release()
            ts.append((s.elapsed_ms, statistics.mean(lt), s.quota_initial))
        ts = ts[1:]
        el = statistics.median(t[0] for t in ts)
        per = statistics.median(t[1] for t in ts)
        print(f"{kern} {nm} elapsed_ms {el:.4f} per_launch_us {per * 1e3:.2f} GBps {b / per / 1e6:.0f} "
              f"(request-level {b * d['sweeps'] / el / 1e6:.0f}) quota {ts[-1][2]}", flush=True)
