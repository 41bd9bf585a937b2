"""histo_wide at the SURVEY default (2^24 u32 samples, 16,384 bins, 100
passes): isolated per-pass time for several VG sizes (samples per VG), NATIVE
and SHARED-STATIC; algorithmic bytes = 4 B/sample + 4 B/bin per pass."""
import os
import statistics
import sys

os.environ.setdefault("CUDA_DEVICE_MAX_CONNECTIONS", "32")
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import synth  # noqa: E402
from paper_conf_cgo_margiolaso16_b200 import abi  # noqa: E402
from paper_conf_cgo_margiolaso16_b200.jobs import HistoJob  # noqa: E402
from paper_conf_cgo_margiolaso16_b200.runtime import Accel  # noqa: E402

d0 = synth.preset("histo", "default", seed=1)
acc = Accel(0)
flush = torch.empty(64 << 20, dtype=torch.float32, device="cuda")
b = 4 * d0["n"] + 4 * d0["bins"]
for per_vg in [int(x) for x in (sys.argv[1:] or ["16384", "32768", "61440"])]:
    job = HistoJob(dict(d0, per_vg=per_vg))
    for mode, pol, nm in [(abi.MODE_NATIVE, abi.POLICY_STATIC, "native"), (abi.MODE_SHARED, abi.POLICY_STATIC, "static"),
                          (abi.MODE_SHARED, abi.POLICY_RESOLVE, "resolve")]:
        acc.set_mode(mode, pol)
        ts = []
        for _ in range(6):
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
        print(f"per_vg {per_vg} VGs {job.steps[0].grid[0]} {nm} elapsed_ms {el:.3f} per_pass_us {per * 1e3:.1f} "
              f"GBps {b / per / 1e6:.0f} quota {ts[-1][2]}", flush=True)
