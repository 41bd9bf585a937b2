"""Isolated SHARED-static time of each tenant as its persistent CTAs per SM
are capped (solver caps.ctas_per_sm = c): the occupancy at which a kernel
stops gaining -- what a co-runner can have for free.

    python scripts/occ_scaling.py mriq cutcp tpacf ... [--caps 1,2,3,4,8]
"""
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


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("tenants", nargs="+")
    ap.add_argument("--caps", default="1,2,3,4,6,8,32")
    ap.add_argument("--reps", type=int, default=3)
    a = ap.parse_args()
    flush = torch.empty(64 * 1024 * 1024, dtype=torch.float32, device="cuda")
    out = {}
    for c in [int(x) for x in a.caps.split(",")]:
        caps = abi.accel_caps(0, 0, 0, 0, c)
        acc = Accel(0, mode=abi.MODE_SHARED, policy=abi.POLICY_STATIC, caps=caps)
        for t in a.tenants:
            job = make_job(t, synth.preset(t, "default", seed=1))
            if hasattr(job, "fit_levels"):
                job.fit_levels(acc)
            el = []
            q = 0
            for _ in range(a.reps + 1):
                flush.fill_(1)
                torch.cuda.synchronize()
                s = acc.run([job])[0]
                el.append(s.elapsed_ms)
                q = s.quota_initial
            out.setdefault(t, {})[c] = (statistics.median(el[1:]), q)
        acc.close()
    for t, d in out.items():
        print(t, json.dumps({c: [round(v[0], 3), v[1]] for c, v in d.items()}))


if __name__ == "__main__":
    main()
