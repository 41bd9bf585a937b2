"""Per-tenant share profile: isolated SHARED-static time when the solver is
given a fraction f of the device (caps.sms = round(f * SMs): the request gets
the CTAs of f of the SMs, spread over all of them by the hardware, exactly as
a share of a mix is).  Feeds the profile-guided sharing ratios
(paper_conf_cgo_margiolaso16_b200/guided.py, DESIGN.md R-solver-11).

    python scripts/share_profile.py [--out profiles/r2/share_profile.json]
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

TENANTS = ["bfs", "cutcp", "stencil", "tpacf", "histo", "spmv", "sgemm", "mriq"]
FRACS = [1.0, 0.75, 0.5, 0.375, 0.25, 0.1875, 0.125, 0.0625]


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--tenants", default=",".join(TENANTS))
    ap.add_argument("--reps", type=int, default=3)
    ap.add_argument("--out", default=None)
    ap.add_argument("--fracs", default=None, help="comma-separated device fractions (default: the full list)")
    a = ap.parse_args()
    fracs = [float(x) for x in a.fracs.split(",")] if a.fracs else FRACS
    sms = torch.cuda.get_device_properties(0).multi_processor_count
    flush = torch.empty(64 * 1024 * 1024, dtype=torch.float32, device="cuda")
    tenants = a.tenants.split(",")
    inputs = {t: synth.preset(t, "default", seed=11) for t in tenants}
    prof = {t: {} for t in tenants}
    for f in fracs:
        s = max(1, round(f * sms))
        acc = Accel(0, mode=abi.MODE_SHARED, policy=abi.POLICY_STATIC, caps=abi.accel_caps(s, 0, 0, 0, 0))
        for t in tenants:
            job = make_job(t, inputs[t])
            if hasattr(job, "fit_levels"):
                job.fit_levels(acc)
            el, q = [], 0
            for _ in range(a.reps + 1):
                flush.fill_(1)
                torch.cuda.synchronize()
                st = acc.run([job])[0]
                el.append(st.elapsed_ms)
                q = st.quota_initial
            prof[t][f] = {"ms": statistics.median(el[1:]), "quota": q, "sms": s}
            print(t, f, round(prof[t][f]["ms"], 4), q, flush=True)
        acc.close()
    out = {"sms": sms, "fracs": fracs,
           "profile": {t: {"ms": [prof[t][f]["ms"] for f in fracs], "quota": [prof[t][f]["quota"] for f in fracs]}
                       for t in tenants}}
    print(json.dumps(out))
    if a.out:
        json.dump(out, open(a.out, "w"), indent=1)


if __name__ == "__main__":
    main()
