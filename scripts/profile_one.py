"""Run one tenant request (few launches) for ncu:
    python scripts/profile_one.py tenant [native|persistent|resolve] [size] [key=val ...]
(persistent = STATIC policy, resolve = RESOLVE policy)"""
import os
import sys

os.environ.setdefault("CUDA_DEVICE_MAX_CONNECTIONS", "32")
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import synth  # noqa: E402
from paper_conf_cgo_margiolaso16_b200 import abi  # noqa: E402
from paper_conf_cgo_margiolaso16_b200.jobs import make_job  # noqa: E402
from paper_conf_cgo_margiolaso16_b200.runtime import Accel  # noqa: E402

t = sys.argv[1]
mode = abi.MODE_NATIVE if (len(sys.argv) > 2 and sys.argv[2] == "native") else abi.MODE_SHARED
policy = abi.POLICY_RESOLVE if (len(sys.argv) > 2 and sys.argv[2] == "resolve") else abi.POLICY_STATIC
size = sys.argv[3] if len(sys.argv) > 3 else "default"
over = {}
for kv in sys.argv[4:]:
    k, v = kv.split("=")
    over[k] = int(v) if v.isdigit() else float(v)
d = synth.preset(t, size, seed=1, **over)
acc = Accel(0, mode=mode, policy=policy)
job = make_job(t, d)
for _ in range(2):
    acc.run([job])
torch.cuda.synchronize()
acc.close()
print("done", t, sys.argv[2:] if len(sys.argv) > 2 else "")
