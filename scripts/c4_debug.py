import os, sys, json
sys.path.insert(0, os.environ["GRAFT_REPO_ROOT"]); sys.path.insert(0, os.environ["GRAFT_REPO_ROOT"] + "/scripts")
import torch, statistics
import mixes as M
from paper_conf_cgo_margiolaso16_b200 import abi
r = M.Runner(M.TENANTS, "default", torch.device("cuda", 0))
ta = r.isolated(2)
import numpy as np
perm = np.random.Generator(np.random.PCG64(7)).permutation(len(M.TENANTS))
order = [M.TENANTS[i] for i in perm]
delta = 0.25 * statistics.median(ta.values()) / 1e3
jobs = [r.jobs[t][0] for t in order]
for rep in range(3):
    sys.stderr.write(f"===== rep {rep}\n"); sys.stderr.flush()
    st = r.run(jobs, abi.MODE_SHARED, abi.POLICY_RESOLVE, [i * delta for i in range(8)])
    t0 = min(s.first_start_ns for s in st)
    for t, s in zip(order, st):
        sys.stderr.write(f"   {t:8s} T_s {s.elapsed_ms:7.3f} sd {s.elapsed_ms/ta[t]:5.2f} start {(s.first_start_ns-t0)/1e3:8.1f} end {(s.last_end_ns-t0)/1e3:8.1f} q0 {s.quota_initial} qmin {s.quota_min} qmax {s.quota_max} resolves {s.resolves}\n")
