#!/bin/bash
# C4 RESOLVE, many repetitions per library build: the per-rep distribution of U
cd "$GRAFT_REPO_ROOT"; mkdir -p gpurun_out
cat > /tmp/c4many.py <<'P'
import os, sys, statistics, json
sys.path.insert(0, os.environ["GRAFT_REPO_ROOT"]); sys.path.insert(0, os.environ["GRAFT_REPO_ROOT"] + "/scripts")
import numpy as np, torch
import mixes as M
from paper_conf_cgo_margiolaso16_b200 import abi
r = M.Runner(M.TENANTS, "default", torch.device("cuda", 0))
ta = r.isolated(2)
perm = np.random.Generator(np.random.PCG64(7)).permutation(len(M.TENANTS))
order = [M.TENANTS[i] for i in perm]
delta = 0.25 * statistics.median(ta.values()) / 1e3
jobs = [r.jobs[t][0] for t in order]
tal = [ta[t] for t in order]
for mode, pol, name in [(abi.MODE_SHARED, abi.POLICY_RESOLVE, "resolve"), (abi.MODE_SHARED, abi.POLICY_STATIC, "static")]:
    us = []; cut = []
    for rep in range(int(os.environ.get("REPS", 30))):
        m = M.mix_metrics(r.run(jobs, mode, pol, [i * delta for i in range(8)]), tal)
        us.append(m["U"]); cut.append(m["ts_ms"][order.index("cutcp")] / ta["cutcp"])
    us.sort(); cut.sort()
    print(name, "U median %.2f p10 %.2f p90 %.2f max %.2f | cutcp sd median %.2f p90 %.2f | U>9: %d/%d" % (
        statistics.median(us), us[len(us)//10], us[9*len(us)//10], us[-1], statistics.median(cut), cut[9*len(cut)//10],
        sum(u > 9 for u in us), len(us)))
P
for L in ${LIBS:-default}; do
  if [ "$L" = default ]; then unset ACCEL_LIB; else export ACCEL_LIB=$PWD/$L; fi
  echo "== $(basename $L .so)"; timeout 600 python /tmp/c4many.py 2>&1 | tail -2
done
