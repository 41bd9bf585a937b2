#!/bin/bash
# Iteration check (overwritten per change): GPU suite, per-tenant dispatch
# overhead (NATIVE vs STATIC vs RESOLVE), one bench line.
cd "$GRAFT_REPO_ROOT"; mkdir -p gpurun_out
T=${ITER_TAG:-it}
timeout 1500 python -m pytest tests -m gpu -x -q --timeout 600 -p no:cacheprovider > gpurun_out/${T}_gputest.log 2>&1
echo "pytest rc=$?" >> gpurun_out/${T}_gputest.log
timeout 900 python scripts/isolated.py --reps 8 ${ITER_TENANTS:-stencil spmv lbm sad histo_pipeline cutcp tpacf bfs} > gpurun_out/${T}_isolated.log 2>&1
[ -n "$ITER_TIMELINE" ] && TL_LINES=100 timeout 300 python scripts/timeline.py resolve c2 > gpurun_out/${T}_timeline.log 2>&1
timeout 600 python bench.py --out gpurun_out/${T}_bench.json > gpurun_out/${T}_bench.log 2>&1
echo "bench rc=$?" >> gpurun_out/${T}_bench.log
tail -3 gpurun_out/${T}_gputest.log
python - <<'P'
import json,os
T=os.environ.get("ITER_TAG","it")
for l in open(f"gpurun_out/{T}_isolated.log"):
    if l[:1].isalpha() and "{" in l:
        n,j=l.split(" ",1); j=json.loads(j)
        print(f"{n:15s} static {j.get('overhead',0)*100:+.1f}%  resolve {j.get('overhead_resolve',0)*100:+.1f}%")
P
tail -c 600 gpurun_out/${T}_bench.log
