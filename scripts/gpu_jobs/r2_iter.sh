#!/bin/bash
# Iteration check (overwritten per change): GPU suite, per-tenant dispatch
# overhead (NATIVE vs STATIC vs RESOLVE), one bench line.
cd "$GRAFT_REPO_ROOT"; mkdir -p gpurun_out
T=${ITER_TAG:-it}
timeout 1500 python -m pytest tests -m gpu -x -q --timeout 600 -p no:cacheprovider > gpurun_out/${T}_gputest.log 2>&1
echo "pytest rc=$?" >> gpurun_out/${T}_gputest.log
timeout 900 python scripts/isolated.py --reps 8 ${ITER_TENANTS:-stencil spmv lbm sad histo_pipeline cutcp tpacf bfs} > gpurun_out/${T}_isolated.log 2>&1
[ -n "$ITER_MIXDIAG" ] && timeout 600 python scripts/mixdiag.py $ITER_MIXDIAG > gpurun_out/${T}_mixdiag.log 2>&1
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
        print(f"{n:15s} static {j.get('overhead',0)*100:+.1f}%  resolve {j.get('overhead_resolve',0)*100:+.1f}%  launch us nat {j['native']['launch_ms_mean']*1e3:.1f} st {j['persistent']['launch_ms_mean']*1e3:.1f} rs {j['persistent_resolve']['launch_ms_mean']*1e3:.1f}")
P
[ -n "$ITER_MIXDIAG" ] && grep -A6 "resolve\|native" gpurun_out/${T}_mixdiag.log | grep "==\|slowdown\|U " | head -40
python -c "
import json; d=json.load(open('gpurun_out/${T}_bench.json')); s=d['sharing']
print(round(d['value'],1), 'native', round(s['native_mixes_per_s'],1), 'U', round(s['unfairness_shared'],3), 'STP', round(s['stp_ratio'],3), {k: round(v,2) for k,v in s['T_s_ms_shared'].items()}, 'frac', round(d['roofline']['frac'],3))"
