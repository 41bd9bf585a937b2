#!/bin/bash
# A/B: the working-tree library vs ab/libaccel_head.so (the last commit) on
# the C2 timeline (ACCEL_DEBUG re-solve stamps) and the bench line.
cd "$GRAFT_REPO_ROOT"; mkdir -p gpurun_out
T=${ITER_TAG:-ab}
for v in new head; do
  if [ $v = head ]; then export ACCEL_LIB=$PWD/ab/libaccel_head.so; else unset ACCEL_LIB; fi
  ACCEL_DEBUG=1 TL_LINES=100 timeout 300 python scripts/timeline.py resolve c2 > gpurun_out/${T}_timeline_$v.log 2>&1
  timeout 600 python bench.py --no-cpu-baseline --out gpurun_out/${T}_bench_$v.json > gpurun_out/${T}_bench_$v.log 2>&1
  echo "$v bench rc=$?"
  python -c "
import json; d=json.load(open('gpurun_out/${T}_bench_$v.json')); s=d['sharing']
print('$v', round(d['value'],1), 'U', round(s['unfairness_shared'],3), 'STP', round(s['stp_ratio'],3), {k: round(v,2) for k,v in s['T_s_ms_shared'].items()})"
done
