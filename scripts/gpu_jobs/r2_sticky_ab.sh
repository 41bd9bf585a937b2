#!/bin/bash
# ACCEL_STICKY_MAIN experiment: one long-lived grid per multi-launch main step (RESOLVE)
cd "$GRAFT_REPO_ROOT"; mkdir -p gpurun_out/sticky
ACCEL_STICKY_MAIN=1 timeout 900 python -m pytest tests -m gpu -q -x -p no:cacheprovider 2>&1 | tail -2
for v in base sticky; do
  if [ $v = sticky ]; then export ACCEL_STICKY_MAIN=1; else unset ACCEL_STICKY_MAIN; fi
  echo "=== $v"
  timeout 300 python scripts/isolated.py --reps 8 --policy resolve stencil spmv lbm bfs histo 2>&1 | python -c "
import json,sys
for l in sys.stdin:
    if l[:1].isalpha() and '{' in l:
        n,j=l.split(' ',1); j=json.loads(j); print(n, 'native %.3f resolve %+.1f%%' % (j['native']['elapsed_ms'], j['overhead_resolve']*100))"
  timeout 300 python scripts/mixdiag.py bfs,cutcp,stencil,tpacf 2>&1 | grep -A6 "resolve" | grep "slowdown\|U "
  timeout 900 python scripts/mixes.py --config f2 --repeat --k 4 --n 300 --reps 2 --seed 2024 --modes resolve --out gpurun_out/sticky/f2_$v.json > /dev/null 2>&1
  timeout 600 python scripts/mixes.py --config c4 --reps 10 --modes resolve --out gpurun_out/sticky/c4_$v.json > /dev/null 2>&1
  timeout 600 python scripts/mixes.py --config c3 --reps 2 --modes resolve --out gpurun_out/sticky/c3_$v.json > /dev/null 2>&1
  python - <<P
import json
t="$v"
f2=json.load(open(f"gpurun_out/sticky/f2_{t}.json"))["summary"]["resolve"]
c4=json.load(open(f"gpurun_out/sticky/c4_{t}.json"))["summary"]["resolve"]
c3=json.load(open(f"gpurun_out/sticky/c3_{t}.json"))["summary"]["resolve"]
print(f"{t:8s} f2 U {f2['U_gmean']:.2f} STPr {f2['STP_ratio_gmean']:.3f} thr {f2['throughput_speedup_gmean']:.3f} U<=1.5 {f2['U_le_1.5_pct']:.1f}% | C4 U {c4['U']:.2f} STPr {c4['STP_ratio']:.2f} thr {c4['throughput_speedup']:.2f} | C3 U {c3['U_gmean']:.2f} STPr {c3['STP_ratio_gmean']:.3f} thr {c3['throughput_speedup_gmean']:.3f}")
P
done
