#!/bin/bash
# Library builds compared on every sharing workload: C2 bench, C4, C3, f2 (300 4-mixes), RESOLVE.
cd "$GRAFT_REPO_ROOT"; mkdir -p gpurun_out/pab
for L in ${LIBS:-default}; do
  if [ "$L" = default ]; then unset ACCEL_LIB; else export ACCEL_LIB=$PWD/$L; fi
  tag=$(basename $L .so)
  timeout 600 python bench.py --no-cpu-baseline --out gpurun_out/pab/bench_$tag.json > gpurun_out/pab/bench_$tag.log 2>&1
  timeout 600 python scripts/mixes.py --config c4 --reps 5 --modes resolve --out gpurun_out/pab/c4_$tag.json > /dev/null 2>&1
  timeout 600 python scripts/mixes.py --config c3 --reps 2 --modes resolve --out gpurun_out/pab/c3_$tag.json > /dev/null 2>&1
  timeout 900 python scripts/mixes.py --config f2 --repeat --k 4 --n 300 --reps 2 --seed 2024 --modes resolve --out gpurun_out/pab/f2_$tag.json > /dev/null 2>&1
  python - <<P
import json
t="$tag"
b=json.load(open(f"gpurun_out/pab/bench_{t}.json")); s=b["sharing"]
c4=json.load(open(f"gpurun_out/pab/c4_{t}.json"))["summary"]["resolve"]
c3=json.load(open(f"gpurun_out/pab/c3_{t}.json"))["summary"]["resolve"]
f2=json.load(open(f"gpurun_out/pab/f2_{t}.json"))["summary"]["resolve"]
print(f"{t:14s} C2 {b['value']:.1f}/s U {s['unfairness_shared']:.2f} STP {s['stp_ratio']:.3f} | C4 U {c4['U']:.2f} STPr {c4['STP_ratio']:.2f} thr {c4['throughput_speedup']:.2f} | C3 U {c3['U_gmean']:.2f} STPr {c3['STP_ratio_gmean']:.3f} thr {c3['throughput_speedup_gmean']:.3f} | f2 U {f2['U_gmean']:.2f} STPr {f2['STP_ratio_gmean']:.3f} thr {f2['throughput_speedup_gmean']:.3f} U<=1.5 {f2['U_le_1.5_pct']:.1f}%")
P
done
