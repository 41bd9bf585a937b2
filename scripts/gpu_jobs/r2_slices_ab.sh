#!/bin/bash
# VG-range slicing of more kernels (ACCEL_SLICES experiment) on f2 (300 4-mixes), C4 and C2
cd "$GRAFT_REPO_ROOT"; mkdir -p gpurun_out/sab
for v in "base:" "cut2:cutcp:2" "cut2tp2:cutcp:2,tpacf:2" "all:cutcp:2,tpacf:2,sgemm_tc1:2,sad_4x4:2"; do
  tag=${v%%:*}; spec=${v#*:}
  if [ -n "$spec" ]; then export ACCEL_SLICES=$spec; else unset ACCEL_SLICES; fi
  timeout 600 python scripts/mixes.py --config f2 --repeat --k 4 --n 300 --reps 2 --seed 2024 --modes resolve --out gpurun_out/sab/f2_$tag.json > /dev/null 2>&1
  timeout 600 python scripts/mixes.py --config c4 --reps 10 --modes resolve --out gpurun_out/sab/c4_$tag.json > /dev/null 2>&1
  timeout 600 python scripts/mixes.py --config c3 --reps 2 --modes resolve --out gpurun_out/sab/c3_$tag.json > /dev/null 2>&1
  python - <<P
import json
t="$tag"
f2=json.load(open(f"gpurun_out/sab/f2_{t}.json"))["summary"]["resolve"]
c4=json.load(open(f"gpurun_out/sab/c4_{t}.json"))["summary"]["resolve"]
c3=json.load(open(f"gpurun_out/sab/c3_{t}.json"))["summary"]["resolve"]
print(f"{t:8s} f2 U {f2['U_gmean']:.2f} STPr {f2['STP_ratio_gmean']:.3f} thr {f2['throughput_speedup_gmean']:.3f} U<=1.5 {f2['U_le_1.5_pct']:.1f}% | C4 U {c4['U']:.2f} STPr {c4['STP_ratio']:.2f} | C3 U {c3['U_gmean']:.2f} STPr {c3['STP_ratio_gmean']:.3f} thr {c3['throughput_speedup_gmean']:.3f}")
P
done
