#!/bin/bash
# C4 (8 staggered arrivals) with several library builds
cd "$GRAFT_REPO_ROOT"; mkdir -p gpurun_out
for L in ${LIBS:-default}; do
  if [ "$L" = default ]; then unset ACCEL_LIB; else export ACCEL_LIB=$PWD/$L; fi
  tag=$(basename $L .so)
  timeout 600 python scripts/mixes.py --config c4 --reps 5 --modes resolve,static --out gpurun_out/c4_$tag.json > gpurun_out/c4_$tag.log 2>&1
  python -c "
import json; d=json.load(open('gpurun_out/c4_$tag.json'))['summary']
for m in ['native','resolve','static']:
    x=d[m]; print('$tag',m,'U %.2f STP %.2f mk %.2f'%(x['U'],x['STP'],x['makespan_ms']), {k:round(v,2) for k,v in x['slowdowns'].items()})"
done
