#!/bin/bash
# one-step sgemm: parity + isolated timing of both forms
python -m pytest tests/test_gpu_sgemm_tc.py tests/test_gpu_tenants2.py tests/test_gpu_resolve.py -x -q -k "sgemm" > gpurun_out/s1_tests.log 2>&1
echo "tests rc=$?" >> gpurun_out/s1_tests.log
for os in 1; do
  echo "== ACCEL_SGEMM_ONESTEP=$os"
  ACCEL_SGEMM_ONESTEP=$os python scripts/isolated.py sgemm --reps 5
done > gpurun_out/s1_iso.log 2>&1
ACCEL_SGEMM_ONESTEP=1 ncu --metrics gpu__time_duration.sum --clock-control none -c 40 --csv --log-file gpurun_out/s1_launch.csv python scripts/isolated.py sgemm --reps 1 --policy static > /dev/null 2>&1
