#!/bin/bash
# kGroup sweep for sgemm_tc1 (rebuild on the box per value)
for g in 8 2 4; do
  ACCEL_NVCC_EXTRA="-DSGEMM1_GROUP=$g" python -m paper_conf_cgo_margiolaso16_b200.build > /dev/null 2>&1
  echo "== group $g"
  python -m pytest tests/test_gpu_sgemm_tc.py -x -q -k "onestep" 2>&1 | tail -1
  python scripts/isolated.py sgemm --reps 5 --policy static 2>&1 | grep -o '"native": {"elapsed_ms": [0-9.]*\|"persistent": {"elapsed_ms": [0-9.]*\|"launch_ms_mean": [0-9.]*'
done > gpurun_out/s1_group.log 2>&1
