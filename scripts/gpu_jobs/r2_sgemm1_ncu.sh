#!/bin/bash
# full ncu capture of one sgemm_tc1 launch and of one sgemm_tc launch (persistent)
for os in 1; do
  k=$([ $os = 1 ] && echo 'regex:accel_persistent<accel::SgemmTc1' || echo 'regex:accel_persistent<accel::SgemmTc,')
  ACCEL_SGEMM_ONESTEP=$os timeout 600 ncu --set full --clock-control none --import-source on --kernel-name-base demangled -k "$k" -c 1 -o gpurun_out/s1_full_os$os python scripts/isolated.py sgemm --reps 1 --policy static > gpurun_out/s1_ncu_os$os.log 2>&1
done
