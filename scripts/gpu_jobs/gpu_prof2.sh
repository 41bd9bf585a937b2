NCU="ncu --set full --clock-control none --import-source on"
$NCU -k regex:accel_native -s 3 -c 1 -o gpurun_out/spmv_native python scripts/profile_one.py spmv native default iters=4 > /dev/null 2>&1
$NCU -k regex:accel_persistent -s 3 -c 1 -o gpurun_out/spmv_persist python scripts/profile_one.py spmv persistent default iters=4 > /dev/null 2>&1
$NCU -k regex:accel_native -s 3 -c 1 -o gpurun_out/stencil2_native python scripts/profile_one.py stencil native default sweeps=4 > /dev/null 2>&1
$NCU -k regex:accel_persistent -s 3 -c 1 -o gpurun_out/stencil2_persist python scripts/profile_one.py stencil persistent default sweeps=4 > /dev/null 2>&1
$NCU -k regex:accel_native -s 1 -c 1 -o gpurun_out/tpacf_native python scripts/profile_one.py tpacf native default > /dev/null 2>&1
$NCU -k regex:accel_native -s 1 -c 1 -o gpurun_out/cutcp_native python scripts/profile_one.py cutcp native default > /dev/null 2>&1
ls gpurun_out
