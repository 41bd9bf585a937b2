NCU="ncu --set full --clock-control none --import-source on"
$NCU -k regex:accel_native -s 4 -c 1 -o gpurun_out/stencil_n5 python scripts/profile_one.py stencil native default sweeps=8 > /dev/null 2>&1
$NCU -k regex:accel_persistent -s 4 -c 1 -o gpurun_out/stencil_p5 python scripts/profile_one.py stencil persistent default sweeps=8 > /dev/null 2>&1
$NCU -k regex:accel_native -s 1 -c 1 -o gpurun_out/cutcp_n5 python scripts/profile_one.py cutcp native default > /dev/null 2>&1
$NCU -k regex:accel_persistent -s 1 -c 1 -o gpurun_out/cutcp_p5 python scripts/profile_one.py cutcp persistent default > /dev/null 2>&1
ls -la gpurun_out/
