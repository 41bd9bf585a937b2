NCU="ncu --set full --clock-control none --import-source on"
$NCU -k regex:accel_native -s 1 -c 1 -o gpurun_out/tpacf_n2 python scripts/profile_one.py tpacf native default > /dev/null 2>&1
$NCU -k regex:accel_persistent -s 1 -c 1 -o gpurun_out/tpacf_p2 python scripts/profile_one.py tpacf persistent default > /dev/null 2>&1
