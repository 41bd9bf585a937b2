NCU="ncu --set full --clock-control none --import-source on"
$NCU -k regex:accel_persistent -s 3 -c 1 -o gpurun_out/spmv_persist2 python scripts/profile_one.py spmv persistent default iters=4 > /dev/null 2>&1
ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/launches_spmv.csv python scripts/profile_one.py spmv persistent default iters=6 > /dev/null 2>&1
ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/launches_spmv_n.csv python scripts/profile_one.py spmv native default iters=6 > /dev/null 2>&1
