# session 3d: footprint-first placement on the sgemm pairs; C3 all pairs; C4 staggered; round profiles
export ACCEL_DEBUG_OFF=1
timeout 900 python scripts/mixes.py --config c3 --reps 3 --modes resolve,static --out gpurun_out/c3_pairs.json > gpurun_out/c3.log 2>&1; tail -25 gpurun_out/c3.log
timeout 600 python scripts/mixes.py --config c4 --reps 5 --modes resolve,static --out gpurun_out/c4.json > gpurun_out/c4.log 2>&1; tail -8 gpurun_out/c4.log
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none -c 800 --csv --log-file gpurun_out/launches_c2.csv python bench.py --steps 2 --warmup 3 --calib-reps 1 --no-cpu-baseline > gpurun_out/ncu_launch_bench.log 2>&1
NCU="timeout 600 ncu --set full --clock-control none --import-source on"
$NCU -k regex:accel_persistent -s 10 -c 1 -o gpurun_out/r1b_stencil_resolve python scripts/profile_one.py stencil resolve default sweeps=12 > /dev/null 2>&1
$NCU -k regex:accel_native -s 10 -c 1 -o gpurun_out/r1b_stencil_native python scripts/profile_one.py stencil native default sweeps=12 > /dev/null 2>&1
$NCU -k regex:accel_persistent -s 1 -c 1 -o gpurun_out/r1b_cutcp_resolve python scripts/profile_one.py cutcp resolve default > /dev/null 2>&1
$NCU -k regex:accel_native -s 1 -c 1 -o gpurun_out/r1b_cutcp_native python scripts/profile_one.py cutcp native default > /dev/null 2>&1
ls gpurun_out/*.ncu-rep
