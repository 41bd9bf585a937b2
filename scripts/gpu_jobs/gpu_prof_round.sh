# round evidence: bench line, ncu launch list of a short bench run, full ncu of the key kernels
timeout 900 python bench.py --steps 10 --warmup 3 --out gpurun_out/bench_c2.json > gpurun_out/bench_c2.log 2>&1
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none -c 800 --csv --log-file gpurun_out/launches_c2.csv python bench.py --steps 2 --warmup 1 --calib-reps 1 --no-cpu-baseline > gpurun_out/ncu_launch_bench.log 2>&1
NCU="timeout 600 ncu --set full --clock-control none --import-source on"
$NCU -k regex:accel_persistent -s 10 -c 1 -o gpurun_out/r1_stencil_resolve python scripts/profile_one.py stencil resolve default sweeps=12 > /dev/null 2>&1
$NCU -k regex:accel_persistent -s 10 -c 1 -o gpurun_out/r1_stencil_static python scripts/profile_one.py stencil persistent default sweeps=12 > /dev/null 2>&1
$NCU -k regex:accel_native -s 10 -c 1 -o gpurun_out/r1_stencil_native python scripts/profile_one.py stencil native default sweeps=12 > /dev/null 2>&1
$NCU -k regex:accel_persistent -s 1 -c 1 -o gpurun_out/r1_cutcp_static python scripts/profile_one.py cutcp persistent default > /dev/null 2>&1
$NCU -k regex:accel_persistent -s 1 -c 1 -o gpurun_out/r1_tpacf_static python scripts/profile_one.py tpacf persistent default > /dev/null 2>&1
$NCU -k regex:"accel_persistent<accel::SgemmTc" -s 1 -c 1 -o gpurun_out/r1_sgemmtc_static python scripts/profile_one.py sgemm persistent default > /dev/null 2>&1
$NCU -k regex:accel_persistent -s 4 -c 1 -o gpurun_out/r1_histo_static python scripts/profile_one.py histo persistent default > /dev/null 2>&1
ls -la gpurun_out/ | tail -12
tail -c 1500 gpurun_out/bench_c2.log
