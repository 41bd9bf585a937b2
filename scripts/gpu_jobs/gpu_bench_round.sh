# round evidence: bench line, ncu launch list of a short bench run, full ncu of the dominant kernel
timeout 900 python bench.py --steps 10 --warmup 3 --out gpurun_out/bench_c2.json > gpurun_out/bench_c2.log 2>&1
ncu --metrics gpu__time_duration.sum --clock-control none -c 600 --csv --log-file gpurun_out/launches_c2.csv python bench.py --steps 2 --warmup 1 --calib-reps 1 --no-cpu-baseline > gpurun_out/ncu_launch_bench.log 2>&1
ncu --set full --clock-control none --import-source on -k regex:accel_persistent -s 10 -c 1 -o gpurun_out/stencil_persist_r1 python scripts/profile_one.py stencil persistent default sweeps=12 > /dev/null 2>&1
ncu --set full --clock-control none --import-source on -k regex:accel_native -s 10 -c 1 -o gpurun_out/stencil_native_r1 python scripts/profile_one.py stencil native default sweeps=12 > /dev/null 2>&1
tail -c 3000 gpurun_out/bench_c2.log
