# re-entry session 4 evidence: full GPU parity suite, default bench line, launch list, single-tenant dispatch overhead
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv
python -m paper_conf_cgo_margiolaso16_b200.build > /dev/null 2>&1
timeout 1500 python -m pytest tests -m gpu -q -x 2>&1 | tail -3
timeout 900 python bench.py --steps 10 --warmup 3 --out gpurun_out/bench_c2.json > gpurun_out/bench_c2.log 2>&1; tail -c 600 gpurun_out/bench_c2.log
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none -c 600 --csv --log-file gpurun_out/launches_c2.csv python bench.py --steps 2 --warmup 1 --calib-reps 1 --no-cpu-baseline > gpurun_out/ncu_launch_bench.log 2>&1
timeout 600 python scripts/isolated.py stencil histo bfs spmv sgemm mriq cutcp tpacf --reps 3 > gpurun_out/isolated.log 2>&1; cut -c1-300 gpurun_out/isolated.log
