# final session-4 build (cutcp predicated loop + 56-register cap, tpacf float4 tile + shared RED counters): full GPU suite, default bench line, launch list, isolated overheads, C3/C4/f2 mixes
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv
python -m paper_conf_cgo_margiolaso16_b200.build --force > /dev/null 2>&1
timeout 1500 python -m pytest tests -m gpu -q -x 2>&1 | tail -3
timeout 900 python bench.py --steps 10 --warmup 3 --out gpurun_out/bench_c2.json > gpurun_out/bench_c2.log 2>&1; tail -c 400 gpurun_out/bench_c2.log
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none -c 600 --csv --log-file gpurun_out/launches_c2.csv python bench.py --steps 2 --warmup 1 --calib-reps 1 --no-cpu-baseline > gpurun_out/ncu_launch_bench.log 2>&1
timeout 600 python scripts/isolated.py stencil histo bfs spmv sgemm mriq cutcp tpacf --reps 3 > gpurun_out/isolated.log 2>&1; cut -c1-200 gpurun_out/isolated.log
timeout 600 python scripts/mixes.py --config c3 --reps 3 --modes resolve,static --out gpurun_out/c3.json > gpurun_out/c3.log 2>&1; echo "c3 rc=$?"; grep SUMMARY gpurun_out/c3.log | cut -c1-600
timeout 600 python scripts/mixes.py --config c4 --reps 5 --modes resolve,static --out gpurun_out/c4.json > gpurun_out/c4.log 2>&1; echo "c4 rc=$?"; grep -E "^(native|resolve|static) " gpurun_out/c4.log | cut -c1-160
timeout 600 python scripts/mixes.py --config f2 --k 4 --n 40 --reps 3 --modes resolve,static --out gpurun_out/f2_k4.json > gpurun_out/f2.log 2>&1; echo "f2 rc=$?"; grep SUMMARY gpurun_out/f2.log | cut -c1-600
