# session 3h: new placement-aware solver on the GPU: suite, C2 bench line, C3 pairs, C4, sgemm timeline
export ACCEL_DEBUG_OFF=1
timeout 1200 python -m pytest tests -m gpu -q > gpurun_out/gpu_suite3.log 2>&1; tail -4 gpurun_out/gpu_suite3.log; grep -E "FAILED|Error" gpurun_out/gpu_suite3.log | head -10
timeout 600 python bench.py --steps 10 --warmup 3 --out gpurun_out/bench_c2.json > gpurun_out/bench_c2.log 2>&1; tail -c 200 gpurun_out/bench_c2.log
timeout 900 python scripts/mixes.py --config c3 --reps 3 --modes resolve,static --out gpurun_out/c3_pairs.json > gpurun_out/c3.log 2>&1; grep SUMMARY gpurun_out/c3.log
timeout 600 python scripts/mixes.py --config c4 --reps 5 --modes resolve,static --out gpurun_out/c4.json > gpurun_out/c4.log 2>&1; grep SUMMARY gpurun_out/c4.log | cut -c1-600
timeout 120 python scripts/timeline.py resolve spmv,sgemm 2>&1 | grep -v "launch  *[1-9][0-9]:" | tail -12
