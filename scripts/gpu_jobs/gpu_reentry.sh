# re-entry (session 3): GPU suite, bench under each policy, isolated overhead
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv
timeout 1500 python -m pytest tests -m gpu -q -x 2>&1 | tail -5
for p in fair partition resolve; do
  timeout 900 python bench.py --steps 5 --warmup 3 --calib-reps 3 --policy $p --no-cpu-baseline --out gpurun_out/bench_$p.json > gpurun_out/bench_$p.log 2>&1; echo "== $p"; tail -c 300 gpurun_out/bench_$p.log
done
timeout 600 python scripts/isolated.py stencil histo bfs spmv sgemm mriq cutcp tpacf --reps 3 --policy all > gpurun_out/iso.log 2>&1; cut -c1-300 gpurun_out/iso.log
