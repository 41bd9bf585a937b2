# session 3s: GEMM pre-placed ahead of its split steps (R-place-3)
export ACCEL_DEBUG_OFF=1 ACCEL_SYNC_TIMEOUT_S=60
timeout 1200 python -m pytest tests -m gpu -q > gpurun_out/gpu_suite10.log 2>&1; tail -2 gpurun_out/gpu_suite10.log; grep -E "FAILED|STUCK" gpurun_out/gpu_suite10.log | head
for mix in spmv,sgemm cutcp,sgemm,spmv,histo tpacf,bfs,sgemm,spmv; do echo "== $mix"; timeout 120 python scripts/timeline.py resolve $mix 2>&1 | grep "T(s)"; done
timeout 900 python scripts/mixes.py --config f2 --k 4 --n 40 --reps 3 --modes resolve,static --out gpurun_out/f2_k4.json > gpurun_out/f2.log 2>&1; grep SUMMARY gpurun_out/f2.log
timeout 900 python scripts/mixes.py --config c3 --reps 3 --modes resolve,static --out gpurun_out/c3_pairs.json > gpurun_out/c3.log 2>&1; grep SUMMARY gpurun_out/c3.log | cut -c1-400
