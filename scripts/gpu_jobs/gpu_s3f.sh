# session 3f: reproduce the intermittent bench stall with the sync watchdog
export ACCEL_SYNC_TIMEOUT_S=20
for i in 1 2 3 4 5 6 7 8; do
  timeout 150 python -u bench.py --steps 5 --warmup 3 --calib-reps 3 --no-cpu-baseline --hang-dump-s 120 > gpurun_out/bench_loop_$i.log 2>&1
  rc=$?; echo "run $i rc=$rc $(grep -c STUCK gpurun_out/bench_loop_$i.log) stuck-lines"
  if [ $rc -ne 0 ]; then grep -v "^\s*$" gpurun_out/bench_loop_$i.log | grep -v "site-packages" | tail -60; break; fi
done
timeout 900 python -m pytest tests -m gpu -q -x > gpurun_out/gpu_suite2.log 2>&1; tail -5 gpurun_out/gpu_suite2.log; grep -B2 -A30 STUCK gpurun_out/gpu_suite2.log | head -60
