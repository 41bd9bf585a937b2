# session 3e: where does the default bench stall?  (unbuffered, stack dumps)
export ACCEL_DEBUG_OFF=1
ACCEL_DEBUG=1 timeout 300 python -u bench.py --steps 3 --warmup 3 --calib-reps 2 --no-cpu-baseline --hang-dump-s 100 > gpurun_out/bench_dbg.log 2>&1; echo "rc=$?"
grep -v "^\[accel\] resolve req" gpurun_out/bench_dbg.log | tail -c 6000
grep -c "" gpurun_out/bench_dbg.log
