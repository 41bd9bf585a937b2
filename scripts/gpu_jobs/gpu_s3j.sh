# session 3j: suite after the test fix; per-VG trace of stencil / spmv (persistent vs native)
export ACCEL_DEBUG_OFF=1
timeout 1200 python -m pytest tests -m gpu -q > gpurun_out/gpu_suite4.log 2>&1; tail -3 gpurun_out/gpu_suite4.log; grep FAILED gpurun_out/gpu_suite4.log
timeout 300 python scripts/vg_trace.py stencil --policy resolve 2>&1 | tail -14
timeout 300 python scripts/vg_trace.py spmv --policy resolve 2>&1 | tail -14
