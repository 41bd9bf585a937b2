#!/bin/bash
cd "$GRAFT_REPO_ROOT"; mkdir -p gpurun_out
echo "== global maps"; timeout 600 python scripts/diag_tma.py --reps 2 --sweeps 40 --global-maps --combos=-,bfs 2>&1 | tee gpurun_out/r2g_diag_gmaps.log
echo "== cp.async control"; timeout 600 python scripts/diag_tma.py --reps 2 --sweeps 40 --kernel stencil --combos=-,bfs,bfs+cutcp+tpacf 2>&1 | tee gpurun_out/r2g_diag_cpasync.log
echo "== intercept"; timeout 600 python -m pytest tests/test_gpu_intercept.py -q -x -p no:cacheprovider 2>&1 | tail -30 | tee gpurun_out/r2g_intercept.log
ACCEL_INTERCEPT_VERBOSE=1 LD_PRELOAD=$PWD/paper_conf_cgo_margiolaso16_b200/libaccel_intercept.so ./examples/intercept_app 2>&1 | tail -12 | tee -a gpurun_out/r2g_intercept.log
timeout 1500 python -m pytest tests -m gpu -x -q --timeout 600 -p no:cacheprovider > gpurun_out/r2g_gputest.log 2>&1
echo "pytest rc=$?" >> gpurun_out/r2g_gputest.log; tail -5 gpurun_out/r2g_gputest.log
timeout 300 python bench.py --steps 10 --warmup 3 > gpurun_out/r2g_bench.log 2>&1
tail -c 700 gpurun_out/r2g_bench.log
