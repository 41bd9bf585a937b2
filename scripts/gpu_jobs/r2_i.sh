#!/bin/bash
cd "$GRAFT_REPO_ROOT"; mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_tenants.py tests/test_gpu_order.py -k "tpacf or order" -q -x --timeout 300 -p no:cacheprovider 2>&1 | tail -3
for q in 1 2 4; do echo "== qsplit $q"; ACCEL_TPACF_QSPLIT=$q timeout 300 python scripts/isolated.py --reps 8 tpacf 2>&1 | cut -c 1-400; done | tee gpurun_out/r2i_tpacf.log
ncu --set full --clock-control none --import-source on -k regex:"accel_native.*StencilTILb1ELi4" -s 3 -c 1 -o gpurun_out/r2i_stencil_native -f python scripts/profile_one.py stencil native default sweeps=8 > gpurun_out/r2i_ncu1.log 2>&1
ncu --set full --clock-control none --import-source on -k regex:"accel_persistent.*StencilTILb1ELi4" -s 3 -c 1 -o gpurun_out/r2i_stencil_static -f python scripts/profile_one.py stencil persistent default sweeps=8 > gpurun_out/r2i_ncu2.log 2>&1
ncu --set full --clock-control none --import-source on -k regex:"accel_persistent.*Tpacf" -c 1 -o gpurun_out/r2i_tpacf_static -f python scripts/profile_one.py tpacf persistent > gpurun_out/r2i_ncu3.log 2>&1
ls -la gpurun_out/*.ncu-rep
