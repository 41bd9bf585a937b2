#!/bin/bash
cd "$GRAFT_REPO_ROOT"; mkdir -p gpurun_out
N="--kernel-name-base demangled"
ncu --set full --clock-control none --import-source on $N -k regex:"accel_native<accel::StencilT<true, 4>" -s 3 -c 1 -o gpurun_out/r2j_stencil_native -f python scripts/profile_one.py stencil native default sweeps=8 > gpurun_out/r2j_ncu1.log 2>&1
ncu --set full --clock-control none --import-source on $N -k regex:"accel_persistent<accel::StencilT<true, 4>" -s 3 -c 1 -o gpurun_out/r2j_stencil_static -f python scripts/profile_one.py stencil persistent default sweeps=8 > gpurun_out/r2j_ncu2.log 2>&1
ncu --set full --clock-control none --import-source on $N -k regex:"accel_persistent<accel::Tpacf" -c 1 -o gpurun_out/r2j_tpacf_static -f python scripts/profile_one.py tpacf persistent > gpurun_out/r2j_ncu3.log 2>&1
ncu --set full --clock-control none --import-source on $N -k regex:"accel_native<accel::Tpacf" -c 1 -o gpurun_out/r2j_tpacf_native -f python scripts/profile_one.py tpacf native > gpurun_out/r2j_ncu4.log 2>&1
ncu --set full --clock-control none --import-source on $N -k regex:"accel_native<accel::HistoT<true" -s 2 -c 1 -o gpurun_out/r2j_histo_native -f python scripts/profile_one.py histo native default iters=4 > gpurun_out/r2j_ncu5.log 2>&1
ls -la gpurun_out/r2j*.ncu-rep; tail -3 gpurun_out/r2j_ncu1.log
bash scripts/gpu_jobs/r2_f2.sh
