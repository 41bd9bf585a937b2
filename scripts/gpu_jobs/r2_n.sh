#!/bin/bash
cd "$GRAFT_REPO_ROOT"; mkdir -p gpurun_out
timeout 1800 python -m pytest tests -m gpu -q --timeout 600 -p no:cacheprovider > gpurun_out/r2n_gputest.log 2>&1
echo "pytest rc=$?" >> gpurun_out/r2n_gputest.log; tail -8 gpurun_out/r2n_gputest.log
N="--kernel-name-base demangled"
ncu --set full --clock-control none --import-source on $N -k regex:"accel_native<accel::StencilT<\(bool\)1, \(int\)4" -s 3 -c 1 -o gpurun_out/r2n_stencil_native -f python scripts/profile_one.py stencil native default sweeps=8 > gpurun_out/r2n_ncu1.log 2>&1
ncu --set full --clock-control none --import-source on $N -k regex:"accel_persistent<accel::StencilT<\(bool\)1, \(int\)4" -s 3 -c 1 -o gpurun_out/r2n_stencil_static -f python scripts/profile_one.py stencil persistent default sweeps=8 > gpurun_out/r2n_ncu2.log 2>&1
ncu --set full --clock-control none --import-source on $N -k regex:"accel_native<accel::HistoT<\(bool\)1" -s 2 -c 1 -o gpurun_out/r2n_histo_native -f python scripts/profile_one.py histo native default iters=4 > gpurun_out/r2n_ncu3.log 2>&1
ls gpurun_out/r2n*.ncu-rep; tail -2 gpurun_out/r2n_ncu1.log
