#!/bin/bash
# Final round-2 evidence (code frozen): isolated overheads, f2 (paper shape),
# c3, c4, bench, bench launch list, sgemm_tc1 / stencil ncu captures.
cd "$GRAFT_REPO_ROOT"; mkdir -p gpurun_out
timeout 900 python scripts/isolated.py --reps 8 bfs cutcp stencil tpacf histo spmv sgemm mriq sad lbm gridding histo_pipeline > gpurun_out/fz_isolated.log 2>&1
timeout 300 python scripts/isolated.py --reps 5 --chunk 1 bfs cutcp stencil tpacf histo spmv sgemm mriq > gpurun_out/fz_isolated_naive.log 2>&1
timeout 2400 python scripts/mixes.py --config f2 --repeat --k 4 --n 1000 --reps 2 --seed 2024 --out gpurun_out/fz_f2_k4.json > gpurun_out/fz_f2_k4.log 2>&1
timeout 1800 python scripts/mixes.py --config f2 --repeat --k 8 --n 500 --reps 2 --seed 2025 --out gpurun_out/fz_f2_k8.json > gpurun_out/fz_f2_k8.log 2>&1
timeout 900 python scripts/mixes.py --config c3 --reps 3 --out gpurun_out/fz_c3.json > gpurun_out/fz_c3.log 2>&1
timeout 600 python scripts/mixes.py --config c4 --reps 5 --out gpurun_out/fz_c4.json > gpurun_out/fz_c4.log 2>&1
timeout 600 python bench.py --out gpurun_out/fz_bench.json > gpurun_out/fz_bench.log 2>&1
N="--kernel-name-base demangled"
ncu --metrics gpu__time_duration.sum --clock-control none -c 1500 --csv --log-file gpurun_out/fz_launches.csv python bench.py --steps 2 --warmup 1 --no-cpu-baseline --calib-reps 2 > gpurun_out/fz_ncu_bench.log 2>&1
ncu --set full --clock-control none --import-source on $N -k 'regex:accel_persistent<accel::SgemmTc1' -c 1 -o gpurun_out/fz_sgemm_tc1 -f python scripts/isolated.py sgemm --reps 1 --policy static > gpurun_out/fz_ncu_sgemm.log 2>&1
ls -la gpurun_out/fz*
