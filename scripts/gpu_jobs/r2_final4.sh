#!/bin/bash
# Round-2 final evidence, session 3 build, cutcp row gather, 4-A cells, share profile refreshed: GPU suite, isolated overheads
# (tuned + naive chunk 1 + tiny grids), bench line, f2 (paper shape), C3, C4,
# bench launch list and one --set full capture of the dominant kernel.
cd "$GRAFT_REPO_ROOT"; mkdir -p gpurun_out
O=gpurun_out/fin4
mkdir -p $O
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv > $O/smi.txt 2>&1
timeout 900 python -m pytest tests -m gpu -q --timeout 600 -p no:cacheprovider > $O/gputest.log 2>&1; echo "pytest rc=$?" >> $O/gputest.log
timeout 500 python scripts/share_profile.py --out profiles/r2/share_profile.json > $O/share_profile.log 2>&1; cp profiles/r2/share_profile.json $O/share_profile.json
timeout 900 python scripts/isolated.py --reps 8 bfs cutcp stencil tpacf histo spmv sgemm mriq sad lbm gridding histo_pipeline > $O/isolated.log 2>&1
timeout 600 python scripts/cutcp_cell.py --cells 4,2,1 > $O/cutcp_cell.log 2>&1
timeout 600 python scripts/isolated.py --reps 5 --chunk 1 bfs cutcp stencil tpacf histo spmv sgemm mriq > $O/isolated_naive_chunk1.log 2>&1
timeout 600 python bench.py --out $O/bench_c2.json > $O/bench_c2.log 2>&1; echo "bench rc=$?" >> $O/bench_c2.log
timeout 900 python bench.py --impl reference --steps 3 --warmup 3 > $O/bench_reference.log 2>&1; echo "ref rc=$?" >> $O/bench_reference.log
timeout 2400 python scripts/mixes.py --config f2 --repeat --k 4 --n 1000 --reps 2 --seed 2024 --out $O/f2_k4_1000.json > $O/f2_k4_1000.log 2>&1
timeout 1800 python scripts/mixes.py --config f2 --repeat --k 8 --n 500 --reps 2 --seed 2025 --out $O/f2_k8_500.json > $O/f2_k8_500.log 2>&1
timeout 900 python scripts/mixes.py --config c3 --reps 3 --out $O/c3.json > $O/c3.log 2>&1
timeout 900 python scripts/mixes.py --config c4 --reps 20 --out $O/c4.json > $O/c4.log 2>&1
timeout 300 python scripts/starve.py mriq cutcp 1.0 > $O/starve_mriq_cutcp.log 2>&1
timeout 300 python scripts/starve.py mriq tpacf 1.0 > $O/starve_mriq_tpacf.log 2>&1
N="--kernel-name-base demangled"
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none -c 1500 --csv --log-file $O/launches_c2.csv python bench.py --steps 2 --warmup 1 --no-cpu-baseline --calib-reps 2 > $O/ncu_bench.log 2>&1
timeout 900 ncu --set full --clock-control none --import-source on $N -k 'regex:accel_persistent<accel::StencilT' -s 20 -c 1 -o $O/stencil_resolve -f python scripts/isolated.py stencil --reps 1 --policy resolve > $O/ncu_stencil.log 2>&1
ls -la $O
tail -2 $O/gputest.log; tail -c 400 $O/bench_c2.log
