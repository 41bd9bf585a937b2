#!/bin/bash
# evidence refresh: bench (x2, default and stencil_deep), launch list, sgemm tensor-pipe ncu
cd "$GRAFT_REPO_ROOT"; mkdir -p gpurun_out
ncu --query-metrics 2>/dev/null | grep -i "tensor" | head -40 > gpurun_out/r2q_tensor_metrics.txt
timeout 300 python bench.py --steps 10 --warmup 3 --out gpurun_out/r2q_bench.json > gpurun_out/r2q_bench.log 2>&1
ACCEL_STENCIL_KERNEL=stencil_deep timeout 300 python bench.py --steps 10 --warmup 3 --no-cpu-baseline --out gpurun_out/r2q_bench_deep.json > gpurun_out/r2q_bench_deep.log 2>&1
timeout 300 python bench.py --steps 10 --warmup 3 --no-cpu-baseline --out gpurun_out/r2q_bench2.json > gpurun_out/r2q_bench2.log 2>&1
for f in r2q_bench r2q_bench_deep r2q_bench2; do python -c "
import json; b=json.load(open('gpurun_out/$f.json')); print('$f', b['headline'], round(b['roofline']['frac'],3), round(b['value'],1), round(b['e2e']['value'],1))"; done
N="--kernel-name-base demangled"
ncu --set full --clock-control none --import-source on $N -k regex:"accel_persistent<accel::SgemmTc" -c 1 -o gpurun_out/r2q_sgemm_tc -f python scripts/profile_one.py sgemm persistent > gpurun_out/r2q_ncu_sgemm.log 2>&1
ncu --metrics gpu__time_duration.sum --clock-control none -c 1500 --csv --log-file gpurun_out/r2q_launches.csv python bench.py --steps 2 --warmup 1 --no-cpu-baseline --calib-reps 2 > gpurun_out/r2q_ncu_bench.log 2>&1
ls -la gpurun_out/r2q*
