timeout 1200 python -m pytest tests -m gpu -q -x 2>&1 | tail -3
for i in 1 2; do timeout 300 python -m pytest tests/test_gpu_resolve.py -q -x 2>&1 | tail -1; done
python scripts/isolated.py stencil --reps 3 2>&1 | tail -1
for kd in 2 4 5; do ACCEL_NVCC_EXTRA=-DSTENCIL_KD=$kd python -m paper_conf_cgo_margiolaso16_b200.build --force 2>&1 | grep -c error; echo KD $kd; python scripts/isolated.py stencil --reps 3 2>&1 | tail -1; done
