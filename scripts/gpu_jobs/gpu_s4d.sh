# stencil mbarrier pipeline (STENCIL_MBAR=1) vs the barrier-per-plane default: parity + isolated timing
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv
for mb in 1 0; do
  ACCEL_NVCC_EXTRA="-DSTENCIL_MBAR=$mb" python -m paper_conf_cgo_margiolaso16_b200.build --force > /dev/null 2>&1 || echo "build fail mbar=$mb"
  echo "mbar=$mb"
  timeout 600 python -m pytest tests -m gpu -q -x -k "stencil or config1 or mix or resolve" 2>&1 | tail -2
  timeout 120 python scripts/isolated.py stencil --reps 5 2>&1 | cut -c1-700
done
ACCEL_NVCC_EXTRA="-DSTENCIL_MBAR=1" python -m paper_conf_cgo_margiolaso16_b200.build --force > /dev/null 2>&1
timeout 300 ncu --set full --clock-control none --import-source on -k regex:accel_persistent -s 10 -c 1 -o gpurun_out/s4d_stencil_mbar_static python scripts/profile_one.py stencil persistent default sweeps=12 > /dev/null 2>&1
