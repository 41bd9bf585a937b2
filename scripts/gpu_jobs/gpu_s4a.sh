# stencil tile-depth / planes-in-flight sweep (isolated, default 512x512x64, 100 sweeps) + ncu source capture of the current kernel
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv
mkdir -p gpurun_out
timeout 300 ncu --set full --clock-control none --import-source on -k regex:accel_persistent -s 10 -c 1 -o gpurun_out/s4_stencil_static python scripts/profile_one.py stencil persistent default sweeps=12 > /dev/null 2>&1
cp paper_conf_cgo_margiolaso16_b200/csrc/tenants/stencil.cuh /tmp/st.cuh; cp paper_conf_cgo_margiolaso16_b200/jobs.py /tmp/jobs.py
for tz in 8 16 4; do for kd in 2 3 4 6; do
  cp /tmp/st.cuh paper_conf_cgo_margiolaso16_b200/csrc/tenants/stencil.cuh; cp /tmp/jobs.py paper_conf_cgo_margiolaso16_b200/jobs.py
  sed -i "s/kTY = 8, kTZ = 8;/kTY = 8, kTZ = $tz;/" paper_conf_cgo_margiolaso16_b200/csrc/tenants/stencil.cuh
  sed -i "s/TX, TY, TZ = 128, 8, 8/TX, TY, TZ = 128, 8, $tz/" paper_conf_cgo_margiolaso16_b200/jobs.py
  ACCEL_NVCC_EXTRA="-DSTENCIL_KD=$kd" python -m paper_conf_cgo_margiolaso16_b200.build --force > /dev/null 2>&1 || { echo "build fail tz=$tz kd=$kd"; continue; }
  echo "tz=$tz kd=$kd"; timeout 120 python scripts/isolated.py stencil --reps 3 2>&1 | cut -c1-420
done; done
