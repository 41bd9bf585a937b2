set -x
ACCEL_DEBUG=1 timeout 300 python -m pytest tests/test_gpu_resolve.py -x -q -s 2>&1 | tail -30
for m in native static resolve; do ACCEL_DEBUG=1 timeout 300 python scripts/timeline.py $m 2>&1 | tail -70; done
