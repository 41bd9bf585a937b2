ACCEL_DEBUG=1 timeout 300 python -m pytest tests/test_gpu_resolve.py -x -q -s 2>&1 | tail -30
ACCEL_DEBUG=1 timeout 300 python scripts/timeline.py resolve 2>&1 | tail -40
