"""Multi-process host logic of the N > 1 bench path on CPU (gloo, world size 2):
the real bench.main self-spawns its ranks (`--gpus 2`, no torchrun), each rank
runs the per-rank leg with the device work stubbed (ACCEL_BENCH_STUB), the
ranks barrier and gather over gloo, and rank 0 prints ONE line with the
max-over-ranks time and the whole-job value (PAPER.md has one accelerator per
platform, lines 844-852; BASELINE config 5: independent mixes per GPU)."""
import json
import os
import subprocess
import sys

import pytest

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def _run(args, extra_env=None):
    env = dict(os.environ, ACCEL_BENCH_STUB="1")
    env.pop("WORLD_SIZE", None)
    env.update(extra_env or {})
    p = subprocess.run([sys.executable, os.path.join(ROOT, "bench.py"), *args], env=env, cwd=ROOT,
                       capture_output=True, text=True, timeout=240)
    assert p.returncode == 0, p.stderr[-3000:]
    lines = [ln for ln in p.stdout.splitlines() if ln.startswith("{")]
    assert len(lines) == 1, p.stdout   # rank 0 alone prints
    return json.loads(lines[0])


@pytest.mark.timeout(300)
def test_bench_self_spawns_two_ranks_c5():
    line = _run(["--gpus", "2", "--config", "c5", "--steps", "5", "--warmup", "3", "--no-cpu-baseline"])
    assert line["n_gpus"] == 2
    mixes = line["config"]["tenants"]
    assert len(mixes) == 2 and mixes[0] != mixes[1]            # independent mixes per GPU
    assert all(len(set(m)) == 4 for m in mixes)
    # stub device time of rank r = 10 * steps + r ms: the slowest rank sets the time
    assert line["ms_per_step"] == pytest.approx((50.0 + 1) / 5)
    assert line["value"] == pytest.approx(2 * 5 / 0.051)       # all mixes / slowest rank
    assert line["sharing"]["unfairness_shared"] == pytest.approx((1.2 * 1.3) ** 0.5)
    assert [r["rank"] for r in line["sharing"]["per_rank"]] == [0, 1]
    assert list(line)[-1] == "headline"                        # compact summary is the tail


@pytest.mark.timeout(300)
def test_bench_one_rank_equals_plain_run():
    """--gpus 1 takes no spawn path and reports n_gpus 1."""
    line = _run(["--gpus", "1", "--steps", "4", "--warmup", "3", "--no-cpu-baseline"])
    assert line["n_gpus"] == 1
    assert line["ms_per_step"] == pytest.approx(10.0)
    assert line["headline"]["targets"]["U<=1.5"] is True


def test_aggregate_max_over_ranks():
    sys.path.insert(0, ROOT)
    import bench
    mk = lambda u, d: {"rank": 0, "dev_ms": d, "e2e_ms": d, "nat_ms": 15.0, "oth_ms": {"static": 11.0},  # noqa: E731
                       "sh": {"U": [u], "STP": [2.0], "ANTT": [2.0]}, "na": {"U": [4.0], "STP": [1.5], "ANTT": [3.0]},
                       "ot": {"static": {"U": [2.0], "STP": [1.8], "ANTT": [2.5]}}}
    agg = bench.aggregate([mk(1.5, 10.0), mk(2.5, 11.0)], 2, 5, "resolve")
    assert agg["tmax"] == 11.0
    assert agg["value"] == pytest.approx(2 * 5 / 0.011)
    assert agg["U_sh"] == pytest.approx((1.5 * 2.5) ** 0.5)
    assert agg["other"]["static"]["throughput_speedup"] == pytest.approx(15.0 / 11.0)
