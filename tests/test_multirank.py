"""Multi-process host logic of the N > 1 bench path on CPU (gloo, world size 2):
independent per-rank mixes, gather of per-rank results, max-over-ranks time."""
import os
import socket

import pytest
import torch.distributed as dist
import torch.multiprocessing as mp


def _port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def _worker(rank, world, port, q):
    os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port), RANK=str(rank), WORLD_SIZE=str(world))
    dist.init_process_group("gloo", rank=rank, world_size=world)
    import bench
    mix = bench.c5_mix(rank)
    res = {"rank": rank, "dev_ms": 10.0 + rank, "e2e_ms": 12.0 + rank, "nat_ms": 15.0, "oth_ms": {"resolve": 11.0},
           "tenants": mix, "sh": {"U": [1.5 + rank], "STP": [2.0], "ANTT": [2.0]},
           "na": {"U": [4.0], "STP": [1.5], "ANTT": [3.0]}, "ot": {"resolve": {"U": [2.0], "STP": [1.8], "ANTT": [2.5]}}}
    allres = [None] * world
    dist.all_gather_object(allres, res)
    dist.barrier()
    if rank == 0:
        q.put((allres, bench.aggregate(allres, world, 5, "partition")))
    dist.destroy_process_group()


@pytest.mark.timeout(120)
def test_two_rank_aggregation():
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _port()
    procs = [ctx.Process(target=_worker, args=(r, 2, port, q)) for r in range(2)]
    for p in procs:
        p.start()
    allres, agg = q.get(timeout=100)
    for p in procs:
        p.join(timeout=60)
        assert p.exitcode == 0
    assert [r["rank"] for r in allres] == [0, 1]
    assert allres[0]["tenants"] != allres[1]["tenants"]          # independent mixes (config 5)
    assert len(set(allres[0]["tenants"])) == 4
    assert agg["tmax"] == 11.0                                     # max over ranks
    assert agg["value"] == pytest.approx(2 * 5 / 0.011)           # all mixes / slowest rank
    assert agg["U_sh"] == pytest.approx((1.5 * 2.5) ** 0.5)       # geometric mean over ranks
    assert agg["other"]["resolve"]["throughput_speedup"] == pytest.approx(15.0 / 11.0)
