"""Multi-process host logic of bench.py on CPU (gloo, world_size 2): replicas only
 -- every rank gets its own instance, times reduce by MAX over ranks
and units by SUM, no data-path collective."""
import os
import socket

import pytest
import torch
import torch.distributed as dist
import torch.multiprocessing as mp

import bench


def _free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def _worker(rank, world, port, q):
    os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        g = bench._graph("C1", rank)
        t = 10.0 + rank  # rank 1 is the slowest
        out = bench.reduce_over_ranks(t, 2 * t, 3 * t, 4 * t, float(g.nnz), world, torch.device("cpu"))
        q.put((rank, out, g.digest(), g.m, g.nnz))
    finally:
        dist.destroy_process_group()


@pytest.mark.timeout(300)
def test_two_rank_reduction_and_instances():
    world = 2
    port = _free_port()
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    procs = [ctx.Process(target=_worker, args=(r, world, port, q)) for r in range(world)]
    for p in procs:
        p.start()
    res = [q.get(timeout=240) for _ in range(world)]
    for p in procs:
        p.join(60)
        assert p.exitcode == 0
    res.sort()
    (r0, out0, d0, m0, nnz0), (r1, out1, d1, m1, nnz1) = res
    assert out0 == out1  # every rank sees the same reduced numbers
    t_step, t_e2e, t_solve, t_create, nnz = out0
    assert (t_step, t_e2e, t_solve, t_create) == (11.0, 22.0, 33.0, 44.0)  # max over ranks
    assert nnz == nnz0 + nnz1  # units: sum over ranks
    assert d0 != d1 and m0 == m1  # independent instances of the same recipe


def test_single_rank_passthrough():
    assert bench.reduce_over_ranks(1.0, 2.0, 3.0, 4.0, 5.0, 1, torch.device("cpu")) == (1.0, 2.0, 3.0, 4.0, 5.0)
