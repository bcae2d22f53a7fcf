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


def _batch_worker(rank, world, port, q):
    """bench.run_batch's host logic on CPU: rank r takes graphs r, r+N, ... of the C5
    recipe (here at 1/256 scale), solves them (the oracle stands in for the GPU
    solve on this CPU tier), and the job's units are summed over ranks."""
    import oracle

    os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        mine = bench.batch_partition(8, world, rank)
        graphs = bench.batch_graphs(mine, scale=1 / 256)
        cards = [oracle.hopcroft_karp(g)[0] for g in graphs]
        nnz = float(sum(g.nnz for g in graphs))
        out = bench.reduce_over_ranks(1.0 + rank, 2.0, 1.0, 0.0, nnz, world, torch.device("cpu"))
        got = [None] * world
        dist.all_gather_object(got, (mine, cards, [g.digest() for g in graphs], nnz))
        q.put((rank, out, got))
    finally:
        dist.destroy_process_group()


@pytest.mark.timeout(300)
def test_two_rank_batch_partition():
    world = 2
    port = _free_port()
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    procs = [ctx.Process(target=_batch_worker, args=(r, world, port, q)) for r in range(world)]
    for p in procs:
        p.start()
    res = sorted(q.get(timeout=240) for _ in range(world))
    for p in procs:
        p.join(60)
        assert p.exitcode == 0
    (_, out0, got), (_, out1, _) = res
    assert out0 == out1
    idx = sorted(i for mine, _, _, _ in got for i in mine)
    assert idx == list(range(8))  # every graph on exactly one rank
    assert got[0][0] == [0, 2, 4, 6] and got[1][0] == [1, 3, 5, 7]
    digests = [d for _, _, ds, _ in got for d in ds]
    assert len(set(digests)) == 8  # independent instances (seed 1000 + i)
    for mine, cards, _, _ in got:
        for i, c in zip(mine, cards):
            g = bench.batch_graphs([i], scale=1 / 256)[0]
            assert c == g.n or c == oracle_mm(g)
    assert out0[4] == sum(x[3] for x in got)  # units: sum over ranks
    assert out0[0] == 2.0  # time: max over ranks


def oracle_mm(g):
    import oracle

    return oracle.hopcroft_karp(g)[0]


def test_batch_partition_covers():
    for world in (1, 2, 3, 4, 8):
        parts = [bench.batch_partition(64, world, r) for r in range(world)]
        flat = sorted(i for p in parts for i in p)
        assert flat == list(range(64))
        assert max(len(p) for p in parts) - min(len(p) for p in parts) <= 1
