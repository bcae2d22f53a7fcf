"""SURVEY NEXT-4 experiment: the 1D row-partitioned GR with one all-gather per BFS
level (paper_conf_icpp_devecikuc13_b200/pgr.py; kernels include/mcm.h mcm_pgr_*).

CPU tier: the orchestration (slices, count words, termination, min-reduction,
maxLevel) with the level step written out here in numpy from Alg. 2's definition
(a column's label is one more than its first-reached row's, its mate
row one more again), single-process with P parts and under gloo at world size 2
-- every label, maxLevel and the reached-free count must equal the oracle's GR.
GPU tier: the same with libmcm's level kernels, bit-exact against the oracle."""
import os
import socket

import numpy as np
import pytest
import torch

import oracle
import synth
from paper_conf_icpp_devecikuc13_b200 import pgr


class NumpyParts:
    """Test stand-in for pgr.DeviceParts on CPU tensors (the pull step in numpy)."""

    def __init__(self, g, rm, cm):
        self.g, self.rm, self.cm = g, np.asarray(rm), np.asarray(cm)
        order = np.argsort(g.indices, kind="stable")  # CSC: Gamma(v) of every column
        self.cadj = np.repeat(np.arange(g.m), np.diff(g.indptr))[order]
        self.cptr = np.concatenate([[0], np.cumsum(np.bincount(g.indices, minlength=g.n))])
        self.rf = torch.zeros(1, dtype=torch.int64)

    def zeros(self, k):
        return torch.zeros(k, dtype=torch.int32)

    def labels(self):
        return torch.empty(self.g.m, dtype=torch.int32), torch.empty(self.g.n, dtype=torch.int32)

    def _bits(self, F, W, P):
        words = F.numpy().view(np.uint32).reshape(P, W + 1)[:, :W].reshape(-1)
        bits = np.unpackbits(words.view(np.uint8), bitorder="little").astype(bool)
        return bits[: self.g.m]

    def _write(self, slice_, mask):
        W = slice_.numel() - 1
        b = np.zeros(32 * W, bool)
        b[: mask.size] = mask
        slice_[:W] = torch.from_numpy(np.packbits(b, bitorder="little").view(np.int32).copy())
        slice_[W] = int(mask.sum())

    def init(self, P, p, W, slice_, pr, pc):
        INF = self.g.m + self.g.n
        r0, r1 = 32 * W * p, min(self.g.m, 32 * W * (p + 1))
        src = self.rm[r0:r1] == -1
        pr[:] = INF
        pr[r0:r1] = torch.from_numpy(np.where(src, 0, INF).astype(np.int32))
        pc[:] = INF
        self._write(slice_, src)

    def level(self, P, p, W, L, F, slice_, pr, pc):
        g, INF = self.g, self.g.m + self.g.n
        inF = self._bits(F, W, P)
        hit = lambda v: bool(inF[self.cadj[self.cptr[v]:self.cptr[v + 1]]].any())  # noqa: E731
        r0, r1 = 32 * W * p, min(g.m, 32 * W * (p + 1))
        add = np.zeros(max(r1 - r0, 0), bool)
        for u in range(r0, r1):
            v = self.rm[u]
            if pr[u] == INF and 0 <= v < g.n and self.cm[v] == u and hit(v):
                pc[v], pr[u] = 2 * L + 1, 2 * L + 2
                add[u - r0] = True
        self._write(slice_, add)
        CB = -(-g.n // P)
        for v in range(CB * p, min(g.n, CB * (p + 1))):
            w = self.cm[v]
            if pc[v] != INF or (0 <= w < g.m and self.rm[w] == v):
                continue
            if hit(v):
                pc[v] = 2 * L + 1
                self.rf += 1

    def reached_free(self):
        return self.rf


def _cases():
    rng = np.random.default_rng(5)
    out = []
    for g in (synth.config("C1", 0.05), synth.config("C2", 0.0005), synth.hall_violator(300, 40, 11, 3),
              synth.config("C4", 1 / 8192)):
        _, rm, cm = oracle.cheap_match(g)
        out.append((g, rm, cm))
        rm2, cm2 = rm.copy(), cm.copy()
        for u in rng.choice(np.nonzero(rm >= 0)[0], size=min(5, int((rm >= 0).sum())), replace=False):
            cm2[rm2[u]] = -2 if u % 2 else cm2[rm2[u]]
            rm2[u] = -1
        out.append((g, rm2, cm2))
    return out


def _check(g, rm, cm, pr, pc, ml, rf):
    epr, epc, eml, erf = oracle.global_relabel(g, rm, cm)
    assert np.array_equal(np.asarray(pr), epr)
    assert np.array_equal(np.asarray(pc), epc)
    assert ml == eml and rf == erf


@pytest.mark.parametrize("P", [1, 2, 3, 5])
def test_partitioned_relabel_single_process(P):
    for g, rm, cm in _cases():
        ops = NumpyParts(g, rm, cm)
        pr, pc, ml, rf, levels = pgr.partitioned_relabel(ops, pgr.Collective(False), g.m, g.n, P, list(range(P)))
        _check(g, rm, cm, pr.numpy(), pc.numpy(), ml, rf)
        assert levels >= 1


def test_words_per_part():
    for m in (0, 1, 31, 32, 33, 1000, 4097):
        for P in (1, 2, 3, 8):
            W = pgr.words_per_part(m, P)
            assert W >= 1 and 32 * W * P >= m and (W == 1 or 32 * (W - 1) * P < m)


def _free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def _worker(rank, world, port, q):
    import torch.distributed as dist

    os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        res = []
        for g, rm, cm in _cases():
            ops = NumpyParts(g, rm, cm)
            pr, pc, ml, rf, levels = pgr.partitioned_relabel(ops, pgr.Collective(True), g.m, g.n, world, [rank])
            res.append((pr.numpy().copy(), pc.numpy().copy(), ml, rf, levels))
        q.put((rank, res))
    finally:
        dist.destroy_process_group()


@pytest.mark.timeout(300)
def test_partitioned_relabel_two_ranks_gloo():
    import torch.multiprocessing as mp

    world, port = 2, _free_port()
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    procs = [ctx.Process(target=_worker, args=(r, world, port, q)) for r in range(world)]
    for p in procs:
        p.start()
    res = sorted((q.get(timeout=240) for _ in range(world)), key=lambda x: x[0])
    for p in procs:
        p.join(60)
        assert p.exitcode == 0
    cases = _cases()
    for (_, r0), (_, r1) in [(res[0], res[1])]:
        for (g, rm, cm), a, b in zip(cases, r0, r1):
            _check(g, rm, cm, *a[:4])
            assert all(np.array_equal(x, y) for x, y in zip(a[:2], b[:2])) and a[2:] == b[2:]  # same on every rank


@pytest.mark.gpu
@pytest.mark.parametrize("P", [1, 2, 3, 8])
def test_partitioned_relabel_gpu_bit_exact(P):
    import paper_conf_icpp_devecikuc13_b200 as pkg

    cases = _cases() + [(g, *oracle.cheap_match(g)[1:]) for g in (synth.config("C2", 0.01), synth.config("C3", 0.001))]
    for g, rm, cm in cases:
        ip = torch.from_numpy(g.indptr).cuda()
        ix = torch.from_numpy(g.indices).cuda()
        mt = pkg.Matcher(ip, ix, g.m, g.n)
        drm = torch.from_numpy(np.ascontiguousarray(rm, np.int32)).cuda()
        dcm = torch.from_numpy(np.ascontiguousarray(cm, np.int32)).cuda()
        ops = pgr.DeviceParts(mt, drm, dcm)
        pr, pc, ml, rf, levels = pgr.partitioned_relabel(ops, pgr.Collective(False), g.m, g.n, P, list(range(P)))
        _check(g, rm, cm, pr.cpu().numpy(), pc.cpu().numpy(), ml, rf)
        mt.close()


@pytest.mark.gpu
def test_pgr_rejects_bad_arguments():
    import paper_conf_icpp_devecikuc13_b200 as pkg

    g = synth.config("C1", 0.05)
    mt = pkg.Matcher(torch.from_numpy(g.indptr).cuda(), torch.from_numpy(g.indices).cuda(), g.m, g.n)
    rm = torch.full((g.m,), -1, dtype=torch.int32, device="cuda")
    pr = torch.empty(g.m, dtype=torch.int32, device="cuda")
    pc = torch.empty(g.n, dtype=torch.int32, device="cuda")
    W = pgr.words_per_part(g.m, 2)
    for P, p, w in ((0, 0, W), (2, 2, W), (2, 0, W - 1 if W > 1 else 0)):
        with pytest.raises(pkg.MCMError):
            mt.pgr_init(P, p, w, rm, torch.zeros(max(w, 0) + 1, dtype=torch.int32, device="cuda"), pr, pc)
    mt.close()
