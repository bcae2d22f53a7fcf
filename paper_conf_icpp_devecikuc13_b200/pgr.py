"""an EXPERIMENT, not the solve path: a 1D row-partitioned global
relabel (Alg. 2 with the matched test of Alg. 5 l.6, /root/reference/PAPER.md:257-272,
401-410) whose BFS levels exchange the row frontier as a bitmap with one
all-gather per level (NCCL over NVLink / NVSwitch when run under torchrun).

It exists to measure the claim of SURVEY.md 8(e) that a single G-PR instance does
not shard: a GR is hundreds of dependent BFS levels, and each level here costs a
collective.  The level kernels are libmcm's (include/mcm.h ``mcm_pgr_init`` /
``mcm_pgr_level``); this module only sequences them and the collectives.

Layout (include/mcm.h): P parts, W = ceil(ceil(m / 32) / P) bitmap words per part;
a frontier buffer is P slices of W + 1 int32 words (W bitmap words, one count
word).  Part p writes its slice of the next frontier; the all-gather gives every
part the whole frontier and every count, so the BFS stops, on every part at once,
at the first level whose counts sum to 0.  Labels: each part writes only what it
owns; the GR result is the elementwise minimum over the parts (one all-reduce
each for psi_row / psi_col at the end).
"""
from __future__ import annotations


def words_per_part(m: int, nparts: int) -> int:
    return max(1, -(-(-(-m // 32)) // nparts))


class DeviceParts:
    """The level kernels of libmcm for the parts this process runs (one part per
    rank under torch.distributed, or every part on one device for the
    single-process check).  Device tensors only (no CPU fallback)."""

    def __init__(self, mt, rmatch, cmatch, stream=None):
        import torch

        self.torch, self.mt, self.rm, self.cm, self.stream = torch, mt, rmatch, cmatch, stream
        self.m, self.n, self.device = mt.m, mt.n, mt.device
        self.rf = torch.zeros(1, dtype=torch.int64, device=self.device)

    def zeros(self, k):
        return self.torch.zeros(k, dtype=self.torch.int32, device=self.device)

    def labels(self):
        t = self.torch
        return t.empty(self.m, dtype=t.int32, device=self.device), t.empty(self.n, dtype=t.int32, device=self.device)

    def init(self, P, p, W, slice_, pr, pc):
        self.mt.pgr_init(P, p, W, self.rm, slice_, pr, pc, stream=self.stream)

    def level(self, P, p, W, L, frontier, slice_, pr, pc):
        self.mt.pgr_level(P, p, W, L, self.rm, self.cm, frontier, slice_, pr, pc, self.rf, stream=self.stream)

    def reached_free(self):
        return self.rf


class Collective:
    """The exchange: torch.distributed (``group`` None = the default group) when
    ``distributed``, else nothing (every part runs in this process)."""

    def __init__(self, distributed: bool, group=None):
        self.distributed, self.group = distributed, group

    def all_gather(self, buf, own):
        if self.distributed:
            import torch.distributed as dist

            dist.all_gather_into_tensor(buf, own, group=self.group)

    def all_reduce(self, t, op: str):
        if self.distributed:
            import torch.distributed as dist

            dist.all_reduce(t, op={"min": dist.ReduceOp.MIN, "sum": dist.ReduceOp.SUM}[op], group=self.group)


def partitioned_relabel(ops, coll, m: int, n: int, nparts: int, parts, on_level=None):
    """Run the partitioned GR.  ``parts``: the part ids this process runs (all of
    them when ``coll`` is not distributed).  Returns (psi_row, psi_col, max_level,
    reached_free, levels): labels after the min-reduction, maxLevel as GETITERGR
    uses it ((deepest row level) + 2, reading R6), the number of unmatched columns
    labelled, and the BFS levels run (= collectives in the level loop).
    ``on_level(L)`` (optional) is called after each level's exchange."""
    W = words_per_part(m, nparts)
    A, B = ops.zeros(nparts * (W + 1)), ops.zeros(nparts * (W + 1))
    lab = {p: ops.labels() for p in parts}  # every part its own label arrays, as on its own rank

    def own(buf, p):
        return buf[p * (W + 1):(p + 1) * (W + 1)]

    for p in parts:
        ops.init(nparts, p, W, own(A, p), *lab[p])
    if len(parts) == 1:
        coll.all_gather(A, own(A, parts[0]))
    total = int(A.view(nparts, W + 1)[:, W].sum().item())  # the level's counts (one D2H)
    L, deepest = 0, 0
    while total > 0:
        for p in parts:
            ops.level(nparts, p, W, L, A, own(B, p), *lab[p])
        if len(parts) == 1:
            coll.all_gather(B, own(B, parts[0]))
        total = int(B.view(nparts, W + 1)[:, W].sum().item())
        if total > 0:
            deepest = 2 * (L + 1)
        A, B = B, A
        L += 1
        if on_level is not None:
            on_level(L)
    pr, pc = lab[parts[0]]
    for p in parts[1:]:  # parts of this process, then the ranks
        pr, pc = pr.minimum(lab[p][0]), pc.minimum(lab[p][1])
    coll.all_reduce(pr, "min")
    coll.all_reduce(pc, "min")
    rf = ops.reached_free()
    coll.all_reduce(rf, "sum")
    return pr, pc, deepest + 2, int(rf.item()), L
