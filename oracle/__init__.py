"""CPU ORACLE -- test infrastructure only.

Only ``tests/``, ``__graft_entry__.smoke()`` and ``bench.py``'s ``cpu_baseline`` /
``--impl reference`` legs may import this package.  The product package
``paper_conf_icpp_devecikuc13_b200`` never imports it, and ``liboracle.so`` shares
no code with the CUDA library.

Contents (all cite PAPER.md, see ``oracle.c``'s header):

* C (``oracle.c``): transpose, cheap matching (reading R13), GR (Alg. 2),
  sequential PR-FIFO (Alg. 1 + GR every k(m+n) pushes), Hopcroft-Karp, validity
  checker, Konig certificate, the G-PR kernels as plain functions (INITKRNL
  Alg. 8, SHRKRNL, PUSHKRNL Alg. 9, FIXMATCHING) and the serial G-PR simulator
  built from them (Alg. 7/8/9 + Alg. 4/5).
* Python: brute force by edge-subset enumeration (<= ~16 edges) and by a
  column-bitmask DP (m small); shortest alternating distances by Bellman-Ford
  over the residual digraph (an independent pin for GR).

Pins (tests/test_oracle_*.py): brute force, closed forms (K_{a,b}, P_k, C_2k,
stars, grid double cover, permutation+noise, planted Hall violator, disjoint
unions), PR == HK, scipy's maximum_bipartite_matching, Konig cover of equal size.
"""
from __future__ import annotations

import ctypes
import os
import subprocess
from itertools import combinations

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_LIB_PATH = os.path.join(_HERE, "liboracle.so")
_lib = None


def build_lib(force: bool = False) -> str:
    src = os.path.join(_HERE, "oracle.c")
    if force or not os.path.exists(_LIB_PATH) or os.path.getmtime(_LIB_PATH) < os.path.getmtime(src):
        subprocess.check_call(["gcc", "-O3", "-march=x86-64-v2", "-fPIC", "-shared", "-o", _LIB_PATH, src, "-lm"])
    return _LIB_PATH


def _get():
    global _lib
    if _lib is None:
        build_lib()
        lib = ctypes.CDLL(_LIB_PATH)
        P32 = ctypes.POINTER(ctypes.c_int32)
        P64 = ctypes.POINTER(ctypes.c_int64)
        PU8 = ctypes.POINTER(ctypes.c_uint8)
        i32, i64, dbl = ctypes.c_int32, ctypes.c_int64, ctypes.c_double
        lib.or_transpose.argtypes = [i32, i32, P32, P32, P32, P32]
        lib.or_transpose.restype = ctypes.c_int
        lib.or_cheap_match.argtypes = [i32, i32, P32, P32, P32, P32]
        lib.or_cheap_match.restype = i64
        lib.or_global_relabel.argtypes = [i32, i32, P32, P32, P32, P32, P32, P32, P32, P64]
        lib.or_global_relabel.restype = ctypes.c_int
        lib.or_pr_fifo.argtypes = [i32, i32, P32, P32, P32, P32, P32, P32, dbl, P64]
        lib.or_pr_fifo.restype = i64
        lib.or_hopcroft_karp.argtypes = [i32, i32, P32, P32, P32, P32, P64]
        lib.or_hopcroft_karp.restype = i64
        lib.or_check_matching.argtypes = [i32, i32, P32, P32, P32, P32]
        lib.or_check_matching.restype = i64
        lib.or_konig_cover.argtypes = [i32, i32, P32, P32, P32, P32, PU8, PU8]
        lib.or_konig_cover.restype = i64
        lib.or_gpr_serial.argtypes = [i32, i32, P32, P32, P32, P32, P32, P32, dbl, P64, P64]
        lib.or_gpr_serial.restype = i64
        lib.or_gap_relabel.argtypes = [i32, i32, P32, P32, i32]
        lib.or_gap_relabel.restype = ctypes.c_int
        lib.or_initkrnl.argtypes = [i64, i32, P32, P32, P32, P32, P32]
        lib.or_initkrnl.restype = i64
        lib.or_shrkrnl.argtypes = [i64, i32, P32, P32, P32, P32, P32]
        lib.or_shrkrnl.restype = i64
        lib.or_pushkrnl.argtypes = [i32, i32, P32, P32, i64, i32, P32, P32, P32, P32, P32, P32, P32, ctypes.c_int, P64]
        lib.or_pushkrnl.restype = None
        lib.or_fixmatching.argtypes = [i32, i32, P32, P32]
        lib.or_fixmatching.restype = i64
        _lib = lib
    return _lib


def _p32(a):
    return a.ctypes.data_as(ctypes.POINTER(ctypes.c_int32))


def _p64(a):
    return a.ctypes.data_as(ctypes.POINTER(ctypes.c_int64))


def _i32(a):
    return np.ascontiguousarray(a, dtype=np.int32)


def _nonempty(n):
    return max(int(n), 1)


class CSC:
    """Gamma(v) of every column, built by the oracle's own stable transpose."""

    def __init__(self, m, n, indptr, indices):
        self.cptr = np.zeros(n + 1, np.int32)
        self.cadj = np.zeros(_nonempty(len(indices)), np.int32)
        rc = _get().or_transpose(m, n, _p32(_i32(indptr)), _p32(_i32(indices)), _p32(self.cptr), _p32(self.cadj))
        if rc != 0:
            raise ValueError(f"or_transpose rc={rc}")


def transpose(g):
    return CSC(g.m, g.n, g.indptr, g.indices)


def cheap_match(g, csc=None):
    """Reading R13: column-order greedy, first free row."""
    csc = csc or transpose(g)
    rm = np.empty(_nonempty(g.m), np.int32)
    cm = np.empty(_nonempty(g.n), np.int32)
    card = _get().or_cheap_match(g.m, g.n, _p32(csc.cptr), _p32(csc.cadj), _p32(rm), _p32(cm))
    return int(card), rm[: g.m], cm[: g.n]


def global_relabel(g, mu_row, mu_col):
    """Alg. 2 / Alg. 4-5 labels: (psi_row, psi_col, max_level, reached_free_cols)."""
    pr = np.empty(_nonempty(g.m), np.int32)
    pc = np.empty(_nonempty(g.n), np.int32)
    ml = np.zeros(1, np.int32)
    rf = np.zeros(1, np.int64)
    mu_row = _i32(mu_row) if g.m else np.zeros(1, np.int32)
    mu_col = _i32(mu_col) if g.n else np.zeros(1, np.int32)
    rc = _get().or_global_relabel(g.m, g.n, _p32(g.indptr), _p32(_i32(g.indices) if g.nnz else np.zeros(1, np.int32)),
                                  _p32(mu_row), _p32(mu_col), _p32(pr), _p32(pc), _p32(ml), _p64(rf))
    if rc != 0:
        raise RuntimeError(rc)
    return pr[: g.m], pc[: g.n], int(ml[0]), int(rf[0])


def _init(g, init, csc):
    if init == "greedy":
        _, rm, cm = cheap_match(g, csc)
        rm = np.concatenate([rm, [0]]).astype(np.int32)
        cm = np.concatenate([cm, [0]]).astype(np.int32)
    elif init == "empty":
        rm = np.full(g.m + 1, -1, np.int32)
        cm = np.full(g.n + 1, -1, np.int32)
    else:
        rm0, cm0 = init
        rm = np.concatenate([_i32(rm0), [0]]).astype(np.int32)
        cm = np.concatenate([_i32(cm0), [0]]).astype(np.int32)
    return rm, cm


def _adj(g):
    return _i32(g.indices) if g.nnz else np.zeros(1, np.int32)


def pr_fifo(g, k: float = 0.5, init="greedy", csc=None):
    """Sequential PR (Alg. 1) with FIFO and GR every ceil(k(m+n)) pushes.

    Returns (card, rmatch, cmatch, stats dict)."""
    csc = csc or transpose(g)
    rm, cm = _init(g, init, csc)
    st = np.zeros(4, np.int64)
    card = _get().or_pr_fifo(g.m, g.n, _p32(g.indptr), _p32(_adj(g)), _p32(csc.cptr), _p32(csc.cadj),
                             _p32(rm), _p32(cm), k, _p64(st))
    if card < 0:
        raise RuntimeError(card)
    return int(card), rm[: g.m], cm[: g.n], dict(pushes=int(st[0]), grs=int(st[1]), dead=int(st[2]), scanned=int(st[3]))


def hopcroft_karp(g, init="greedy", csc=None):
    csc = csc or transpose(g)
    rm, cm = _init(g, init, csc)
    ph = np.zeros(1, np.int64)
    card = _get().or_hopcroft_karp(g.m, g.n, _p32(csc.cptr), _p32(csc.cadj), _p32(rm), _p32(cm), _p64(ph))
    if card < 0:
        raise RuntimeError(card)
    return int(card), rm[: g.m], cm[: g.n]


def check_matching(g, rmatch, cmatch) -> int:
    """|M| if (rmatch, cmatch) is a valid, mutually consistent matching of g; else a negative code."""
    rm = _i32(rmatch) if g.m else np.zeros(1, np.int32)
    cm = _i32(cmatch) if g.n else np.zeros(1, np.int32)
    return int(_get().or_check_matching(g.m, g.n, _p32(g.indptr), _p32(_adj(g)), _p32(rm), _p32(cm)))


def konig_cover(g, rmatch, cmatch):
    """(size, cover_row, cover_col); size < 0 if M is not certified maximum."""
    cr = np.zeros(_nonempty(g.m), np.uint8)
    cc = np.zeros(_nonempty(g.n), np.uint8)
    rm = _i32(rmatch) if g.m else np.zeros(1, np.int32)
    cm = _i32(cmatch) if g.n else np.zeros(1, np.int32)
    PU8 = ctypes.POINTER(ctypes.c_uint8)
    size = _get().or_konig_cover(g.m, g.n, _p32(g.indptr), _p32(_adj(g)), _p32(rm), _p32(cm),
                                 cr.ctypes.data_as(PU8), cc.ctypes.data_as(PU8))
    return int(size), cr[: g.m], cc[: g.n]


def gap_relabel(m, n, psi_row, psi_col, H=None):
    """Reading R14 on copies of the labels -> (g, psi_row', psi_col'); g = -1: no gap."""
    if H is None:
        H = min(m + n + 2, 1 << 20)
    pr = np.concatenate([_i32(psi_row), [0]]).astype(np.int32)
    pc = np.concatenate([_i32(psi_col), [0]]).astype(np.int32)
    gl = _get().or_gap_relabel(m, n, _p32(pr), _p32(pc), H)
    if gl < -1:
        raise RuntimeError(gl)
    return int(gl), pr[:m], pc[:n]


def gpr_serial(g, k: float = 0.7, gr_fixed: bool = False, shrink_min: int = 512, dead_skip: bool = False,
               init="greedy", max_loops: int = 0, gap: bool = False, csc=None):
    """Serial G-PR (Alg. 7/8/9) -> (card, mu_row, mu_col, stats dict)."""
    csc = csc or transpose(g)
    rm, cm = _init(g, init, csc)
    opts = np.array([int(gr_fixed), shrink_min, int(dead_skip), max_loops, int(gap)], np.int64)
    st = np.zeros(8, np.int64)
    card = _get().or_gpr_serial(g.m, g.n, _p32(g.indptr), _p32(_adj(g)), _p32(csc.cptr), _p32(csc.cadj),
                                _p32(rm), _p32(cm), k, _p64(opts), _p64(st))
    if card < 0:
        raise RuntimeError(card)
    keys = ["loops", "grs", "levels", "pushes", "shrinks", "dead", "blocked", "gaps"]
    return int(card), rm[: g.m], cm[: g.n], dict(zip(keys, map(int, st)))


# ---------------------------------------------------------------- pure-Python pins
def edges_of(g):
    r = np.repeat(np.arange(g.m), np.diff(g.indptr))
    return list(zip(r.tolist(), g.indices.tolist()))


def brute_force_subsets(g) -> int:
    """Maximum |M| by enumerating edge subsets from the largest size down."""
    E = edges_of(g)
    for size in range(min(len(E), g.m, g.n), 0, -1):
        for sub in combinations(E, size):
            rs = {e[0] for e in sub}
            cs = {e[1] for e in sub}
            if len(rs) == size and len(cs) == size:
                return size
    return 0


def brute_force_dp(g) -> int:
    """Maximum |M| by DP over rows with a bitmask of used columns (n <= ~20)."""
    adj = [g.indices[g.indptr[u]: g.indptr[u + 1]].tolist() for u in range(g.m)]
    best = {0: 0}
    for u in range(g.m):
        nxt = dict(best)
        for mask, val in best.items():
            for v in adj[u]:
                b = 1 << v
                if not mask & b:
                    nm = mask | b
                    if nxt.get(nm, -1) < val + 1:
                        nxt[nm] = val + 1
        best = nxt
    return max(best.values())


def alternating_distances(g, mu_row, mu_col):
    """Shortest alternating distances from unmatched rows by Bellman-Ford over the
    digraph row -> each column of Gamma(u) (weight 1), column v -> its matched row
    (weight 1, when mu_row[mu_col[v]] == v).  Unreached = m+n.  Independent of
    or_global_relabel (no queue, no levels): an independent pin for GR labels."""
    INF = g.m + g.n
    dr = [0 if mu_row[u] == -1 else INF for u in range(g.m)]
    dc = [INF] * g.n
    adj = [g.indices[g.indptr[u]: g.indptr[u + 1]].tolist() for u in range(g.m)]
    changed = True
    while changed:
        changed = False
        for u in range(g.m):
            if dr[u] >= INF:
                continue
            for v in adj[u]:
                if dr[u] + 1 < dc[v]:
                    dc[v] = dr[u] + 1
                    changed = True
        for v in range(g.n):
            w = mu_col[v]
            if dc[v] < INF and w > -1 and mu_row[w] == v and dc[v] + 1 < dr[w]:
                dr[w] = dc[v] + 1
                changed = True
    return np.array(dr, np.int32), np.array(dc, np.int32)


# ---------------------------------------------------------------- G-PR kernels as functions
def _pad(a):
    a = _i32(a)
    return np.concatenate([a, [0]]).astype(np.int32)


def initkrnl(loop, mu_row, mu_col, Ac, Ap, iA):
    """G-PR-INITKRNL (Alg. 8) on copies -> (active_slots, Ac', iA')."""
    Ac, iA = _pad(Ac), _pad(iA)
    a = _get().or_initkrnl(len(Ac) - 1, int(loop), _p32(_pad(mu_row)), _p32(_pad(mu_col)), _p32(Ac), _p32(_pad(Ap)),
                           _p32(iA))
    return int(a), Ac[:-1], iA[:-1]


def shrkrnl(loop, mu_row, mu_col, Ac, Ap, iA):
    """G-PR-SHRKRNL on copies -> (len', Ac'[:len'], iA')."""
    Ac, iA = _pad(Ac), _pad(iA)
    ln = _get().or_shrkrnl(len(Ac) - 1, int(loop), _p32(_pad(mu_row)), _p32(_pad(mu_col)), _p32(Ac), _p32(_pad(Ap)),
                           _p32(iA))
    return int(ln), Ac[:ln], iA[:-1]


def pushkrnl(g, loop, mu_row, mu_col, psi_row, psi_col, iA, Ac, dead_skip=False, csc=None):
    """G-PR-PUSHKRNL (Alg. 9), slots in order, on copies ->
    dict(mu_row, mu_col, psi_row, psi_col, Ac, Ap, pushes, blocked, dead)."""
    csc = csc or transpose(g)
    mr, mc, pr, pc, Acp = _pad(mu_row), _pad(mu_col), _pad(psi_row), _pad(psi_col), _pad(Ac)
    Ap = np.full(len(Acp), -7, np.int32)
    st = np.zeros(3, np.int64)
    _get().or_pushkrnl(g.m, g.n, _p32(csc.cptr), _p32(csc.cadj), len(Acp) - 1, int(loop), _p32(mr), _p32(mc), _p32(pr),
                       _p32(pc), _p32(_pad(iA)), _p32(Acp), _p32(Ap), int(bool(dead_skip)), _p64(st))
    return dict(mu_row=mr[: g.m], mu_col=mc[: g.n], psi_row=pr[: g.m], psi_col=pc[: g.n], Ac=Acp[:-1], Ap=Ap[:-1],
                pushes=int(st[0]), blocked=int(st[1]), dead=int(st[2]))


def fixmatching(m, n, mu_row, mu_col):
    """FIXMATCHING on a copy -> (|M|, mu_col')."""
    mc = _pad(mu_col)
    card = _get().or_fixmatching(int(m), int(n), _p32(_pad(mu_row)), _p32(mc))
    return int(card), mc[:n]
