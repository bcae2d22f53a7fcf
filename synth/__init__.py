"""Seeded synthetic bipartite graphs (CSR rows -> cols) for tests and the bench.

This module is the ONLY code shared by the oracle side and the CUDA side, and it
holds none of the matching method's arithmetic: it only draws patterns.  The
heavy families are C (``synth.c``, OpenMP, counter-based RNG so the output does
not depend on the thread count); the small closed-form families used to pin the
oracle are plain numpy on top of :func:`from_pairs`.

Config recipes follow SURVEY.md §8(d):

====  =====================================================================
C1    uniform 10,000 x 10,000, 80,000 samples, dedup (seed 1)
C2    permuted banded 1.5M x 1.5M, diag + Poisson(2.47) in +-64 + 150 rails
      x 2,000 rows (seed 2); MM = n (full diagonal)
C3    road lattice s = 4,900 (24.01M vertices), planted dominoes, a=.5 b=.4
      c=.1, symmetric id scramble inside blocks of 256 ids (seed 3); MM = N
C4    R-MAT scale 23, 2^27 samples, (.57,.19,.19,.05), permuted (seed 4)
C5    64 x uniform 2^21 x 2^21, 16 * 2^21 samples (seeds 1000+i)
====  =====================================================================
"""
from __future__ import annotations

import ctypes
import hashlib
import os
from dataclasses import dataclass

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_LIB_PATH = os.path.join(_HERE, "libsynth.so")


class _Csr(ctypes.Structure):
    _fields_ = [
        ("m", ctypes.c_int32),
        ("n", ctypes.c_int32),
        ("nnz", ctypes.c_int64),
        ("indptr", ctypes.POINTER(ctypes.c_int32)),
        ("indices", ctypes.POINTER(ctypes.c_int32)),
    ]


_lib = None


def build_lib(force: bool = False) -> str:
    """Compile libsynth.so (gcc -O3 -fopenmp)."""
    src = os.path.join(_HERE, "synth.c")
    if force or not os.path.exists(_LIB_PATH) or os.path.getmtime(_LIB_PATH) < os.path.getmtime(src):
        import subprocess

        subprocess.check_call(
            ["gcc", "-O3", "-march=x86-64-v2", "-fopenmp", "-fPIC", "-shared", "-o", _LIB_PATH, src, "-lm"]
        )
    return _LIB_PATH


def _get():
    global _lib
    if _lib is None:
        build_lib()
        lib = ctypes.CDLL(_LIB_PATH)
        P = ctypes.POINTER
        i32, i64, u64, dbl = ctypes.c_int32, ctypes.c_int64, ctypes.c_uint64, ctypes.c_double
        lib.synth_uniform.argtypes = [i32, i32, i64, u64, P(_Csr)]
        lib.synth_banded.argtypes = [i32, dbl, i32, i32, i32, u64, ctypes.c_int, P(_Csr)]
        lib.synth_road.argtypes = [i32, dbl, dbl, dbl, u64, ctypes.c_int, ctypes.c_int, i32, P(_Csr)]
        lib.synth_rmat.argtypes = [i32, i64, dbl, dbl, dbl, u64, ctypes.c_int, P(_Csr)]
        lib.synth_from_pairs.argtypes = [i32, i32, P(i32), P(i32), i64, P(_Csr)]
        lib.synth_free.argtypes = [P(_Csr)]
        lib.synth_set_threads.argtypes = [ctypes.c_int]
        _lib = lib
    return _lib


@dataclass
class Graph:
    """CSR of the m x n pattern: rows V_R = V1, columns V_C = V2."""

    m: int
    n: int
    indptr: np.ndarray  # int32 [m+1]
    indices: np.ndarray  # int32 [nnz]
    name: str = ""
    mm: int | None = None  # closed-form maximum cardinality, when the recipe fixes it

    @property
    def nnz(self) -> int:
        return int(self.indices.shape[0])

    def digest(self) -> str:
        h = hashlib.sha256()
        h.update(np.array([self.m, self.n, self.nnz], dtype=np.int64).tobytes())
        h.update(np.ascontiguousarray(self.indptr, dtype=np.int32).tobytes())
        h.update(np.ascontiguousarray(self.indices, dtype=np.int32).tobytes())
        return h.hexdigest()[:32]


def _take(c: _Csr, name: str, mm=None) -> Graph:
    lib = _get()
    m, nnz = c.m, c.nnz
    indptr = np.ctypeslib.as_array(c.indptr, shape=(m + 1,)).copy()
    indices = np.ctypeslib.as_array(c.indices, shape=(max(nnz, 1),))[:nnz].copy()
    lib.synth_free(ctypes.byref(c))
    return Graph(m, c.n, indptr, indices, name, mm)


def _check(rc: int, what: str):
    if rc != 0:
        raise RuntimeError(f"synth: {what} failed (rc={rc})")


def set_threads(t: int) -> int:
    return _get().synth_set_threads(t)


def uniform(m: int, n: int, samples: int, seed: int, name: str = "uniform") -> Graph:
    c = _Csr()
    _check(_get().synth_uniform(m, n, samples, seed, ctypes.byref(c)), "uniform")
    return _take(c, name)


def banded(n: int, lam: float = 2.47, w: int = 64, rails: int = 150, rail_len: int = 2000, seed: int = 2,
           permute: bool = True, name: str = "banded") -> Graph:
    c = _Csr()
    _check(_get().synth_banded(n, lam, w, rails, rail_len, seed, int(permute), ctypes.byref(c)), "banded")
    return _take(c, name, mm=n)  # full diagonal => perfect matching


def road(s: int, a: float = 0.5, b: float = 0.4, cdiag: float = 0.1, seed: int = 3, shuffle: bool = True,
         permute: bool = False, scramble: int = 256, name: str = "road") -> Graph:
    c = _Csr()
    _check(_get().synth_road(s, a, b, cdiag, seed, int(shuffle), int(permute), scramble, ctypes.byref(c)), "road")
    # planted dominoes (x, x+1), x even, give a perfect matching iff s is even
    return _take(c, name, mm=s * s if s % 2 == 0 else None)


def rmat(scale: int, samples: int, a: float = 0.57, b: float = 0.19, c: float = 0.19, seed: int = 4,
         permute: bool = True, name: str = "rmat") -> Graph:
    cs = _Csr()
    _check(_get().synth_rmat(scale, samples, a, b, c, seed, int(permute), ctypes.byref(cs)), "rmat")
    return _take(cs, name)


def from_pairs(m: int, n: int, rows, cols, name: str = "pairs", mm=None) -> Graph:
    rows = np.ascontiguousarray(rows, dtype=np.int32)
    cols = np.ascontiguousarray(cols, dtype=np.int32)
    c = _Csr()
    P = ctypes.POINTER(ctypes.c_int32)
    _check(
        _get().synth_from_pairs(m, n, rows.ctypes.data_as(P), cols.ctypes.data_as(P), rows.shape[0], ctypes.byref(c)),
        "from_pairs",
    )
    return _take(c, name, mm)


# ---------------------------------------------------------------- the five configs
def config(name: str, scale: float = 1.0, index: int = 0) -> Graph:
    """The BASELINE.json configs.  ``scale`` < 1 shrinks the vertex count for tests."""
    if name == "C1":
        m = max(2, int(10_000 * scale))
        return uniform(m, m, 8 * m, 1, name="C1")
    if name == "C2":
        n = max(256, int(1_500_000 * scale))
        rails = max(1, int(150 * scale)) if scale < 1 else 150
        return banded(n, 2.47, 64, rails, min(2000, n), 2, True, name="C2")
    if name == "C3":
        s = max(4, int(4900 * scale ** 0.5)) & ~1
        return road(s, 0.5, 0.4, 0.1, 3, True, False, 256, name="C3")
    if name == "C4":
        sc = max(4, 23 + int(np.round(np.log2(scale)))) if scale < 1 else 23
        return rmat(sc, 16 << sc, seed=4, name="C4")
    if name == "C5":
        sc = max(4, 21 + int(np.round(np.log2(scale)))) if scale < 1 else 21
        return uniform(1 << sc, 1 << sc, 16 << sc, 1000 + index, name=f"C5[{index}]")
    raise KeyError(name)


# ---------------------------------------------------------------- closed-form families
def complete(a: int, b: int) -> Graph:
    """K_{a,b}: MM = min(a, b)."""
    r, c = np.meshgrid(np.arange(a), np.arange(b), indexing="ij")
    return from_pairs(a, b, r.ravel(), c.ravel(), f"K{a},{b}", mm=min(a, b))


def path(k: int) -> Graph:
    """Path P_k on k vertices alternating row/col (row first): MM = floor(k/2)."""
    nr, nc = (k + 1) // 2, k // 2
    rows, cols = [], []
    for i in range(k - 1):  # edge between vertex i and i+1
        if i % 2 == 0:
            rows.append(i // 2); cols.append(i // 2)
        else:
            rows.append((i + 1) // 2); cols.append(i // 2)
    return from_pairs(nr, nc, rows, cols, f"P{k}", mm=k // 2)


def cycle(k: int) -> Graph:
    """Even cycle C_{2k}: rows i, cols i, edges i-i and i-(i+1 mod k): MM = k."""
    i = np.arange(k)
    rows = np.concatenate([i, i])
    cols = np.concatenate([i, (i + 1) % k])
    return from_pairs(k, k, rows, cols, f"C{2*k}", mm=k)


def star(leaves: int) -> Graph:
    """One column adjacent to `leaves` rows: MM = 1 (0 leaves -> 0)."""
    return from_pairs(leaves, 1, np.arange(leaves), np.zeros(leaves), f"star{leaves}", mm=min(1, leaves))


def grid_double_cover(s: int) -> Graph:
    """s x s grid graph G, bipartite double cover (row i - col j for each arc i->j).

    The grid is bipartite, so its double cover is two disjoint copies of it, and
    MM = 2 * floor(s^2 / 2) = s^2 - (s mod 2) (the grid has a perfect matching
    for even s, a near-perfect one for odd s)."""
    idx = np.arange(s * s).reshape(s, s)
    a = np.concatenate([idx[:, :-1].ravel(), idx[:-1, :].ravel()])
    b = np.concatenate([idx[:, 1:].ravel(), idx[1:, :].ravel()])
    rows = np.concatenate([a, b])
    cols = np.concatenate([b, a])
    return from_pairs(s * s, s * s, rows, cols, f"grid{s}", mm=s * s - (s % 2))


def permutation_noise(n: int, noise: int, seed: int) -> Graph:
    """Random permutation matrix plus `noise` random entries: MM = n."""
    rng = np.random.default_rng(seed)
    p = rng.permutation(n)
    rows = np.concatenate([np.arange(n), rng.integers(0, n, noise)])
    cols = np.concatenate([p, rng.integers(0, n, noise)])
    return from_pairs(n, n, rows, cols, f"perm{n}+{noise}", mm=n)


def hall_violator(n: int, t: int, d: int, seed: int, extra: int = 2) -> Graph:
    """Planted Hall violator: columns S = {0..t+d-1} adjacent only
    to rows T = {0..t-1} (diagonal i-i for i<t plus random); row i >= t has edge
    i-(i+d) when i+d < n plus `extra` random edges into columns >= t+d.  Random row
    and column permutations.  MM = n - d."""
    rng = np.random.default_rng(seed)
    rows, cols = [np.arange(t)], [np.arange(t)]
    kS = (t + d) * 2
    rows.append(rng.integers(0, t, kS)); cols.append(rng.integers(0, t + d, kS))
    i = np.arange(t, n)
    ok = i + d < n
    rows.append(i[ok]); cols.append(i[ok] + d)
    if n > t + d:
        rr = np.repeat(i, extra)
        rows.append(rr); cols.append(rng.integers(t + d, n, rr.shape[0]))
    rows = np.concatenate(rows); cols = np.concatenate(cols)
    pr, pc = rng.permutation(n), rng.permutation(n)
    return from_pairs(n, n, pr[rows], pc[cols], f"hall{n},{t},{d}", mm=n - d)


def disjoint_union(parts: list[Graph], seed: int) -> Graph:
    """Disjoint union with random row and column relabelling: MM = sum of the parts."""
    rows, cols = [], []
    ro = co = 0
    for g in parts:
        r = np.repeat(np.arange(g.m, dtype=np.int64), np.diff(g.indptr))
        rows.append(r + ro); cols.append(g.indices.astype(np.int64) + co)
        ro += g.m; co += g.n
    rng = np.random.default_rng(seed)
    pr, pc = rng.permutation(ro), rng.permutation(co)
    rows = np.concatenate(rows) if rows else np.zeros(0, np.int64)
    cols = np.concatenate(cols) if cols else np.zeros(0, np.int64)
    mm = sum(g.mm for g in parts) if all(g.mm is not None for g in parts) else None
    return from_pairs(ro, co, pr[rows], pc[cols], "union", mm=mm)


def random_small(m: int, n: int, p: float, seed: int) -> Graph:
    """Erdos-Renyi bipartite pattern (each entry w.p. p) for brute-force pins."""
    rng = np.random.default_rng(seed)
    mask = rng.random((m, n)) < p
    r, c = np.nonzero(mask)
    return from_pairs(m, n, r, c, f"er{m}x{n}")


# ---------------------------------------------------------------- unit-step inputs
def push_instance(K: int, seed: int, loop: int = 5, deg_mix=((0.6, 1, 8), (0.25, 9, 64), (0.1, 65, 512),
                                                             (0.05, 513, 3000)),
                  p_mate=0.5, p_inf=0.1, p_dead=0.05, p_empty=0.05, p_inf_col=0.02, p_blocked=0.3):
    """A PUSHKRNL input (Alg. 9) whose active columns do not interact, so a parallel
    push is deterministic: K active columns, each with a PRIVATE set of rows (no row
    is adjacent to two active columns); a row may be matched to a private "mate"
    column w (G(w) = {that row}, w not in the worklist).  Labels respect the
    neighbourhood invariant psi(u) >= psi(v) - 1 on every edge of an active column
    (P:203-209), under which the first minimum of a chunked scan equals the serial
    one (reading R11).  Degrees follow deg_mix (fraction, min, max) so lane groups,
    warps and CTA-wide scans all occur.  Pure input construction: no matching
    arithmetic.  Returns (graph, state) with state = dict(mu_row, mu_col, psi_row,
    psi_col, iA, Ac, loop) as int32 arrays (INF = m + n)."""
    rng = np.random.default_rng(seed)
    fr = np.array([f for f, _, _ in deg_mix])
    kind = rng.choice(len(deg_mix), size=K, p=fr / fr.sum())
    lo = np.array([a for _, a, _ in deg_mix])[kind]
    hi = np.array([b for _, _, b in deg_mix])[kind]
    deg = rng.integers(lo, hi + 1)
    R = int(deg.sum())
    owner = np.repeat(np.arange(K), deg)              # active column (local id) of each private row
    has_mate = rng.random(R) < p_mate
    nm = int(has_mate.sum())
    m, n = R, K + nm
    INF = m + n
    rperm = rng.permutation(m)                        # row ids shuffled
    cperm = rng.permutation(n)                        # column ids shuffled (active: local 0..K-1, mates: K..)
    row_id = rperm[np.arange(R)]
    act_id = cperm[np.arange(K)]
    mate_id = np.full(R, -1, np.int64)
    mate_id[has_mate] = cperm[K + np.arange(nm)]
    rows = np.concatenate([row_id, row_id[has_mate]])
    cols = np.concatenate([act_id[owner], mate_id[has_mate]])
    g = from_pairs(m, n, rows, cols, name=f"push_instance(K={K},seed={seed})")
    mu_row = np.full(m, -1, np.int32)
    mu_col = np.full(n, -1, np.int32)
    mu_row[row_id[has_mate]] = mate_id[has_mate]
    mu_col[mate_id[has_mate]] = row_id[has_mate]
    psi_row = np.full(m, INF, np.int32)
    psi_col = rng.integers(1, 2 * INF if INF < 40 else 40, n).astype(np.int32)
    psi_col = np.minimum(psi_col, INF)
    pv = rng.integers(1, 30, K)
    pv[rng.random(K) < p_inf_col] = INF               # label already infinite (R19 when dead_skip)
    psi_col[act_id] = pv
    base = np.maximum(pv[owner] - 1, 0)
    lab = base + rng.integers(0, 12, R)
    lab[rng.random(R) < p_inf] = INF
    lab[np.isin(owner, np.nonzero(rng.random(K) < p_dead)[0])] = INF   # every row infinite: the column dies
    psi_row[row_id] = np.minimum(lab, INF)
    iA = rng.integers(-1, loop, n).astype(np.int32)
    blk = has_mate & (rng.random(R) < p_blocked)
    iA[mate_id[blk]] = loop                           # the displaced column was active this loop: blocked
    iA[act_id] = loop                                 # the fix step marked the active columns
    Ac = act_id[rng.permutation(K)].astype(np.int64)
    empty = rng.random(K) < p_empty
    Ac[empty] = -1
    state = dict(mu_row=mu_row, mu_col=mu_col, psi_row=psi_row, psi_col=psi_col.astype(np.int32), iA=iA,
                 Ac=Ac.astype(np.int32), loop=loop)
    return g, state
