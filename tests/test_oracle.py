"""Pins for the CPU oracle (runs on CPU, -m "not gpu").

The oracle is pinned to things other than itself (SURVEY.md §8(c) "Pins"):
brute force (edge-subset enumeration, bitmask DP, permutation closed form),
closed forms (K_{a,b}, P_k, C_2k, stars, grid double cover, permutation+noise,
planted Hall violator, disjoint unions), a third-party library
(scipy.sparse.csgraph.maximum_bipartite_matching), Bellman-Ford distances for GR
labels, and the Konig certificate.  Two independent oracles (PR-FIFO, Hopcroft-
Karp) and the serial G-PR simulator must all agree with the pins.
"""
import itertools

import numpy as np
import pytest

import oracle
import synth


def all_oracles(g, **kw):
    """Cardinalities from every oracle, each result validity- and Konig-checked."""
    out = {}
    for init in ("greedy", "empty"):
        c, rm, cm, _ = oracle.pr_fifo(g, init=init)
        out[f"pr_{init}"] = (c, rm, cm)
        c, rm, cm = oracle.hopcroft_karp(g, init=init)
        out[f"hk_{init}"] = (c, rm, cm)
        c, rm, cm, _ = oracle.gpr_serial(g, init=init, **kw)
        out[f"gpr_{init}"] = (c, rm, cm)
    cards = {}
    for k, (c, rm, cm) in out.items():
        assert oracle.check_matching(g, rm, cm) == c, (g.name, k)
        size, cr, cc = oracle.konig_cover(g, rm, cm)
        assert size == c, (g.name, k, size, c)
        cards[k] = c
    return cards


def assert_all(g, expected, **kw):
    cards = all_oracles(g, **kw)
    assert set(cards.values()) == {expected}, (g.name, cards, expected)


# ---------------------------------------------------------------- brute force
def _graph_from_dense(A):
    m, n = A.shape
    r, c = np.nonzero(A)
    return synth.from_pairs(m, n, r, c)


def test_exhaustive_3x3_and_sampled_4x4():
    """Every 3x3 pattern, and 3000 random 4x4 patterns: MM = max over permutations
    sigma of #{i : A[i, sigma(i)] = 1} (a square pattern's maximum matching
    extends to a permutation)."""
    perms3 = np.array(list(itertools.permutations(range(3))))
    for mask in range(1 << 9):
        A = np.array([(mask >> b) & 1 for b in range(9)], dtype=np.int8).reshape(3, 3)
        mm = int(A[np.arange(3)[None, :], perms3].sum(1).max())
        assert_all(_graph_from_dense(A), mm)
    rng = np.random.default_rng(7)
    perms4 = np.array(list(itertools.permutations(range(4))))
    for _ in range(3000):
        A = (rng.random((4, 4)) < rng.random()).astype(np.int8)
        mm = int(A[np.arange(4)[None, :], perms4].sum(1).max())
        assert_all(_graph_from_dense(A), mm)


def test_brute_force_subsets_small():
    """Random graphs with <= 12 edges: enumerate all edge subsets."""
    rng = np.random.default_rng(11)
    for t in range(300):
        m, n = rng.integers(1, 7, 2)
        k = int(rng.integers(0, 13))
        r = rng.integers(0, m, k)
        c = rng.integers(0, n, k)
        g = synth.from_pairs(int(m), int(n), r, c)
        assert g.nnz <= 12
        assert_all(g, oracle.brute_force_subsets(g), shrink_min=int(rng.choice([1, 2, 512])))


def test_brute_force_dp_denser():
    rng = np.random.default_rng(12)
    for t in range(150):
        m, n = int(rng.integers(1, 11)), int(rng.integers(1, 13))
        g = synth.random_small(m, n, float(rng.uniform(0.05, 0.6)), int(rng.integers(1 << 30)))
        assert_all(g, oracle.brute_force_dp(g), k=float(rng.choice([0.3, 0.7, 2.0])))


# ---------------------------------------------------------------- closed forms
@pytest.mark.parametrize("a,b", [(0, 0), (0, 3), (3, 0), (1, 1), (1, 5), (5, 1), (4, 4), (7, 3), (3, 7), (50, 30)])
def test_complete_bipartite(a, b):
    g = synth.complete(a, b)
    assert_all(g, min(a, b))


@pytest.mark.parametrize("k", list(range(1, 31)) + [201, 1000])
def test_paths(k):
    assert_all(synth.path(k), k // 2)


@pytest.mark.parametrize("k", [1, 2, 3, 10, 99, 1000])
def test_even_cycles(k):
    assert_all(synth.cycle(k), k)


@pytest.mark.parametrize("leaves", [0, 1, 2, 17])
def test_stars(leaves):
    assert_all(synth.star(leaves), min(1, leaves))


@pytest.mark.parametrize("s", range(2, 12))
def test_grid_double_cover(s):
    assert_all(synth.grid_double_cover(s), s * s - (s % 2))


@pytest.mark.parametrize("n,noise,seed", [(10, 3, 1), (1000, 5000, 2), (20000, 40000, 3)])
def test_permutation_plus_noise(n, noise, seed):
    assert_all(synth.permutation_noise(n, noise, seed), n)


@pytest.mark.parametrize("n,t,d", [(200, 20, 5), (1000, 50, 17), (5000, 300, 120)])
def test_hall_violator(n, t, d):
    g = synth.hall_violator(n, t, d, seed=n + t + d)
    assert_all(g, n - d)


def test_disjoint_union_of_pinned_pieces():
    parts = [synth.complete(5, 3), synth.path(11), synth.cycle(40), synth.star(9), synth.grid_double_cover(7),
             synth.permutation_noise(500, 700, 4), synth.hall_violator(300, 30, 9, 5), synth.complete(0, 4)]
    g = synth.disjoint_union(parts, seed=9)
    assert g.mm == sum(p.mm for p in parts)
    assert_all(g, g.mm)


def test_banded_and_road_closed_forms():
    """C2's full diagonal and C3's planted dominoes fix MM at any size."""
    g2 = synth.config("C2", scale=0.01)
    assert g2.mm == g2.n
    assert_all(g2, g2.n)
    g3 = synth.config("C3", scale=0.001)
    assert g3.mm == g3.n
    c, rm, cm, _ = oracle.pr_fifo(g3)
    assert c == g3.n


# ---------------------------------------------------------------- third-party pin
def _scipy_mm(g):
    from scipy.sparse import csr_matrix
    from scipy.sparse.csgraph import maximum_bipartite_matching

    A = csr_matrix((np.ones(g.nnz), g.indices, g.indptr), shape=(g.m, g.n))
    return int((maximum_bipartite_matching(A, perm_type="column") >= 0).sum())


@pytest.mark.parametrize("name,scale", [("C1", 1.0), ("C2", 0.02), ("C3", 0.004), ("C4", 1 / 256), ("C5", 1 / 64)])
def test_configs_against_scipy(name, scale):
    g = synth.config(name, scale)
    mm = _scipy_mm(g)
    if g.mm is not None:
        assert mm == g.mm
    c1, rm, cm, _ = oracle.pr_fifo(g)
    c2, _, _ = oracle.hopcroft_karp(g)
    c3, _, _, _ = oracle.gpr_serial(g)
    assert c1 == c2 == c3 == mm
    assert oracle.konig_cover(g, rm, cm)[0] == mm


# ---------------------------------------------------------------- checkers
def test_check_matching_rejects_invalid():
    g = synth.complete(3, 3)
    ok_r, ok_c = np.array([0, 1, 2]), np.array([0, 1, 2])
    assert oracle.check_matching(g, ok_r, ok_c) == 3
    assert oracle.check_matching(g, [0, 0, -1], [0, -1, -1]) == -4      # non-injective rows
    assert oracle.check_matching(g, [0, 1, 2], [1, 0, 2]) == -4          # not inverse
    assert oracle.check_matching(g, [5, -1, -1], [-1, -1, -1]) == -1     # out of range
    assert oracle.check_matching(g, [-1, -1, -1], [0, -1, -1]) == -4     # column claims unmatched row
    p = synth.path(4)  # rows {0,1}, cols {0,1}; edges r0-c0, r1-c0, r1-c1
    assert oracle.check_matching(p, [1, -1], [-1, 0]) == -2              # r0-c1 is not an edge


def test_konig_rejects_non_maximum():
    g = synth.path(4)  # r0-c0, r1-c0, r1-c1 ; MM = 2
    size, _, _ = oracle.konig_cover(g, [-1, 0], [1, -1])  # |M| = 1, augmenting path r0-c0-r1-c1
    assert size == -1
    size, cr, cc = oracle.konig_cover(g, [0, 1], [0, 1])
    assert size == 2


# ---------------------------------------------------------------- GR labels
def _random_mu(g, rng, stale=True):
    """A matching plus GPU-style column noise: stale column entries and -2."""
    c, rm, cm = oracle.hopcroft_karp(g, init="empty")
    rm, cm = rm.copy(), cm.copy()
    # drop a random subset of pairs
    for u in range(g.m):
        if rm[u] >= 0 and rng.random() < 0.4:
            v = rm[u]
            rm[u] = -1
            cm[v] = -1
            if stale and rng.random() < 0.5:
                cm[v] = u  # stale column pointer: mu(mu(v)) != v
    if stale:
        for v in range(g.n):
            if cm[v] == -1 and rng.random() < 0.2:
                cm[v] = -2  # dead marker
    return rm, cm


def test_global_relabel_equals_bellman_ford():
    """GR labels = shortest alternating distances computed by
    Bellman-Ford relaxation (no queue, no levels); maxLevel = deepest row + 2."""
    rng = np.random.default_rng(21)
    for t in range(200):
        m, n = int(rng.integers(1, 25)), int(rng.integers(1, 25))
        g = synth.random_small(m, n, float(rng.uniform(0.03, 0.3)), int(rng.integers(1 << 30)))
        rm, cm = _random_mu(g, rng)
        pr, pc, ml, rf = oracle.global_relabel(g, rm, cm)
        dr, dc = oracle.alternating_distances(g, rm, cm)
        assert np.array_equal(pr, dr) and np.array_equal(pc, dc)
        finite = dr[dr < m + n]
        assert ml == (int(finite.max()) if finite.size else 0) + 2
        unmatched_col = np.array([not (cm[v] > -1 and rm[cm[v]] == v) for v in range(n)], bool)
        assert rf == int(((dc < m + n) & unmatched_col).sum())
        # parity: finite row labels even, finite column labels odd
        assert np.all(finite % 2 == 0)
        assert np.all(dc[dc < m + n] % 2 == 1)


def test_global_relabel_certifies_maximum():
    """On a maximum matching no unmatched column is reachable (Berge)."""
    for g in [synth.config("C1", 0.2), synth.hall_violator(400, 40, 11, 3), synth.config("C4", 1 / 1024)]:
        c, rm, cm = oracle.hopcroft_karp(g)
        _, pc, _, rf = oracle.global_relabel(g, rm, cm)
        assert rf == 0
        _, rm0, cm0 = oracle.cheap_match(g)
        if oracle.check_matching(g, rm0, cm0) < c:
            assert oracle.global_relabel(g, rm0, cm0)[3] > 0


# ---------------------------------------------------------------- G-PR simulator options
@pytest.mark.parametrize("k,fixed,shrink,dead_skip", [
    (0.3, False, 512, False), (0.7, False, 512, False), (2.0, False, 512, True), (10, True, -1, False),
    (50, True, 1, True), (0.7, False, 0, True), (1.5, False, 2, False)])
def test_gpr_serial_variants(k, fixed, shrink, dead_skip):
    rng = np.random.default_rng(int(k * 10) + shrink)
    graphs = [synth.config("C1", 0.3), synth.hall_violator(600, 50, 13, 2), synth.config("C2", 0.003),
              synth.config("C3", 0.0005), synth.config("C4", 1 / 2048), synth.complete(30, 20)]
    for _ in range(20):
        graphs.append(synth.random_small(int(rng.integers(1, 40)), int(rng.integers(1, 40)),
                                         float(rng.uniform(0.02, 0.2)), int(rng.integers(1 << 30))))
    for g in graphs:
        mm = oracle.hopcroft_karp(g)[0]
        for init in ("greedy", "empty"):
            c, rm, cm, st = oracle.gpr_serial(g, k=k, gr_fixed=fixed, shrink_min=shrink, dead_skip=dead_skip,
                                              init=init)
            assert c == mm, (g.name, init, c, mm, st)
            assert oracle.check_matching(g, rm, cm) == mm
            if g.mm == g.n == g.m:
                # perfect matching: FIXMATCHING has nothing to fix
                assert np.all(cm >= 0)


def test_pr_fifo_k_insensitive():
    g = synth.config("C2", 0.005)
    for k in (0.05, 0.5, 1.0, 2.0, 100.0):
        c, rm, cm, st = oracle.pr_fifo(g, k=k)
        assert c == g.n


@pytest.mark.slow
@pytest.mark.parametrize("name", ["C1", "C2", "C3", "C5"])
def test_full_size_oracles_agree(name):
    g = synth.config(name)
    csc = oracle.transpose(g)
    c1, rm, cm, _ = oracle.pr_fifo(g, csc=csc)
    c2, _, _ = oracle.hopcroft_karp(g, csc=csc)
    assert c1 == c2
    if g.mm is not None:
        assert c1 == g.mm
    assert oracle.konig_cover(g, rm, cm)[0] == c1


# ---------------------------------------------------------------- gap relabel (reading R14)
def test_gap_hand_examples():
    """Worked by hand from reading R14: INF = m+n."""
    g, pr, pc = oracle.gap_relabel(3, 2, [0, 2, 4], [1, 3])  # INF 5, labels 0..4 all present
    assert g == -1 and list(pr) == [0, 2, 4] and list(pc) == [1, 3]
    g, pr, pc = oracle.gap_relabel(3, 2, [0, 4, 9], [1, 3])  # label 2 empty, L_max 4
    assert g == 2 and list(pr) == [0, 5, 5] and list(pc) == [1, 5]
    g, pr, pc = oracle.gap_relabel(2, 2, [2, 4], [1, 3])  # no label 0: no unmatched row left
    assert g == 0 and list(pr) == [4, 4] and list(pc) == [4, 4]
    g, pr, pc = oracle.gap_relabel(2, 2, [0, -1], [1, 7])  # negatives / >= INF are infinite
    assert g == -1 and list(pr) == [0, 4] and list(pc) == [1, 4]


def test_gap_is_noop_on_exact_labels():
    """BFS layers are contiguous, so exact GR labels never contain a gap."""
    rng = np.random.default_rng(31)
    for t in range(100):
        m, n = int(rng.integers(1, 40)), int(rng.integers(1, 40))
        g = synth.random_small(m, n, float(rng.uniform(0.03, 0.3)), int(rng.integers(1 << 30)))
        rm, cm = _random_mu(g, rng)
        pr, pc, _, _ = oracle.global_relabel(g, rm, cm)
        gl, pr2, pc2 = oracle.gap_relabel(g.m, g.n, pr, pc)
        assert gl == -1 and np.array_equal(pr, pr2) and np.array_equal(pc, pc2)


def test_gpr_serial_with_gap_stays_exact():
    """Soundness pin: G-PR with gap relabelling (R14) still reaches the maximum
    cardinality (HK) -- an unsound gap would kill an augmentable column."""
    rng = np.random.default_rng(41)
    total_gaps = 0
    graphs = [synth.config("C4", 1 / 2048), synth.config("C1", 0.3), synth.hall_violator(900, 60, 21, 4)]
    for _ in range(60):
        m, n = int(rng.integers(2, 60)), int(rng.integers(2, 60))
        graphs.append(synth.random_small(m, n, float(rng.uniform(0.02, 0.2)), int(rng.integers(1 << 30))))
    for g in graphs:
        mm = oracle.hopcroft_karp(g)[0]
        for k in (0.7, 3.0, 10.0):
            c, rm, cm, st = oracle.gpr_serial(g, k=k, gap=True)
            assert c == mm, (g.name, k, c, mm, st)
            assert oracle.check_matching(g, rm, cm) == mm
            total_gaps += st["gaps"]
    assert total_gaps > 0  # the gap path was exercised
