"""GPU parity tests (-m gpu): the CUDA path through the C ABI against the CPU oracle.

* GR labels (deterministic): bit-exact psi_row, psi_col, maxLevel and the
  reached-unmatched count against oracle.global_relabel (Alg. 2 / Alg. 4-5).
* Full solves: the cardinality is unique -> bit-exact against the oracle
  (Hopcroft-Karp == PR-FIFO) or the closed form; the matching itself is not
  unique -> checked valid (pairs are edges, mates mutual, injective) and
  certified maximum by a Konig cover of equal size computed on the host.
"""
import numpy as np
import pytest

import oracle
import synth

torch = pytest.importorskip("torch")
pytestmark = pytest.mark.gpu

import paper_conf_icpp_devecikuc13_b200 as pkg  # noqa: E402

DEV = "cuda:0"


def dev(g):
    return torch.from_numpy(np.ascontiguousarray(g.indptr)).to(DEV), torch.from_numpy(
        np.ascontiguousarray(g.indices)).to(DEV)


def check_solve(g, mm=None, **opts):
    ip, ix = dev(g)
    mt = pkg.Matcher(ip, ix, g.m, g.n, **opts)
    card, rm, cm = mt.solve()
    st = mt.stats()
    mt.close()
    rm, cm = rm.cpu().numpy(), cm.cpu().numpy()
    if mm is None:
        mm = g.mm if g.mm is not None else oracle.hopcroft_karp(g)[0]
    assert card == mm, (g.name, opts, card, mm, st)
    assert oracle.check_matching(g, rm, cm) == card, (g.name, opts)
    size, _, _ = oracle.konig_cover(g, rm, cm)
    assert size == card, (g.name, opts, size)
    assert st["card"] == card and st["guard_reactivated"] >= 0
    return card, st


# ---------------------------------------------------------------- GR, bit-exact
def _noisy_matching(g, rng):
    c, rm, cm = oracle.hopcroft_karp(g, init="empty")
    rm, cm = rm.copy(), cm.copy()
    for u in np.nonzero(rm >= 0)[0]:
        if rng.random() < 0.3:
            v = rm[u]
            rm[u] = -1
            cm[v] = u if rng.random() < 0.5 else -1  # stale column pointer or unmatched
    dead = (cm == -1) & (rng.random(g.n) < 0.2)
    cm[dead] = -2
    return rm.astype(np.int32), cm.astype(np.int32)


GR_GRAPHS = [
    lambda: synth.config("C1", 0.2), lambda: synth.config("C2", 0.01), lambda: synth.config("C3", 0.002),
    lambda: synth.config("C4", 1 / 512), lambda: synth.config("C5", 1 / 256), lambda: synth.complete(40, 25),
    lambda: synth.path(2001), lambda: synth.hall_violator(2000, 100, 31, 3),
]


@pytest.mark.parametrize("bu", [32, 0, 1], ids=["bu32", "topdown", "bottomup"])
@pytest.mark.parametrize("gi", range(len(GR_GRAPHS)))
def test_global_relabel_bit_exact(gi, bu):
    """Top-down, bottom-up (direction-optimising) and mixed BFS levels must all give
    the oracle's labels."""
    g = GR_GRAPHS[gi]()
    rng = np.random.default_rng(gi)
    ip, ix = dev(g)
    mt = pkg.Matcher(ip, ix, g.m, g.n, bu_div=bu, gr_early=0)  # complete GR (early stop: test_gpu_units)
    for trial in range(3):
        if trial == 0:
            _, rm, cm = oracle.cheap_match(g)
        elif trial == 1:
            rm, cm = _noisy_matching(g, rng)
        else:
            rm, cm = np.full(g.m, -1, np.int32), np.full(g.n, -1, np.int32)
        ml, pr, pc, rf = mt.global_relabel(torch.from_numpy(rm).to(DEV), torch.from_numpy(cm).to(DEV))
        epr, epc, eml, erf = oracle.global_relabel(g, rm, cm)
        assert np.array_equal(pr.cpu().numpy(), epr), (g.name, trial)
        assert np.array_equal(pc.cpu().numpy(), epc), (g.name, trial)
        assert ml == eml and rf == erf, (g.name, trial, ml, eml, rf, erf)
    mt.close()


# ---------------------------------------------------------------- solves
SOLVE_GRAPHS = [
    ("C1", lambda: synth.config("C1")), ("C2s", lambda: synth.config("C2", 0.01)),
    ("C3s", lambda: synth.config("C3", 0.002)), ("C4s", lambda: synth.config("C4", 1 / 256)),
    ("C5s", lambda: synth.config("C5", 1 / 64)), ("hall", lambda: synth.hall_violator(5000, 300, 77, 1)),
    ("K64x40", lambda: synth.complete(64, 40)), ("P1001", lambda: synth.path(1001)),
    ("C2000", lambda: synth.cycle(1000)), ("grid9", lambda: synth.grid_double_cover(9)),
    ("union", lambda: synth.disjoint_union([synth.complete(7, 5), synth.path(99), synth.star(12),
                                            synth.hall_violator(900, 40, 13, 2), synth.cycle(77)], seed=3)),
]


@pytest.mark.parametrize("name,mk", SOLVE_GRAPHS, ids=[s[0] for s in SOLVE_GRAPHS])
def test_solve_default(name, mk):
    check_solve(mk())


OPTION_SETS = [
    dict(k=0.3), dict(k=2.0), dict(gr_strategy="fixed", k=10), dict(gr_strategy="fixed", k=50), dict(shrink_min=-1),
    dict(shrink_min=1), dict(compact_every=1), dict(init="empty"), dict(final_check=0), dict(dead_skip=0),
    dict(tail_max=0), dict(tail_max=100000), dict(grid_ctas=1), dict(grid_ctas=7), dict(gap=1), dict(tail_ctas=1),
    dict(tail_ctas=2), dict(tail_ctas=16), dict(compact_adapt=0), dict(grid_ctas=16, tail_ctas=16), dict(tail_f=64),
    dict(tail_max=4096, tail_f=100000), dict(tail_max=32, tail_f=32), dict(gr_early=1), dict(gr_early=1, tail_max=0),
    dict(gr_early=1, k=3.0), dict(gr_early=0), dict(variant=1), dict(variant=1, gr_early=0, k=0.3), dict(bu_div=0),
    dict(bu_div=1), dict(bu_div=100000), dict(scan_rot=1), dict(tail_chain=0), dict(tail_chain=1),
    dict(tail_chain=1 << 30), dict(tail_chain=4, tail_max=16), dict(tail_chain=64, k=3.0), dict(grid_chain=0),
    dict(grid_chain=1), dict(grid_chain=1 << 30), dict(grid_chain=4, tail_max=0), dict(grid_chain=0, tail_chain=0),
    dict(grid_chain=1000, tail_max=0, k=0.1), dict(gr_target=1.0), dict(gr_target=0.8, gr_target_min=0),
    dict(gr_target=0.3, k=0.3, gr_target_min=0), dict(gr_target=0.01, tail_max=0, gr_target_min=16),
    dict(gr_concurrent=48), dict(gr_concurrent=16, k=3.0), dict(gr_concurrent=100, tail_max=0),
    dict(gr_concurrent=1, grid_chain=0, tail_chain=0),
    dict(gr_window=4), dict(gr_window=8, gr_window_max=1 << 30, tail_max=0), dict(gr_window=16, k=0.1),
]


@pytest.mark.parametrize("opts", OPTION_SETS, ids=lambda o: ",".join(f"{k}={v}" for k, v in o.items()))
def test_solve_options(opts):
    for g in (synth.config("C1", 0.5), synth.config("C2", 0.005), synth.config("C3", 0.001),
              synth.config("C4", 1 / 1024), synth.hall_violator(3000, 150, 41, 9)):
        check_solve(g, **opts)


def test_given_initial_matching():
    g = synth.config("C2", 0.01)
    _, rm0, cm0 = oracle.cheap_match(g)
    ip, ix = dev(g)
    mt = pkg.Matcher(ip, ix, g.m, g.n, init="given")
    rm = torch.from_numpy(rm0.astype(np.int32)).to(DEV)
    cm = torch.from_numpy(cm0.astype(np.int32)).to(DEV)
    card, rm, cm = mt.solve(rm, cm)
    assert mt.stats()["init_card"] == int((rm0 >= 0).sum())
    assert card == g.n
    assert oracle.check_matching(g, rm.cpu().numpy(), cm.cpu().numpy()) == card


@pytest.mark.parametrize("final_check", [1, 0])
@pytest.mark.parametrize("drop_cols", [False, True])
def test_stale_rows_repaired(drop_cols, final_check):
    """R27: rows whose column does not point back (the state a late chain store can
    leave) are repaired before the guard GR.  An initial matching with such rows
    reproduces it deterministically: drop_cols=False -> the column words point to
    rows that do not point back (the column is re-attached to its row or the row is
    freed); drop_cols=True -> the column words are -1.  final_check=0 (no guard, no
    repair pass): FIXMATCHING reports stale rows unmatched, so the output is still
    a valid matching, not necessarily maximum."""
    g = synth.config("C2", 0.01)
    _, rm0, cm0 = oracle.cheap_match(g)
    rm0 = rm0.astype(np.int32).copy()
    cm0 = cm0.astype(np.int32).copy()
    rng = np.random.default_rng(7)
    matched = np.nonzero(rm0 >= 0)[0]
    stale = rng.choice(matched, size=64, replace=False)
    for u in stale:
        c = rm0[u]
        cm0[c] = -1 if drop_cols else (u + 1) % g.m  # row (u+1) % m does not hold c
    ip, ix = dev(g)
    mt = pkg.Matcher(ip, ix, g.m, g.n, init="given", final_check=final_check)
    card, rm, cm = mt.solve(torch.from_numpy(rm0).to(DEV), torch.from_numpy(cm0).to(DEV))
    rm, cm = rm.cpu().numpy(), cm.cpu().numpy()
    assert oracle.check_matching(g, rm, cm) == card
    if final_check:
        assert card == g.n  # C2 has a perfect matching (closed form)
        assert oracle.konig_cover(g, rm, cm)[0] == card


@pytest.mark.parametrize("rate", [2048, 16384, 49152])
@pytest.mark.parametrize("chains", [0, 1])
def test_perturb_fault_injection(rate, chains):
    """SURVEY.md 5 fault injection: option perturb drops the row store of a share of
    the paper's pushes (the state a lost race for the row leaves).  The
    column stays active by reading R1 and is pushed again; the solve must still
    return a valid maximum matching with a Koenig certificate.  With a high rate the
    paper's pushes need several tries, so the push count exceeds the unperturbed one."""
    extra = {} if chains else dict(grid_chain=0, tail_chain=0)
    for g in (synth.config("C1", 0.5), synth.config("C2", 0.005), synth.hall_violator(3000, 150, 41, 9)):
        _, st0 = check_solve(g, **extra)
        _, st = check_solve(g, perturb=rate, **extra)
        if rate >= 16384 and not chains:
            assert st["pushes"] > st0["pushes"], (g.name, st0["pushes"], st["pushes"])


def test_perturb_without_guard_is_valid():
    """perturb with the exactness guard off: FIXMATCHING (R15) still
    reports a valid matching (rows are authoritative)."""
    g = synth.config("C2", 0.005)
    ip, ix = dev(g)
    mt = pkg.Matcher(ip, ix, g.m, g.n, perturb=16384, final_check=0, grid_chain=0, tail_chain=0)
    card, rm, cm = mt.solve()
    assert oracle.check_matching(g, rm.cpu().numpy(), cm.cpu().numpy()) == card


def test_edge_cases():
    check_solve(synth.from_pairs(0, 0, [], []), 0)
    check_solve(synth.from_pairs(5, 0, [], []), 0)
    check_solve(synth.from_pairs(0, 5, [], []), 0)
    check_solve(synth.from_pairs(4, 6, [], []), 0)
    check_solve(synth.from_pairs(1, 1, [0], [0]), 1)
    check_solve(synth.star(1000), 1)
    check_solve(synth.complete(1, 3000), 1)
    check_solve(synth.from_pairs(3000, 50, np.arange(3000), np.arange(3000) % 50), 50)  # m >> n
    check_solve(synth.from_pairs(50, 3000, np.arange(3000) % 50, np.arange(3000)), 50)  # n >> m


def test_unsorted_duplicate_adjacency():
    """The ABI accepts unsorted lists with duplicates (tie-breaks only)."""
    g = synth.config("C1", 0.3)
    rng = np.random.default_rng(5)
    idx = g.indices.copy()
    for u in range(g.m):
        s, e = g.indptr[u], g.indptr[u + 1]
        rng.shuffle(idx[s:e])
    # duplicate every 7th entry of each row (append a copy)
    rows, cols = [], []
    for u in range(g.m):
        lst = idx[g.indptr[u]: g.indptr[u + 1]].tolist()
        lst = lst + lst[::7]
        rows += [u] * len(lst)
        cols += lst
    indptr = np.zeros(g.m + 1, np.int32)
    np.add.at(indptr, np.array(rows) + 1, 1)
    indptr = np.cumsum(indptr).astype(np.int32)
    gd = synth.Graph(g.m, g.n, indptr, np.array(cols, np.int32), "dup")
    mm = oracle.hopcroft_karp(g)[0]
    ip, ix = dev(gd)
    card, rm, cm = pkg.solve(ip, ix, g.m, g.n)
    assert card == mm
    assert oracle.check_matching(g, rm.cpu().numpy(), cm.cpu().numpy()) == mm


def test_rejects_malformed_csr():
    ip = torch.tensor([0, 2, 1], dtype=torch.int32, device=DEV)  # decreasing
    ix = torch.tensor([0, 1], dtype=torch.int32, device=DEV)
    with pytest.raises(pkg.MCMError):
        pkg.Matcher(ip, ix, 2, 2)
    ip = torch.tensor([0, 1, 2], dtype=torch.int32, device=DEV)
    ix = torch.tensor([0, 7], dtype=torch.int32, device=DEV)  # column out of range
    with pytest.raises(pkg.MCMError):
        pkg.Matcher(ip, ix, 2, 2)
    ip = torch.tensor([1, 1, 2], dtype=torch.int32, device=DEV)  # indptr[0] != 0
    with pytest.raises(pkg.MCMError):
        pkg.Matcher(ip, torch.tensor([0, 1], dtype=torch.int32, device=DEV), 2, 2)
    ip = torch.tensor([0, 1, 2], dtype=torch.int32, device=DEV)
    ix = torch.tensor([0, 1], dtype=torch.int32, device=DEV)
    for bad in (0.0, -0.5, 1.5, float("nan")):  # gr_target outside (0, 1]
        with pytest.raises(pkg.MCMError):
            pkg.Matcher(ip, ix, 2, 2, gr_target=bad)


def test_match_host_end_to_end():
    """mcm_match_host: host CSR in, host matching out (the bench's e2e path)."""
    for g in (synth.config("C1", 0.5), synth.config("C2", 0.01), synth.hall_violator(3000, 150, 41, 9),
              synth.from_pairs(4, 6, [], []), synth.from_pairs(0, 0, [], [])):
        ip = torch.from_numpy(np.ascontiguousarray(g.indptr)).pin_memory()
        ix = torch.from_numpy(np.ascontiguousarray(g.indices)).pin_memory()
        card, rm, cm, st = pkg.match_host(ip, ix, g.m, g.n)
        mm = g.mm if g.mm is not None else oracle.hopcroft_karp(g)[0]
        assert card == mm and st["card"] == card, (g.name, card, mm)
        assert not rm.is_cuda and not cm.is_cuda
        assert oracle.check_matching(g, rm.numpy(), cm.numpy()) == card
        assert oracle.konig_cover(g, rm.numpy(), cm.numpy())[0] == card
    # pageable host memory works too; malformed CSR is rejected before any solve
    g = synth.config("C1", 0.2)
    card, rm, cm, _ = pkg.match_host(torch.from_numpy(g.indptr.copy()), torch.from_numpy(g.indices.copy()), g.m, g.n,
                                     rmatch=torch.empty(g.m, dtype=torch.int32), cmatch=torch.empty(g.n, dtype=torch.int32))
    assert card == oracle.hopcroft_karp(g)[0]
    with pytest.raises(pkg.MCMError):
        pkg.match_host(torch.tensor([0, 1, 2], dtype=torch.int32), torch.tensor([0, 7], dtype=torch.int32), 2, 2)


def test_concurrent_solves_on_streams():
    """Several persistent solves at once (one host thread, stream and handle each,
    a quarter of the CTAs each): the batch mode of bench.py --config C5."""
    import threading

    graphs = [synth.config("C5", 1 / 64, index=i) for i in range(4)] + [synth.config("C2", 0.01)]
    out = [None] * len(graphs)

    def run(j):
        g = graphs[j]
        st = torch.cuda.Stream()
        ip, ix = dev(g)
        torch.cuda.synchronize()
        mt = pkg.Matcher(ip, ix, g.m, g.n, stream=st, grid_ctas=37)
        card, rm, cm = mt.solve(stream=st)
        st.synchronize()
        out[j] = (card, rm.cpu().numpy(), cm.cpu().numpy())
        mt.close()

    ths = [threading.Thread(target=run, args=(j,)) for j in range(len(graphs))]
    for t in ths:
        t.start()
    for t in ths:
        t.join()
    for g, (card, rm, cm) in zip(graphs, out):
        mm = g.mm if g.mm is not None else oracle.hopcroft_karp(g)[0]
        assert card == mm, (g.name, card, mm)
        assert oracle.check_matching(g, rm, cm) == card


def test_race_stress():
    """Every column races for the same rows (K_{a,b}, empty M0), repeated."""
    for g in (synth.complete(128, 128), synth.complete(300, 40), synth.complete(40, 300), synth.grid_double_cover(30)):
        for rep in range(10):
            check_solve(g, init="empty")
    for seed in range(30):
        g = synth.random_small(200, 200, 0.02, seed)
        check_solve(g, init="empty", k=0.3)


def test_matcher_reuse_is_deterministic_in_card():
    g = synth.config("C3", 0.004)
    ip, ix = dev(g)
    mt = pkg.Matcher(ip, ix, g.m, g.n)
    cards = {mt.solve()[0] for _ in range(5)}
    assert cards == {g.n}
    mt.close()


# ---------------------------------------------------------------- full-size configs
@pytest.mark.parametrize("name", ["C1", "C2", "C3", "C4", "C5"])
def test_full_size_config(name):
    """BASELINE.json sizes in the bench launch configuration (defaults, all CTAs):
    closed-form MM (C2, C3) or the oracle's (C1, C4, C5); validity; Konig."""
    g = synth.config(name)
    mm = g.mm
    if mm is None:
        mm = oracle.hopcroft_karp(g)[0]
    check_solve(g, mm)


# ---------------------------------------------------------------- gap relabel, bit-exact
def test_gap_relabel_bit_exact():
    """mcm_gap_relabel (the routine the solve runs with gap=1) against the oracle's
    reading R14 on label arrays with and without holes."""
    rng = np.random.default_rng(77)
    for t in range(12):
        g = synth.config("C1", 0.05) if t % 2 else synth.random_small(300, 200, 0.02, t)
        ip, ix = dev(g)
        mt = pkg.Matcher(ip, ix, g.m, g.n)
        INF = g.m + g.n
        top = int(rng.integers(2, 60))
        pr = rng.integers(0, top, g.m).astype(np.int32)
        pc = rng.integers(0, top, g.n).astype(np.int32)
        hole = int(rng.integers(0, top))
        if t % 3 != 2:  # punch a hole (t % 3 == 2: maybe none)
            pr[pr == hole] = hole + 1
            pc[pc == hole] = hole + 1
        pr[rng.random(g.m) < 0.1] = INF + 3
        pc[rng.random(g.n) < 0.1] = -1
        gl, dpr, dpc = mt.gap_relabel(torch.from_numpy(pr), torch.from_numpy(pc))
        egl, epr, epc = oracle.gap_relabel(g.m, g.n, pr, pc)
        assert gl == egl, (t, gl, egl)
        assert np.array_equal(dpr.cpu().numpy(), epr) and np.array_equal(dpc.cpu().numpy(), epc), t
        mt.close()


def test_gap_solves_exact_without_guard():
    """Soundness on the GPU: with gap relabelling on and the exactness guard off the
    cardinality is still the maximum (an unsound gap would kill augmentable columns)."""
    graphs = [synth.config("C1"), synth.config("C4", 1 / 128), synth.hall_violator(5000, 300, 77, 1),
              synth.from_pairs(3000, 5000, np.arange(9000) % 3000, (np.arange(9000) * 7) % 5000),
              synth.config("C3", 0.002)]
    for g in graphs:
        card, st = check_solve(g, gap=1, final_check=0)
        card2, st2 = check_solve(g, gap=1, final_check=1)
        assert st2["guard_reactivated"] == 0


# ---------------------------------------------------------------- serial mode, bit-exact trajectory
SERIAL_CASES = [
    (lambda: synth.config("C1", 0.3), {}), (lambda: synth.config("C2", 0.003), {}),
    (lambda: synth.config("C3", 0.0005), {}), (lambda: synth.config("C4", 1 / 2048), {}),
    (lambda: synth.hall_violator(800, 60, 17, 3), {}), (lambda: synth.complete(30, 20), {}),
    (lambda: synth.config("C1", 0.3), dict(k=2.0)), (lambda: synth.config("C1", 0.3), dict(gr_fixed=True, k=10)),
    (lambda: synth.config("C2", 0.003), dict(shrink_min=-1)), (lambda: synth.config("C4", 1 / 2048), dict(dead_skip=True)),
    (lambda: synth.config("C1", 0.3), dict(gap=True)), (lambda: synth.config("C4", 1 / 2048), dict(gap=True)),
]


@pytest.mark.parametrize("ci", range(len(SERIAL_CASES)))
def test_serial_mode_matches_simulator(ci):
    """With the slots processed in order by one thread (options serial=1, sorted
    CSC), the GPU run reproduces the oracle's serial simulator of Alg. 7/8/9
    (or_gpr_serial) exactly: final mu arrays, cardinality, loop / GR / push /
    dead / blocked / shrink counts.  Pins the fix, shrink, push, iA-guard,
    rollback, GR and GETITERGR logic of the CUDA path, not just its result."""
    mk, kw = SERIAL_CASES[ci]
    g = mk()
    csc = oracle.transpose(g)
    _, rm0, cm0 = oracle.cheap_match(g, csc)
    sim_kw = dict(k=kw.get("k", 0.7), gr_fixed=kw.get("gr_fixed", False), shrink_min=kw.get("shrink_min", 512),
                  dead_skip=kw.get("dead_skip", False), gap=kw.get("gap", False))
    card, srm, scm, st = oracle.gpr_serial(g, init=(rm0, cm0), csc=csc, **sim_kw)
    opts = dict(serial=1, sort_csc=1, init="given", final_check=0, k=sim_kw["k"],
                gr_strategy="fixed" if sim_kw["gr_fixed"] else "adaptive", shrink_min=sim_kw["shrink_min"],
                dead_skip=int(sim_kw["dead_skip"]), gap=int(sim_kw["gap"]))
    ip, ix = dev(g)
    mt = pkg.Matcher(ip, ix, g.m, g.n, **opts)
    rm = torch.from_numpy(rm0.astype(np.int32)).to(DEV)
    cm = torch.from_numpy(cm0.astype(np.int32)).to(DEV)
    gcard, grm, gcm = mt.solve(rm, cm)
    gst = mt.stats()
    mt.close()
    assert gcard == card
    assert np.array_equal(grm.cpu().numpy(), srm) and np.array_equal(gcm.cpu().numpy(), scm), g.name
    got = dict(loops=gst["loops"], grs=gst["gr_count"], levels=gst["gr_levels"], pushes=gst["pushes"],
               shrinks=gst["shrinks"], dead=gst["dead"], blocked=gst["blocked"], gaps=gst["gaps"])
    want = {k: st[k] for k in got}
    assert got == want, (g.name, kw, got, want)


def test_concurrent_gr_repeated():
    """NEXT-2 (gr_concurrent): the GR kernel and the push kernel race on the matching
    by design; repeated solves stay exact (the guard) and the GR kernel is always
    released (no solve hangs), also after a rejected input."""
    g = synth.config("C2", 0.05)
    ip, ix = dev(g)
    mt = pkg.Matcher(ip, ix, g.m, g.n, gr_concurrent=48)
    for _ in range(10):
        card, rm, cm = mt.solve()
        assert card == g.n
        assert oracle.check_matching(g, rm.cpu().numpy(), cm.cpu().numpy()) == card
    mt.close()
    _, rm0, cm0 = oracle.cheap_match(g)
    bad = rm0.astype(np.int32).copy()
    bad[0] = g.n  # out of range: MCM_EINVAL, the GR kernel must still exit
    mt = pkg.Matcher(ip, ix, g.m, g.n, gr_concurrent=48, init="given")
    with pytest.raises(pkg.MCMError):
        mt.solve(torch.from_numpy(bad).to(DEV), torch.from_numpy(cm0.astype(np.int32)).to(DEV))
    card, _, _ = mt.solve(torch.from_numpy(rm0.astype(np.int32)).to(DEV), torch.from_numpy(cm0.astype(np.int32)).to(DEV))
    assert card == g.n
    mt.close()
