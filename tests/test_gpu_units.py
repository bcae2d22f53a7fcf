"""GPU parity of the phases the production kernel runs, one phase at a time
(-m gpu), through the C ABI's mcm_unit_step / mcm_global_relabel /
mcm_initial_matching against the oracle's plain CPU functions.

* fix step (INITKRNL, Alg. 8) and SHRKRNL: the solve's
  fix_slots / fix_plain / compact_pass1-2 on the grid (1-slot and 4-slot batches,
  several tiles, ragged tails) and in the single-CTA tail (worklist in shared
  memory or in global memory): Ac, iA and the count / new length bit-exact.
* PUSHKRNL (Alg. 9): the solve's push / push_wide / scan / scan_cta on
  inputs whose active columns do not interact (synth.push_instance), so the
  parallel push is deterministic: every mu, psi, Ac, Ap entry and the push /
  blocked / dead counts bit-exact against oracle.pushkrnl.
* FIXMATCHING + |M|.
* GR as the solve runs it: single-CTA tail levels with a shared-memory frontier and
  the grid <-> tail hand-over (complete GR: every label bit-exact), and the early
  stop of R22 / R28 (labelled vertices exact, the rest valid lower bounds that keep
  the neighbourhood invariant).
* the device cheap matching M0 on its own: valid and maximal.
"""
import numpy as np
import pytest

import oracle
import synth

torch = pytest.importorskip("torch")
pytestmark = pytest.mark.gpu

import paper_conf_icpp_devecikuc13_b200 as pkg  # noqa: E402

DEV = "cuda:0"


def T(a):
    return torch.from_numpy(np.ascontiguousarray(a, dtype=np.int32)).to(DEV)


def H(t):
    return t.cpu().numpy()


def matcher(g, **opts):
    return pkg.Matcher(T(g.indptr), T(g.indices), g.m, g.n, **opts)


def random_state(m, n, ln, rng, loop=9):
    """A partial matching with the GPU's column noise (stale pointers, -2), random
    labels, iA marks around `loop`, and a worklist with duplicates and empty slots."""
    k = min(m, n) // 2
    rows = rng.choice(m, k, replace=False)
    cols = rng.choice(n, k, replace=False)
    mu_row = np.full(m, -1, np.int32)
    mu_col = np.full(n, -1, np.int32)
    mu_row[rows] = cols
    mu_col[cols] = rows
    drop = rng.random(k) < 0.25  # rows released, column pointer left stale
    mu_row[rows[drop]] = -1
    free = np.nonzero(mu_col == -1)[0]
    mu_col[free[rng.random(free.size) < 0.3]] = -2
    INF = m + n
    psi_row = rng.integers(0, INF + 1, m).astype(np.int32)
    psi_col = rng.integers(0, INF + 1, n).astype(np.int32)
    iA = rng.integers(loop - 3, loop + 1, n).astype(np.int32)
    Ac = rng.integers(-1, n, ln).astype(np.int32)
    Ap = rng.integers(-1, n, ln).astype(np.int32)
    Ap[rng.random(ln) < 0.4] = -1
    return mu_row, mu_col, psi_row, psi_col, iA, Ac, Ap


@pytest.fixture(scope="module")
def big():
    g = synth.uniform(260_000, 250_000, 4 * 250_000, 77, name="units")
    mt = matcher(g)
    yield g, mt
    mt.close()


@pytest.mark.parametrize("where", ["grid", "tail"])
@pytest.mark.parametrize("ln", [0, 1, 37, 511, 1024, 1025, 5000, 151_553, 240_000])
def test_unit_fix_and_shrink(big, where, ln):
    g, mt = big
    if where == "tail" and ln > 60_000:
        pytest.skip("the tail takes short worklists")
    rng = np.random.default_rng(ln + (where == "tail"))
    loop = 9
    st = random_state(g.m, g.n, ln, rng, loop)
    mu_row, mu_col, psi_row, psi_col, iA, Ac, Ap = st
    for unit in (["fix", "shrink"] if where == "grid" else ["shrink", "fix"]):
        d = [T(a) for a in st]
        r = mt.unit_step(unit, where, loop, *d)
        compacting = unit == "shrink" or where == "tail"  # the tail compacts at every fix step
        if compacting:
            en, eAc, eiA = oracle.shrkrnl(loop, mu_row, mu_col, Ac, Ap, iA)
            assert r == en, (unit, where, ln, r, en)
            assert np.array_equal(H(d[5])[:en], eAc), (unit, where, ln)
        else:
            ea, eAc, eiA = oracle.initkrnl(loop, mu_row, mu_col, Ac, Ap, iA)
            assert r == ea, (unit, where, ln, r, ea)
            assert np.array_equal(H(d[5]), eAc), (unit, where, ln)
        assert np.array_equal(H(d[4]), eiA), (unit, where, ln)
        assert np.array_equal(H(d[6]), Ap)  # the fix step never writes Ap
        assert np.array_equal(H(d[0]), mu_row) and np.array_equal(H(d[1]), mu_col)
        assert np.array_equal(H(d[2]), psi_row) and np.array_equal(H(d[3]), psi_col)


PUSH_CASES = [
    # (K active columns, seed, where, degree mix): tail and grid lane groups, warps,
    # CTA-wide scans (> 512 entries, more than HUGE_CTA per tile), and push_wide
    # (> 2 * 512 * 148 slots)
    (12, 1, "tail", None), (300, 2, "tail", None), (1500, 3, "tail", None),
    (40, 4, "grid", None), (3000, 5, "grid", None), (20_000, 6, "grid", ((0.8, 1, 8), (0.15, 9, 64), (0.05, 65, 700))),
    (160_000, 7, "grid", ((0.9, 1, 8), (0.09, 9, 64), (0.01, 65, 600))),
    (200, 8, "grid", ((0.2, 1, 4), (0.8, 513, 4000))),
]


@pytest.mark.parametrize("dead_skip", [1, 0])
@pytest.mark.parametrize("ci", range(len(PUSH_CASES)))
def test_unit_push(ci, dead_skip):
    K, seed, where, mix = PUSH_CASES[ci]
    kw = {} if mix is None else dict(deg_mix=mix)
    g, st = synth.push_instance(K, seed, **kw)
    loop = st["loop"]
    mt = matcher(g, sort_csc=1, dead_skip=dead_skip)  # CSC in row order = the oracle's transpose order (R11)
    d = dict(mu_row=T(st["mu_row"]), mu_col=T(st["mu_col"]), psi_row=T(st["psi_row"]), psi_col=T(st["psi_col"]),
             iA=T(st["iA"]), Ac=T(st["Ac"]), Ap=T(np.full(K, 12345 % max(g.n, 1), np.int32)))
    mt.unit_step("push", where, loop, d["mu_row"], d["mu_col"], d["psi_row"], d["psi_col"], d["iA"], d["Ac"], d["Ap"])
    sts = mt.stats()
    mt.close()
    e = oracle.pushkrnl(g, loop, st["mu_row"], st["mu_col"], st["psi_row"], st["psi_col"], st["iA"], st["Ac"],
                        dead_skip=bool(dead_skip))
    for k in ("mu_row", "mu_col", "psi_row", "psi_col", "Ac", "Ap"):
        got = H(d[k])
        bad = np.nonzero(got != e[k])[0]
        assert bad.size == 0, (K, where, k, bad[:5], got[bad[:5]], e[k][bad[:5]])
    assert np.array_equal(H(d["iA"]), st["iA"])  # PUSHKRNL never writes iA
    assert (sts["pushes"], sts["blocked"], sts["dead"]) == (e["pushes"], e["blocked"], e["dead"]), (sts, e)
    assert e["pushes"] > 0 and (K < 100 or (e["blocked"] > 0 and e["dead"] > 0))  # every branch exercised


@pytest.mark.parametrize("seed", range(4))
def test_unit_fixmatching(big, seed):
    g, mt = big
    rng = np.random.default_rng(100 + seed)
    mu_row, mu_col, psi_row, psi_col, iA, Ac, Ap = random_state(g.m, g.n, 3, rng)
    d = [T(a) for a in (mu_row, mu_col, psi_row, psi_col, iA, Ac, Ap)]
    card = mt.unit_step("fixmatching", "grid", 0, *d)
    ec, emc = oracle.fixmatching(g.m, g.n, mu_row, mu_col)
    assert card == ec
    assert np.array_equal(H(d[1]), emc) and np.array_equal(H(d[0]), mu_row)


def test_unit_rejects_out_of_range(big):
    g, mt = big
    rng = np.random.default_rng(5)
    st = list(random_state(g.m, g.n, 10, rng))
    st[5][3] = g.n  # Ac entry out of range
    with pytest.raises(pkg.MCMError):
        mt.unit_step("fix", "grid", 1, *[T(a) for a in st])
    st = list(random_state(g.m, g.n, 10, rng))
    st[0][7] = -3  # mu_row out of range
    with pytest.raises(pkg.MCMError):
        mt.unit_step("push", "tail", 1, *[T(a) for a in st])
    # the handle stays usable
    st = list(random_state(g.m, g.n, 10, rng))
    assert mt.unit_step("fix", "grid", 9, *[T(a) for a in st]) >= 0


# ---------------------------------------------------------------- GR as the solve runs it
GR_GRAPHS = [
    lambda: synth.config("C1", 0.2), lambda: synth.config("C2", 0.01), lambda: synth.config("C3", 0.002),
    lambda: synth.config("C4", 1 / 512), lambda: synth.config("C5", 1 / 256), lambda: synth.path(4001),
    lambda: synth.hall_violator(2000, 100, 31, 3),
]


def _matchings(g, rng):
    _, rm, cm = oracle.cheap_match(g)
    yield "cheap", rm, cm
    c, rm2, cm2 = oracle.hopcroft_karp(g, init="empty")
    rm2, cm2 = rm2.copy(), cm2.copy()
    for u in np.nonzero(rm2 >= 0)[0]:  # release pairs, leave stale column pointers and -2 marks
        if rng.random() < 0.05:
            v = rm2[u]
            rm2[u] = -1
            cm2[v] = u if rng.random() < 0.5 else -1
    cm2[(cm2 == -1) & (rng.random(g.n) < 0.1)] = -2
    yield "near-max", rm2.astype(np.int32), cm2.astype(np.int32)


TAIL_OPTS = [dict(tail_max=32, tail_f=128), dict(tail_max=32, tail_f=8), dict(tail_max=32, tail_f=100000),
             dict(tail_max=32, tail_f=4, bu_div=0), dict(tail_max=0),
             # windowed levels (R29): K levels per grid barrier, label-correcting inside a CTA;
             # gr_window_max 2^30 also sends wide levels through windows (local-queue overflow ->
             # dirty windows)
             dict(tail_max=32, tail_f=128, gr_window=4), dict(tail_max=0, gr_window=8, gr_window_max=1 << 30),
             dict(tail_max=32, tail_f=8, gr_window=2, gr_window_max=64, bu_div=0),
             dict(tail_max=0, gr_window=64, gr_window_max=1 << 30, bu_div=0)]


@pytest.mark.parametrize("oi", range(len(TAIL_OPTS)))
@pytest.mark.parametrize("gi", range(len(GR_GRAPHS)))
def test_relabel_tail_paths_bit_exact(gi, oi):
    """Complete GR through the solve's state machine (grid levels, single-CTA tail
    levels with the frontier in shared memory, hand-over both ways): every label,
    maxLevel and the reached-unmatched count equal the oracle's GR (Alg. 2/4/5)."""
    g = GR_GRAPHS[gi]()
    rng = np.random.default_rng(gi * 10 + oi)
    mt = matcher(g, gr_early=0, **TAIL_OPTS[oi])
    tail_seen = 0
    for name, rm, cm in _matchings(g, rng):
        ml, pr, pc, rf, info = mt.global_relabel(T(rm), T(cm), info=True)
        epr, epc, eml, erf = oracle.global_relabel(g, rm, cm)
        assert np.array_equal(H(pr), epr), (g.name, name, TAIL_OPTS[oi])
        assert np.array_equal(H(pc), epc), (g.name, name, TAIL_OPTS[oi])
        assert ml == eml and rf == erf, (g.name, name, ml, eml, rf, erf)
        assert info["floor_row"] == info["floor_col"] == g.m + g.n
        tail_seen += info["tail_levels"]
    mt.close()
    if TAIL_OPTS[oi].get("tail_max", 32) == 0:
        assert tail_seen == 0
    elif TAIL_OPTS[oi]["tail_f"] == 100000:  # every frontier fits the tail
        assert tail_seen > 0, (g.name, TAIL_OPTS[oi])


EARLY_OPTS = [dict(gr_target=1.0), dict(gr_target=0.6, gr_target_min=0), dict(gr_target=0.3, gr_target_min=0, tail_max=0),
              dict(gr_target=0.05, gr_target_min=16, tail_f=16),
              dict(gr_target=1.0, gr_window=4), dict(gr_target=0.3, gr_target_min=0, tail_max=0, gr_window=8,
                                                     gr_window_max=1 << 30)]


@pytest.mark.parametrize("oi", range(len(EARLY_OPTS)))
@pytest.mark.parametrize("gi", range(len(GR_GRAPHS)))
def test_relabel_early_stop_lower_bounds(gi, oi):
    """Early-stop GR (R22 / R28): every vertex the BFS labelled carries its exact
    alternating distance; every other vertex carries the floor, which is a valid
    lower bound (<= the exact distance, m+n included); the labels keep the
    neighbourhood invariant psi(v) <= psi(u) + 1 on every edge with a finite row
    label and psi(mate) = psi(v) + 1 across matched pairs; at least
    ceil(gr_target * alive) alive unmatched columns are labelled."""
    g = GR_GRAPHS[gi]()
    rng = np.random.default_rng(gi * 10 + oi + 5)
    opts = EARLY_OPTS[oi]
    mt = matcher(g, gr_early=1, **opts)
    INF = g.m + g.n
    for name, rm, cm in _matchings(g, rng):
        ml, pr, pc, rf, info = mt.global_relabel(T(rm), T(cm), info=True)
        pr, pc = H(pr), H(pc)
        epr, epc, eml, _ = oracle.global_relabel(g, rm, cm)
        fr, fc = info["floor_row"], info["floor_col"]
        assert fr == fc + 1 or fr == fc == INF
        lab_r, lab_c = pr < fr, pc < fc
        assert np.array_equal(pr[lab_r], epr[lab_r]) and np.array_equal(pc[lab_c], epc[lab_c]), (g.name, name)
        assert np.all(pr[~lab_r] == fr) and np.all(pc[~lab_c] == fc)
        assert np.all(epr[~lab_r] >= fr) and np.all(epc[~lab_c] >= fc), (g.name, name)
        # neighbourhood invariant on every edge with a finite row label
        r = np.repeat(np.arange(g.m), np.diff(g.indptr))
        fin = pr[r] < INF
        assert np.all(pc[g.indices[fin]] <= pr[r[fin]] + 1), (g.name, name)
        matched = (cm >= 0) & (rm[np.maximum(cm, 0)] == np.arange(g.n))
        v = np.nonzero(matched & (pc < INF))[0]
        assert np.all(pr[cm[v]] == pc[v] + 1), (g.name, name)
        # the target: alive unmatched columns (not matched, not -2, with an edge)
        deg_c = np.bincount(g.indices, minlength=g.n)
        alive = (~matched) & (cm != -2) & (deg_c > 0)
        want = int(alive.sum())
        if opts.get("gr_target", 0.6) < 1.0 and want >= opts.get("gr_target_min", 1024):
            want = int(np.ceil(opts["gr_target"] * want))
        reach = int((alive & (epc < INF)).sum())
        got = int((alive & lab_c).sum())
        assert got >= min(want, reach), (g.name, name, got, want, reach)
        if fc == INF:  # ran to completion: identical to the complete GR
            assert np.array_equal(pr, epr) and np.array_equal(pc, epc) and ml == eml
        else:
            assert ml == fr  # GETITERGR sees (stop level) + 4
    mt.close()


# ---------------------------------------------------------------- M0 on its own
@pytest.mark.parametrize("name,scale", [("C1", 1.0), ("C2", 0.05), ("C3", 0.005), ("C4", 1 / 64), ("C5", 1 / 16)])
def test_initial_matching_valid_and_maximal(name, scale):
    """R13: the device greedy's M0 is a valid matching and maximal (no edge joins
    two free vertices), and solving from it (MCM_INIT_GIVEN, the paper's protocol
    P:719-722) reaches the maximum."""
    g = synth.config(name, scale)
    mt = matcher(g)
    c0, rm, cm = mt.initial_matching()
    rm, cm = H(rm), H(cm)
    assert oracle.check_matching(g, rm, cm) == c0
    r = np.repeat(np.arange(g.m), np.diff(g.indptr))
    assert not np.any((rm[r] == -1) & (cm[g.indices] == -1)), name  # maximal
    mt.close()
    mm = g.mm if g.mm is not None else oracle.hopcroft_karp(g)[0]
    mt = matcher(g, init="given")
    card, rm2, cm2 = mt.solve(T(rm), T(cm))
    assert card == mm and mt.stats()["init_card"] == c0
    assert oracle.check_matching(g, H(rm2), H(cm2)) == mm
    mt.close()


def test_given_matching_out_of_range_rejected():
    g = synth.config("C1", 0.2)
    _, rm, cm = oracle.cheap_match(g)
    mt = matcher(g, init="given")
    for bad in ("row", "col", "col-2"):
        r, c = rm.copy(), cm.copy()
        if bad == "row":
            r[5] = g.n
        elif bad == "col":
            c[3] = g.m + 7
        else:
            c[np.nonzero(c == -1)[0][0]] = -2  # -2 is internal: not a valid GIVEN entry
        with pytest.raises(pkg.MCMError):
            mt.solve(T(r), T(c))
    card, _, _ = mt.solve(T(rm), T(cm))  # still usable
    assert card == oracle.hopcroft_karp(g)[0]
    mt.close()
    mt = matcher(g)
    c2 = cm.copy()
    c2[0] = -5
    with pytest.raises(pkg.MCMError):
        mt.global_relabel(T(rm), T(c2))
    mt.close()
