"""Generator determinism and structure (T1): same seed -> byte-identical CSR for
any thread count; digests and oracle MM match tests/golden/configs.json (written
by tools/make_golden.py, which calls only synth/ and oracle/)."""
import json
import os

import numpy as np
import pytest

import synth

GOLDEN = json.load(open(os.path.join(os.path.dirname(__file__), "golden", "configs.json")))


@pytest.mark.parametrize("case", GOLDEN["cases"], ids=lambda c: f"{c['name']}@{c['scale']:.4g}")
def test_digest_matches_golden(case):
    g = synth.config(case["name"], case["scale"])
    assert (g.m, g.n, g.nnz) == (case["m"], case["n"], case["nnz"])
    assert g.digest() == case["digest"]
    if case["closed_form_mm"] is not None:
        assert case["mm"] == case["closed_form_mm"]


@pytest.mark.parametrize("name,scale", [("C1", 0.3), ("C2", 0.01), ("C3", 0.002), ("C4", 1 / 512)])
def test_thread_count_independent(name, scale):
    old = synth.set_threads(0)
    try:
        synth.set_threads(1)
        a = synth.config(name, scale).digest()
        synth.set_threads(7)
        b = synth.config(name, scale).digest()
    finally:
        synth.set_threads(old)
    assert a == b


def test_csr_well_formed_sorted_dedup():
    for name, scale in [("C1", 0.2), ("C2", 0.005), ("C3", 0.001), ("C4", 1 / 512), ("C5", 1 / 512)]:
        g = synth.config(name, scale)
        assert g.indptr[0] == 0 and g.indptr[-1] == g.nnz
        assert np.all(np.diff(g.indptr) >= 0)
        assert g.indices.min() >= 0 and g.indices.max() < g.n
        for u in range(0, g.m, max(1, g.m // 500)):
            row = g.indices[g.indptr[u]: g.indptr[u + 1]]
            assert np.all(np.diff(row) > 0)


def test_road_structure():
    """C3: symmetric pattern, no self loops, average degree ~2.5, planted dominoes."""
    s = 60
    g = synth.road(s)
    r = np.repeat(np.arange(g.m), np.diff(g.indptr))
    fwd = set(zip(r.tolist(), g.indices.tolist()))
    assert all((c, rr) in fwd for rr, c in fwd)
    assert all(rr != c for rr, c in fwd)
    assert abs(g.nnz / g.m - 2.5) < 0.1


def test_banded_has_full_diagonal_before_permutation():
    g = synth.banded(5000, permute=False, rails=3, rail_len=50)
    for u in range(g.m):
        assert u in set(g.indices[g.indptr[u]: g.indptr[u + 1]].tolist())
