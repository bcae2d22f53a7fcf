"""The C-ABI library loads and exports every function include/mcm.h declares
(CPU tier: no compute calls), and the Python binding fails loudly without CUDA."""
import ctypes
import os
import re

import pytest

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
HEADER = os.path.join(ROOT, "include", "mcm.h")


def declared_functions():
    txt = open(HEADER).read()
    txt = re.sub(r"/\*.*?\*/", "", txt, flags=re.S)
    names = re.findall(r"\b(mcm_[a-z_]+)\s*\(", txt)
    return sorted(set(names))


def test_header_declares_the_boundary():
    names = declared_functions()
    for f in ["mcm_create", "mcm_solve", "mcm_set_k", "mcm_get_stats", "mcm_destroy", "mcm_strerror", "mcm_abi_sizes",
              "mcm_gap_relabel",
              "mcm_default_options", "mcm_workspace_bytes", "mcm_global_relabel", "mcm_set_options", "mcm_match_host"]:
        assert f in names


def test_library_exports_every_symbol():
    import __graft_entry__ as ge

    ge.build_cuda()
    L = ctypes.CDLL(os.path.join(ROOT, "paper_conf_icpp_devecikuc13_b200", "libmcm.so"))
    for f in declared_functions():
        assert hasattr(L, f), f


def test_host_only_calls():
    """Calls that touch no device: defaults, sizes, error strings, arg validation."""
    import paper_conf_icpp_devecikuc13_b200 as pkg

    o = pkg.mcm_default_options()
    assert o.k == 0.4 and o.shrink_min == 512 and o.gr_strategy == 0 and o.init == 0 and o.final_check == 1
    assert pkg.mcm_workspace_bytes(10, 10, 20) > 0
    assert pkg.mcm_workspace_bytes(-1, 10, 20) == 0
    assert pkg.mcm_workspace_bytes(1 << 30, 1 << 30, 5) == 0  # m+n+2 >= 2^31
    assert pkg.mcm_workspace_bytes(10, 10, 1 << 31) == 0
    L = pkg.lib()
    assert L.mcm_strerror(0) == b"ok"
    assert b"workspace" in L.mcm_strerror(-3)
    # NULL handle / NULL args -> MCM_EINVAL without touching CUDA
    assert L.mcm_solve(None, None, None, None) == -1
    assert L.mcm_match_host(None, None, 4, 4, 0, None, 0, None, None, None, None, None) == -1
    assert L.mcm_destroy(None) == -1
    assert L.mcm_set_k(None, 0.5) == -1
    L.mcm_pgr_init.restype = ctypes.c_int
    L.mcm_pgr_level.restype = ctypes.c_int
    assert L.mcm_pgr_init(None, None, 1, 0, 1, None, None, None, None) == -1
    assert L.mcm_pgr_level(None, None, 1, 0, 1, 0, None, None, None, None, None, None, None) == -1
    h = ctypes.c_void_p()
    assert L.mcm_create(None, None, 4, 4, 0, None, 0, None, None, ctypes.byref(h)) == -1
    assert pkg.mcm_default_options().gr_target == 0.6 and pkg.mcm_default_options().gr_target_min == 1024
    bad = pkg.mcm_default_options(k=-1.0)
    assert L.mcm_create(None, None, 4, 4, 0, None, 0, None, ctypes.byref(bad), ctypes.byref(h)) == -1


def test_binding_refuses_cpu_tensors():
    import torch

    import paper_conf_icpp_devecikuc13_b200 as pkg

    with pytest.raises((TypeError, RuntimeError, AssertionError)):
        pkg.solve(torch.zeros(3, dtype=torch.int32), torch.zeros(0, dtype=torch.int32), 2, 2)


def test_product_does_not_import_oracle():
    """The product package never references oracle/ (the checker stays test-only)."""
    pkgdir = os.path.join(ROOT, "paper_conf_icpp_devecikuc13_b200")
    for dp, _, files in os.walk(pkgdir):
        for f in files:
            if f.endswith((".py", ".cu", ".cuh", ".h")):
                txt = open(os.path.join(dp, f)).read()
                assert "import oracle" not in txt and "oracle." not in txt and "liboracle" not in txt, f
