"""B200-native push-relabel maximum-cardinality bipartite matching (G-PR,
Deveci, Kaya, Ucar, Catalyurek, ICPP 2013) -- thin Python binding of the C ABI in
``include/mcm.h``.

This module only marshals arguments: every step of the method runs in the CUDA
library ``libmcm.so`` (built in-tree by ``__graft_entry__.build()``).  PyTorch
supplies device memory and streams.  There is no CPU fallback: importing works
anywhere, but every call raises if the library or a CUDA device is missing.

Names follow include/mcm.h:

* :func:`mcm_default_options`, :func:`mcm_workspace_bytes`
* :class:`Matcher` -- ``mcm_create`` / ``mcm_solve`` / ``mcm_global_relabel`` /
  ``mcm_initial_matching`` / ``mcm_unit_step`` / ``mcm_gap_relabel`` /
  ``mcm_set_options`` / ``mcm_get_stats`` / ``mcm_destroy`` on one graph
* :func:`solve` -- create + solve in one call: ``(card, rmatch, cmatch)``
* :func:`match_host` -- ``mcm_match_host``: host CSR in, host matching out (the
  end-to-end path: H2D, create, solve and D2H in one C call)
"""
from __future__ import annotations

import ctypes
import os

__all__ = ["Options", "Stats", "Matcher", "solve", "match_host", "lib", "mcm_default_options", "mcm_workspace_bytes",
           "MCMError", "LIB_PATH"]

_HERE = os.path.dirname(os.path.abspath(__file__))
LIB_PATH = os.environ.get("MCM_LIB") or os.path.join(_HERE, "libmcm.so")  # MCM_LIB: A/B experiments only

MCM_OK, MCM_EINVAL, MCM_ECUDA, MCM_ENOMEM, MCM_EDEVICE, MCM_ENOCONV, MCM_EINTERNAL = 0, -1, -2, -3, -4, -5, -6
MCM_GR_ADAPTIVE, MCM_GR_FIXED = 0, 1
MCM_INIT_GREEDY, MCM_INIT_GIVEN, MCM_INIT_EMPTY = 0, 1, 2
MCM_UNIT_FIX, MCM_UNIT_SHRINK, MCM_UNIT_PUSH, MCM_UNIT_FIXMATCHING = 0, 1, 2, 3
MCM_WHERE_GRID, MCM_WHERE_TAIL = 0, 1


class Options(ctypes.Structure):
    """mcm_options_t"""

    _fields_ = [
        ("k", ctypes.c_double),
        ("gr_strategy", ctypes.c_int32),
        ("shrink_min", ctypes.c_int32),
        ("init", ctypes.c_int32),
        ("gap", ctypes.c_int32),
        ("final_check", ctypes.c_int32),
        ("dead_skip", ctypes.c_int32),
        ("tail_max", ctypes.c_int32),
        ("tail_f", ctypes.c_int32),
        ("compact_every", ctypes.c_int32),
        ("grid_ctas", ctypes.c_int32),
        ("tail_ctas", ctypes.c_int32),
        ("compact_adapt", ctypes.c_int32),
        ("gr_early", ctypes.c_int32),
        ("serial", ctypes.c_int32),
        ("sort_csc", ctypes.c_int32),
        ("bu_div", ctypes.c_int32),
        ("scan_rot", ctypes.c_int32),
        ("variant", ctypes.c_int32),
        ("tail_chain", ctypes.c_int32),
        ("grid_chain", ctypes.c_int32),
        ("max_loops", ctypes.c_int64),
        ("gr_target", ctypes.c_double),
        ("gr_target_min", ctypes.c_int32),
        ("gr_concurrent", ctypes.c_int32),
        ("perturb", ctypes.c_int32),
        ("gr_window", ctypes.c_int32),
        ("gr_window_max", ctypes.c_int32),
    ]


class Stats(ctypes.Structure):
    """mcm_stats_t"""

    _fields_ = [(f, ctypes.c_int64) for f in (
        "loops", "gr_count", "gr_levels", "pushes", "blocked", "dead", "edges_scanned", "slots", "shrinks", "gaps",
        "guard_reactivated", "fixed_cols", "init_card", "card", "tail_loops", "grid_barriers", "gr_rows", "gr_edges",
        "gr_cols", "greedy_edges", "rows_repaired", "tail_gr_levels", "debug_violations", "kernel_launches", "gr_window_levels")] + [
        (f, ctypes.c_double) for f in ("ms_init", "ms_gr", "ms_loop", "ms_total", "ms_setup")] + [
        ("grid_ctas", ctypes.c_int32), ("threads_per_cta", ctypes.c_int32)]

    def as_dict(self):
        return {f: getattr(self, f) for f, _ in self._fields_}


class MCMError(RuntimeError):
    def __init__(self, code, what=""):
        self.code = code
        super().__init__(f"{what}: {lib().mcm_strerror(code).decode()} (code {code})")


_lib = None


def lib():
    """Load libmcm.so (fails loudly when it has not been built)."""
    global _lib
    if _lib is None:
        if not os.path.exists(LIB_PATH):
            raise ImportError(f"{LIB_PATH} missing: run `python -c 'import __graft_entry__ as g; g.build()'`")
        L = ctypes.CDLL(LIB_PATH)
        vp, i32, i64, sz = ctypes.c_void_p, ctypes.c_int32, ctypes.c_int64, ctypes.c_size_t
        P = ctypes.POINTER
        L.mcm_default_options.argtypes = [P(Options)]
        L.mcm_default_options.restype = None
        L.mcm_workspace_bytes.argtypes = [i32, i32, i64, P(Options)]
        L.mcm_workspace_bytes.restype = sz
        L.mcm_create.argtypes = [vp, vp, i32, i32, i64, vp, sz, vp, P(Options), P(vp)]
        L.mcm_create.restype = ctypes.c_int
        L.mcm_solve.argtypes = [vp, vp, vp, vp]
        L.mcm_solve.restype = i64
        L.mcm_match_host.argtypes = [vp, vp, i32, i32, i64, vp, sz, vp, P(Options), vp, vp, P(Stats)]
        L.mcm_match_host.restype = i64
        L.mcm_global_relabel.argtypes = [vp, vp, vp, vp, vp, vp, vp]
        L.mcm_global_relabel.restype = i64
        L.mcm_initial_matching.argtypes = [vp, vp, vp, vp]
        L.mcm_initial_matching.restype = i64
        L.mcm_unit_step.argtypes = [vp, vp, i32, i32, i64, i32, vp, vp, vp, vp, vp, vp, vp]
        L.mcm_unit_step.restype = i64
        L.mcm_gap_relabel.argtypes = [vp, vp, vp, vp]
        L.mcm_gap_relabel.restype = i64
        L.mcm_pgr_init.argtypes = [vp, vp, i32, i32, i32, vp, vp, vp, vp]
        L.mcm_pgr_init.restype = ctypes.c_int
        L.mcm_pgr_level.argtypes = [vp, vp, i32, i32, i32, i32, vp, vp, vp, vp, vp, vp, vp]
        L.mcm_pgr_level.restype = ctypes.c_int
        L.mcm_set_options.argtypes = [vp, P(Options)]
        L.mcm_set_options.restype = ctypes.c_int
        L.mcm_set_k.argtypes = [vp, ctypes.c_double]
        L.mcm_set_k.restype = ctypes.c_int
        L.mcm_get_stats.argtypes = [vp, P(Stats)]
        L.mcm_get_stats.restype = ctypes.c_int
        L.mcm_destroy.argtypes = [vp]
        L.mcm_destroy.restype = ctypes.c_int
        L.mcm_strerror.argtypes = [ctypes.c_int]
        L.mcm_strerror.restype = ctypes.c_char_p
        L.mcm_abi_sizes.argtypes = [P(sz), P(sz)]
        L.mcm_abi_sizes.restype = ctypes.c_int
        so, ss = sz(0), sz(0)
        L.mcm_abi_sizes(ctypes.byref(so), ctypes.byref(ss))
        if so.value != ctypes.sizeof(Options) or ss.value != ctypes.sizeof(Stats):
            raise ImportError(f"libmcm.so ABI mismatch: options {so.value} vs {ctypes.sizeof(Options)}, "
                              f"stats {ss.value} vs {ctypes.sizeof(Stats)}")
        _lib = L
    return _lib


def mcm_default_options(**overrides) -> Options:
    o = Options()
    lib().mcm_default_options(ctypes.byref(o))
    for k, v in overrides.items():
        if k == "gr_strategy" and isinstance(v, str):
            v = {"adaptive": MCM_GR_ADAPTIVE, "fixed": MCM_GR_FIXED}[v]
        if k == "init" and isinstance(v, str):
            v = {"greedy": MCM_INIT_GREEDY, "given": MCM_INIT_GIVEN, "empty": MCM_INIT_EMPTY}[v]
        if not hasattr(o, k):
            raise TypeError(f"unknown option {k}")
        setattr(o, k, v)
    return o


def mcm_workspace_bytes(m: int, n: int, nnz: int, opts: Options | None = None) -> int:
    return lib().mcm_workspace_bytes(m, n, nnz, ctypes.byref(opts) if opts is not None else None)


def _torch():
    import torch

    return torch


def _stream_ptr(stream):
    """The stream the library enqueues on.  A stream other than the current one is
    first ordered after the current stream, where the caller's inputs, outputs and
    workspace were produced / allocated (torch's caching allocator is stream-ordered)."""
    torch = _torch()
    cur = torch.cuda.current_stream()
    s = stream if stream is not None else cur
    if s != cur:
        s.wait_stream(cur)
    return ctypes.c_void_p(s.cuda_stream)


def _dev_i32(t, name, length):
    torch = _torch()
    if not isinstance(t, torch.Tensor) or not t.is_cuda:
        raise TypeError(f"{name} must be a CUDA tensor (no CPU fallback)")
    if t.dtype != torch.int32 or not t.is_contiguous() or t.numel() != length:
        raise ValueError(f"{name}: need a contiguous int32 tensor of {length} elements")
    return ctypes.c_void_p(t.data_ptr() if length else 0)


class Matcher:
    """One graph on one device: mcm_create at construction, mcm_destroy on close().

    indptr (m+1) / indices (nnz): int32 CUDA tensors of the CSR (rows -> columns).
    The workspace is a torch uint8 tensor owned by this object."""

    def __init__(self, indptr, indices, m: int, n: int, stream=None, **opts):
        torch = _torch()
        for name, t in (("indptr", indptr), ("indices", indices)):
            if not isinstance(t, torch.Tensor) or not t.is_cuda:
                raise TypeError(f"{name} must be a CUDA tensor (no CPU fallback)")
        self.m, self.n = int(m), int(n)
        self.nnz = int(indices.numel())
        self.opts = mcm_default_options(**opts)
        self.device = indptr.device
        need = mcm_workspace_bytes(self.m, self.n, self.nnz, self.opts)
        if need == 0:
            raise MCMError(MCM_EINVAL, "mcm_workspace_bytes")
        with torch.cuda.device(self.device):
            self.workspace = torch.empty(need, dtype=torch.uint8, device=self.device)
            h = ctypes.c_void_p()
            rc = lib().mcm_create(_dev_i32(indptr, "indptr", self.m + 1), _dev_i32(indices, "indices", self.nnz),
                                  self.m, self.n, self.nnz, ctypes.c_void_p(self.workspace.data_ptr()), need,
                                  _stream_ptr(stream), ctypes.byref(self.opts), ctypes.byref(h))
        if rc != MCM_OK:
            raise MCMError(rc, "mcm_create")
        self._h = h

    def set_options(self, **opts):
        o = mcm_default_options(**{**{f: getattr(self.opts, f) for f, _ in Options._fields_}, **opts})
        rc = lib().mcm_set_options(self._h, ctypes.byref(o))
        if rc != MCM_OK:
            raise MCMError(rc, "mcm_set_options")
        self.opts = o

    def solve(self, rmatch=None, cmatch=None, stream=None):
        """mcm_solve -> (card, rmatch, cmatch) (int32 CUDA tensors)."""
        torch = _torch()
        if rmatch is None:
            rmatch = torch.empty(self.m, dtype=torch.int32, device=self.device)
        if cmatch is None:
            cmatch = torch.empty(self.n, dtype=torch.int32, device=self.device)
        with torch.cuda.device(self.device):
            card = lib().mcm_solve(self._h, _stream_ptr(stream), _dev_i32(rmatch, "rmatch", self.m),
                                   _dev_i32(cmatch, "cmatch", self.n))
        if card < 0:
            raise MCMError(int(card), "mcm_solve")
        return int(card), rmatch, cmatch

    def global_relabel(self, rmatch, cmatch, stream=None, info=False):
        """mcm_global_relabel -> (max_level, psi_row, psi_col, reached_free), plus
        dict(floor_row, floor_col, tail_levels) when info=True."""
        torch = _torch()
        pr = torch.empty(self.m, dtype=torch.int32, device=self.device)
        pc = torch.empty(self.n, dtype=torch.int32, device=self.device)
        inf = (ctypes.c_int64 * 4)()
        with torch.cuda.device(self.device):
            ml = lib().mcm_global_relabel(self._h, _stream_ptr(stream), _dev_i32(rmatch, "rmatch", self.m),
                                          _dev_i32(cmatch, "cmatch", self.n), _dev_i32(pr, "psi_row", self.m),
                                          _dev_i32(pc, "psi_col", self.n), inf)
        if ml < 0:
            raise MCMError(int(ml), "mcm_global_relabel")
        if info:
            return int(ml), pr, pc, int(inf[0]), dict(floor_row=int(inf[1]), floor_col=int(inf[2]), tail_levels=int(inf[3]))
        return int(ml), pr, pc, int(inf[0])

    def initial_matching(self, rmatch=None, cmatch=None, stream=None):
        """mcm_initial_matching -> (|M0|, rmatch, cmatch): the device cheap matching alone."""
        torch = _torch()
        if rmatch is None:
            rmatch = torch.empty(self.m, dtype=torch.int32, device=self.device)
        if cmatch is None:
            cmatch = torch.empty(self.n, dtype=torch.int32, device=self.device)
        with torch.cuda.device(self.device):
            c = lib().mcm_initial_matching(self._h, _stream_ptr(stream), _dev_i32(rmatch, "rmatch", self.m),
                                           _dev_i32(cmatch, "cmatch", self.n))
        if c < 0:
            raise MCMError(int(c), "mcm_initial_matching")
        return int(c), rmatch, cmatch

    def unit_step(self, unit, where, loop, mu_row, mu_col, psi_row, psi_col, iA, Ac, Ap, stream=None):
        """mcm_unit_step on the given CUDA int32 tensors (updated in place) -> the
        phase's result (see include/mcm.h)."""
        torch = _torch()
        unit = {"fix": MCM_UNIT_FIX, "shrink": MCM_UNIT_SHRINK, "push": MCM_UNIT_PUSH,
                "fixmatching": MCM_UNIT_FIXMATCHING}.get(unit, unit)
        where = {"grid": MCM_WHERE_GRID, "tail": MCM_WHERE_TAIL}.get(where, where)
        ln = int(Ac.numel())
        with torch.cuda.device(self.device):
            r = lib().mcm_unit_step(self._h, _stream_ptr(stream), unit, where, int(loop), ln,
                                    _dev_i32(mu_row, "mu_row", self.m), _dev_i32(mu_col, "mu_col", self.n),
                                    _dev_i32(psi_row, "psi_row", self.m), _dev_i32(psi_col, "psi_col", self.n),
                                    _dev_i32(iA, "iA", self.n), _dev_i32(Ac, "Ac", ln), _dev_i32(Ap, "Ap", ln))
        if r < 0:
            raise MCMError(int(r), "mcm_unit_step")
        return int(r)

    def gap_relabel(self, psi_row, psi_col, stream=None):
        """mcm_gap_relabel on copies of the given labels -> (gap, psi_row', psi_col')."""
        torch = _torch()
        pr = psi_row.to(self.device, torch.int32).contiguous().clone()
        pc = psi_col.to(self.device, torch.int32).contiguous().clone()
        with torch.cuda.device(self.device):
            g = lib().mcm_gap_relabel(self._h, _stream_ptr(stream), _dev_i32(pr, "psi_row", self.m),
                                      _dev_i32(pc, "psi_col", self.n))
        if g < -1:
            raise MCMError(int(g), "mcm_gap_relabel")
        return int(g), pr, pc

    # NEXT-4 experiment (include/mcm.h mcm_pgr_*; orchestration in pgr.py)
    def pgr_init(self, nparts, part, words, rmatch, slice_, psi_row, psi_col, stream=None):
        torch = _torch()
        with torch.cuda.device(self.device):
            rc = lib().mcm_pgr_init(self._h, _stream_ptr(stream), nparts, part, words,
                                    _dev_i32(rmatch, "rmatch", self.m), _dev_i32(slice_, "slice", words + 1),
                                    _dev_i32(psi_row, "psi_row", self.m), _dev_i32(psi_col, "psi_col", self.n))
        if rc != MCM_OK:
            raise MCMError(rc, "mcm_pgr_init")

    def pgr_level(self, nparts, part, words, level, rmatch, cmatch, frontier, slice_, psi_row, psi_col,
                  reached_free, stream=None):
        torch = _torch()
        if not (isinstance(reached_free, torch.Tensor) and reached_free.is_cuda and reached_free.dtype == torch.int64
                and reached_free.numel() == 1):
            raise TypeError("reached_free must be a CUDA int64 tensor of 1 element")
        with torch.cuda.device(self.device):
            rc = lib().mcm_pgr_level(self._h, _stream_ptr(stream), nparts, part, words, level,
                                     _dev_i32(rmatch, "rmatch", self.m), _dev_i32(cmatch, "cmatch", self.n),
                                     _dev_i32(frontier, "frontier", nparts * (words + 1)),
                                     _dev_i32(slice_, "slice", words + 1), _dev_i32(psi_row, "psi_row", self.m),
                                     _dev_i32(psi_col, "psi_col", self.n), ctypes.c_void_p(reached_free.data_ptr()))
        if rc != MCM_OK:
            raise MCMError(rc, "mcm_pgr_level")

    def stats(self) -> dict:
        s = Stats()
        rc = lib().mcm_get_stats(self._h, ctypes.byref(s))
        if rc != MCM_OK:
            raise MCMError(rc, "mcm_get_stats")
        return s.as_dict()

    def close(self):
        if getattr(self, "_h", None):
            lib().mcm_destroy(self._h)
            self._h = None

    def __del__(self):
        try:
            self.close()
        except Exception:
            pass


def solve(indptr, indices, m: int, n: int, stream=None, **opts):
    """Create + solve: ``(card, rmatch, cmatch)`` with rmatch/cmatch int32 CUDA tensors."""
    mt = Matcher(indptr, indices, m, n, stream=stream, **opts)
    try:
        return mt.solve(stream=stream)
    finally:
        mt.close()


def _host_i32(t, name, length):
    torch = _torch()
    if not isinstance(t, torch.Tensor) or t.is_cuda:
        raise TypeError(f"{name} must be a CPU (preferably pinned) tensor")
    if t.dtype != torch.int32 or not t.is_contiguous() or t.numel() != length:
        raise ValueError(f"{name}: need a contiguous int32 tensor of {length} elements")
    return ctypes.c_void_p(t.data_ptr() if length else 0)


def match_host(indptr, indices, m: int, n: int, workspace=None, rmatch=None, cmatch=None, stream=None, device=None,
               **opts):
    """``mcm_match_host``: CSR in HOST memory (int32 CPU tensors, pinned for
    asynchronous copies) -> ``(card, rmatch, cmatch, stats)`` with the matching in
    HOST int32 tensors.  The device work (validation, transpose, solve) runs in
    libmcm.so on ``device`` (default: the current CUDA device); ``workspace`` (a
    CUDA uint8 tensor of at least mcm_workspace_bytes) is allocated when None."""
    torch = _torch()
    m, n, nnz = int(m), int(n), int(indices.numel())
    o = mcm_default_options(**opts)
    need = mcm_workspace_bytes(m, n, nnz, o)
    if need == 0:
        raise MCMError(MCM_EINVAL, "mcm_workspace_bytes")
    dev = torch.device("cuda", torch.cuda.current_device()) if device is None else torch.device(device)
    if workspace is None:
        workspace = torch.empty(need, dtype=torch.uint8, device=dev)
    if not workspace.is_cuda or workspace.numel() < need:
        raise ValueError(f"workspace: need a CUDA uint8 tensor of at least {need} bytes")
    if rmatch is None:
        rmatch = torch.empty(m, dtype=torch.int32, pin_memory=True)
    if cmatch is None:
        cmatch = torch.empty(n, dtype=torch.int32, pin_memory=True)
    st = Stats()
    with torch.cuda.device(workspace.device):
        card = lib().mcm_match_host(_host_i32(indptr, "indptr", m + 1), _host_i32(indices, "indices", nnz), m, n, nnz,
                                    ctypes.c_void_p(workspace.data_ptr()), workspace.numel(), _stream_ptr(stream),
                                    ctypes.byref(o), _host_i32(rmatch, "rmatch", m), _host_i32(cmatch, "cmatch", n),
                                    ctypes.byref(st))
    if card < 0:
        raise MCMError(int(card), "mcm_match_host")
    return int(card), rmatch, cmatch, st.as_dict()
