"""e2e probe (GPU box): mcm_match_host with pinned vs pageable host CSR against a
plain H2D copy of the same bytes; CUDA events.  python tools/probe_e2e.py C4"""
import os
import statistics
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import synth  # noqa: E402
import paper_conf_icpp_devecikuc13_b200 as pkg  # noqa: E402


def ev(fn, reps=5):
    ts = []
    for _ in range(reps):
        a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        torch.cuda.synchronize()
        a.record()
        fn()
        b.record()
        b.synchronize()
        ts.append(a.elapsed_time(b))
    return statistics.median(ts)


for name in sys.argv[1:] or ["C4"]:
    g = synth.config(name)
    ipp, ixp = torch.from_numpy(g.indptr).pin_memory(), torch.from_numpy(g.indices).pin_memory()
    ipq, ixq = torch.from_numpy(g.indptr.copy()), torch.from_numpy(g.indices.copy())
    need = pkg.mcm_workspace_bytes(g.m, g.n, g.nnz)
    ws = torch.empty(need, dtype=torch.uint8, device="cuda")
    rm = torch.empty(g.m, dtype=torch.int32).pin_memory()
    cm = torch.empty(g.n, dtype=torch.int32).pin_memory()
    d_ix = torch.empty(g.nnz, dtype=torch.int32, device="cuda")
    t_copy = ev(lambda: d_ix.copy_(ixp, non_blocking=True))
    t_pin = ev(lambda: pkg.match_host(ipp, ixp, g.m, g.n, workspace=ws, rmatch=rm, cmatch=cm))
    t_page = ev(lambda: pkg.match_host(ipq, ixq, g.m, g.n, workspace=ws, rmatch=rm, cmatch=cm))
    st = pkg.match_host(ipp, ixp, g.m, g.n, workspace=ws, rmatch=rm, cmatch=cm)[3]
    print(f"{name}: H2D copy of indices {t_copy:.2f} ms ({g.nnz * 4 / t_copy / 1e6:.1f} GB/s); match_host pinned "
          f"{t_pin:.2f} ms, pageable {t_page:.2f} ms; setup {st['ms_setup']:.2f} ms, solve {st['ms_total']:.2f} ms",
          flush=True)
