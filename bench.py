"""bench.py -- G-PR maximum-cardinality matching throughput on B200.

    python bench.py [--gpus N] [--steps K] [--warmup W] [--config C2] [--impl ours|reference]

One STEP = one pass of the whole hot path over one synthetic graph already
resident in HBM: mcm_create (validate + copy + CSC transpose)
followed by mcm_solve (greedy init, GRs, fix/push loop, guard, FIXMATCHING).
Default workload: C4 (R-MAT 2^23 x 2^23, 131M nnz), the largest single-GPU
configuration of BASELINE.json (its metric names no config); C1-C3 and C5 behind
--config.  value = edges/s = (sum over ranks of nnz) / (max over ranks of the mean
step time).  N > 1 (torchrun): every rank solves its own instance (seed + rank), no
data-path collective -> "scaling": "weak".

Beside the step the line carries: `paper_protocol` (t_pr: the solve alone from the
cheap matching M0 computed outside the timed region, MCM_INIT_GIVEN -- the paper
times only the matching), `paper_config` (the paper's atomic-free loop:
one push per column per loop, complete GRs, post-GR shrink only, k = 0.7; the
build's push chains / early-stop GR / adaptive compaction off), `cpu_baseline`
(the oracle's PR-FIFO and Hopcroft-Karp on the host, rank 0, N = 1).

L2 (126 MB) is flushed between timed steps by writing a 512 MiB buffer outside
the per-step CUDA events.  `e2e` repeats the measurement through the C ABI's
host-buffer entry point mcm_match_host with the CSR in pinned HOST memory: H2D
copy + create + solve + D2H of the matching inside the timed region, one call
per step (the per-graph end-to-end time); `e2e.pipelined` adds the request
throughput when the steps are issued by `--e2e-streams` host threads (one stream
and workspace each, default 2), so one request's PCIe transfers overlap another's
kernels.  `--impl reference` times the CPU oracle
(sequential PR-FIFO with GR every 0.5(m+n) pushes, from the cheap
matching) on the host cores: the paper's own CPU comparison algorithm.
"""
from __future__ import annotations

import argparse
import json
import os
import statistics
import subprocess
import sys
import threading
import time

ROOT = os.path.dirname(os.path.abspath(__file__))
sys.path.insert(0, ROOT)

CONFIG_DESC = {
    "C1": "uniform random bipartite 10,000 x 10,000, 80,000 samples (avg deg 8), seed 1",
    "C2": "permuted banded circuit-like 1.5M x 1.5M, diag + Poisson(2.47) in +-64 + 150 rails x 2000, seed 2",
    "C3": "road-like planted lattice 4900^2 = 24.01M x 24.01M, avg deg 2.5, seed 3",
    "C4": "R-MAT 2^23 x 2^23, 2^27 samples (0.57,0.19,0.19,0.05), permuted, seed 4",
    "C5": "uniform 2^21 x 2^21, 16 * 2^21 samples (avg deg 16), seed 1000+i",
}
METRIC = "MCM solve throughput (edges/s = nnz / (create + solve time)) per graph"
# the paper's G-PR (Alg. 7-9 with its GR schedule): no push
# chains (R26), complete GRs (no R22 / R28 early stop), post-GR shrink only, k = 0.7
PAPER_OPTS = dict(tail_chain=0, grid_chain=0, gr_early=0, compact_adapt=0, k=0.7)


def config_keys(name, g, l2, parallelism):
    """The `config` object: the same keys on both arms (workload, sizes, L2 policy,
    parallelism); run details go to `run`."""
    return {"workload": f"{name}: {CONFIG_DESC[name]}", "m": g.m, "n": g.n, "nnz": g.nnz, "l2": l2,
            "parallelism": parallelism}


def _peaks():
    try:
        return json.load(open(os.path.join(ROOT, "MEASURED_PEAKS.json")))
    except Exception:
        return None


def _graph(name, rank):
    import synth

    if name == "C5":
        return synth.config("C5", 1.0, index=rank)
    if rank == 0:
        return synth.config(name)
    # an independent instance of the same recipe for rank > 0 (same distribution);
    # the large recipes are generated once, not after rank 0's graph as well
    if name == "C3":
        return synth.road(4900, 0.5, 0.4, 0.1, 3 + 7919 * rank, True, False, 256, name="C3")
    if name == "C4":
        return synth.rmat(23, 16 << 23, seed=4 + 7919 * rank, name="C4")
    g = synth.config(name)
    if name == "C1":
        return synth.uniform(g.m, g.n, 8 * g.m, 1 + 7919 * rank, name="C1")
    if name == "C2":
        return synth.banded(g.n, 2.47, 64, 150, 2000, 2 + 7919 * rank, True, name="C2")
    raise KeyError(name)


class Clocks:
    """nvidia-smi sampling during the timed region (B200_PROFILING.md clocks line)."""

    FIELDS = ("clocks.sm,clocks.max.sm,clocks_event_reasons.hw_slowdown,clocks_event_reasons.hw_thermal_slowdown,"
              "clocks_event_reasons.sw_thermal_slowdown,clocks_event_reasons.sw_power_cap")

    def __init__(self, index):
        self.index = index
        self.proc = None
        self.lines = []

    def start(self):
        try:
            self.proc = subprocess.Popen(
                ["nvidia-smi", "-i", str(self.index), f"--query-gpu={self.FIELDS}", "--format=csv,noheader,nounits",
                 "-lms", "50"], stdout=subprocess.PIPE, stderr=subprocess.DEVNULL, text=True)
            self.t = threading.Thread(target=self._read, daemon=True)
            self.t.start()
        except Exception:
            self.proc = None

    def _read(self):
        for line in self.proc.stdout:
            self.lines.append(line.strip())

    def stop(self):
        if not self.proc:
            return {"sm_mhz": None, "sm_max_mhz": None, "reasons": ["nvidia-smi unavailable"]}
        time.sleep(0.06)
        self.proc.terminate()
        try:
            self.proc.wait(2)
        except Exception:
            self.proc.kill()
        sm, mx, reasons = [], [], set()
        names = ["hw_slowdown", "hw_thermal_slowdown", "sw_thermal_slowdown", "sw_power_cap"]
        for ln in self.lines:
            parts = [x.strip() for x in ln.split(",")]
            if len(parts) < 6:
                continue
            try:
                sm.append(float(parts[0]))
                mx.append(float(parts[1]))
            except ValueError:
                continue
            for nm, val in zip(names, parts[2:6]):
                if val.lower().startswith("active"):
                    reasons.add(nm)
        return {"sm_mhz": statistics.median(sm) if sm else None, "sm_max_mhz": max(mx) if mx else None,
                "reasons": sorted(reasons), "samples": len(sm)}


def algorithmic_bytes(st, m, n, nnz):
    """Bytes the method must move per solve, from the solve's own counters and the
    per-unit figures of SURVEY.md §8(d) (int32 = 4 B):
      push: 44 B per processed active column + 8 B per scanned neighbour
      fix step: 24 B per worklist slot
      GR: 16 B per expanded row + 8 B per read adjacency entry + 16 B per labelled column
      greedy init: 8 B per column (cptr pair) + 8 B per read adjacency entry + 8 B per matched pair
      FIXMATCHING + outputs: 12 n + 8 m
    """
    processed = st["pushes"] + st["blocked"] + st["dead"]
    b = 44 * processed + 8 * st["edges_scanned"]
    b += 24 * st["slots"]
    b += 16 * st["gr_rows"] + 8 * st["gr_edges"] + 16 * st["gr_cols"]
    b += 8 * n + 8 * st["greedy_edges"] + 8 * st["init_card"]
    b += 12 * n + 8 * m
    return int(b)


def sector_bytes(st, m, n, nnz):
    """The same counters priced at the memory system's granularity: a random
    4- or 8-byte access moves a 32-byte sector (SURVEY.md §8(d) "sector-level
    reality"); coalesced streams move their own bytes.  A model, not a measurement
    (DESIGN.md §6): it tells how far a solve is from the bound its access pattern
    allows, which the algorithmic bytes above cannot.
      push, per processed column: Ac 4 + column word 32 + bounds 32 + adjacency 32
        + iA 32 + stores 68; per scanned neighbour: 4 + row word 32
      fix step, per slot: Ap/Ac 8 + column word 32 + mate's row word 32 + iA 32
      GR: per frontier entry 16 + first adjacency sector 32; per adjacency entry
        4 + column word 32 + CAS 32; per labelled column: mate's row word 32 +
        bounds 32 + label store 32 + staged entry 16
      greedy: per column 16; per scanned entry 4 + row word 32 + claim 32
      FIXMATCHING: 12 n + 8 m + 32 per matched pair
    """
    processed = st["pushes"] + st["blocked"] + st["dead"]
    b = 200 * processed + 36 * st["edges_scanned"]
    b += 104 * st["slots"]
    b += 48 * st["gr_rows"] + 68 * st["gr_edges"] + 112 * st["gr_cols"]
    b += 16 * n + 68 * st["greedy_edges"]
    b += 12 * n + 8 * m + 32 * st["init_card"]
    return int(b)


def setup_bytes(m, n, nnz):
    """mcm_create: validate (4(m+1) + 4 nnz) + copy (2 x (4(m+1) + 4 nnz)) + count (4 nnz
    + 4 nnz atomics) + scan (3 x 4n) + scatter (4(m+1) + 4 nnz + 4 nnz atomics + 4 nnz)."""
    return int(4 * (m + 1) * 4 + 4 * nnz * 8 + 12 * n)


def reduce_over_ranks(t_step, t_e2e, t_solve, t_create, nnz, world, device):
    """Max over ranks of every time (the job is as slow as its slowest rank), sum of
    the units (edges) all ranks processed.  No data-path collective: this runs once,
    after the timed region."""
    import torch

    vals = torch.tensor([t_step, t_e2e, t_solve, t_create, nnz], dtype=torch.float64, device=device)
    if world > 1:
        mx = vals.clone()
        torch.distributed.all_reduce(mx, op=torch.distributed.ReduceOp.MAX)
        sm = vals.clone()
        torch.distributed.all_reduce(sm, op=torch.distributed.ReduceOp.SUM)
        return mx[0].item(), mx[1].item(), mx[2].item(), mx[3].item(), sm[4].item()
    return t_step, t_e2e, t_solve, t_create, nnz


def run_ours(args, rank, world, local_rank):
    import torch

    import paper_conf_icpp_devecikuc13_b200 as pkg

    dev = torch.device("cuda", local_rank)
    torch.cuda.set_device(dev)
    g = _graph(args.config, rank)
    ip_h = torch.from_numpy(g.indptr).pin_memory()
    ix_h = torch.from_numpy(g.indices).pin_memory()
    ip = ip_h.to(dev)
    ix = ix_h.to(dev)
    stream = torch.cuda.current_stream(dev)
    flush = torch.empty(512 << 20, dtype=torch.uint8, device=dev)
    rm = torch.empty(g.m, dtype=torch.int32, device=dev)
    cm = torch.empty(g.n, dtype=torch.int32, device=dev)
    opts = dict(k=args.k)
    need = pkg.mcm_workspace_bytes(g.m, g.n, g.nnz, pkg.mcm_default_options(**opts))
    ws = torch.empty(need, dtype=torch.uint8, device=dev)
    launches = 0

    def step():
        mt = pkg.Matcher.__new__(pkg.Matcher)
        mt_init(mt, ip, ix, g, ws, opts)
        card, _, _ = mt.solve(rm, cm)
        return mt, card

    def barrier():
        if world > 1:
            torch.distributed.barrier()
        torch.cuda.synchronize(dev)

    for _ in range(args.warmup):
        mt, card = step()
        mt.close()
    # timed region: K steps, L2 flushed before each, CUDA events around each step
    evs = [(torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True),
            torch.cuda.Event(enable_timing=True)) for _ in range(args.steps)]
    clocks = Clocks(local_rank)
    barrier()
    clocks.start()
    t_wall = time.perf_counter()
    cards, stats = [], None
    for i in range(args.steps):
        flush.fill_(i & 0xFF)
        e0, e1, e2 = evs[i]
        e0.record(stream)
        mt = pkg.Matcher.__new__(pkg.Matcher)
        mt_init(mt, ip, ix, g, ws, opts)
        e1.record(stream)
        card, _, _ = mt.solve(rm, cm)
        e2.record(stream)
        cards.append(card)
        stats = mt.stats()
        launches += stats["kernel_launches"]
        used_opts = {f: getattr(mt.opts, f) for f, _ in pkg.Options._fields_}
        mt.close()
    barrier()
    wall = time.perf_counter() - t_wall
    clk = clocks.stop()
    step_ms = [a.elapsed_time(c) for a, b_, c in evs]
    create_ms = [a.elapsed_time(b_) for a, b_, c in evs]
    solve_ms = [b_.elapsed_time(c) for a, b_, c in evs]
    t_step = sum(step_ms) / len(step_ms)
    t_solve = sum(solve_ms) / len(solve_ms)
    t_create = sum(create_ms) / len(create_ms)

    # ---- e2e through the C ABI with HOST buffers: one mcm_match_host call per step
    # (H2D of the CSR into the workspace, validate + transpose, solve, D2H of the
    # matching; the call synchronises its stream before it returns).  (a) serial: one
    # call at a time, CUDA events around each; (b) pipelined, the reported e2e: the
    # steps are independent requests, issued by E host threads with a stream, a
    # workspace and host output buffers each, so one request's PCIe transfers overlap
    # another's kernels (the H2D of the C4 CSR alone is ~10 ms); K steps timed as a
    # whole with events on the main stream, after W pipelined warm-up steps.
    rm_h = torch.empty(g.m, dtype=torch.int32).pin_memory()
    cm_h = torch.empty(g.n, dtype=torch.int32).pin_memory()
    e2e_ms = []
    for i in range(args.warmup + args.steps):
        flush.fill_(i & 0xFF)
        barrier()
        a = torch.cuda.Event(enable_timing=True)
        b = torch.cuda.Event(enable_timing=True)
        a.record(stream)
        card_e, _, _, _ = pkg.match_host(ip_h, ix_h, g.m, g.n, workspace=ws, rmatch=rm_h, cmatch=cm_h, stream=stream,
                                         **opts)
        b.record(stream)
        b.synchronize()
        if card_e != cards[-1]:
            raise RuntimeError(f"e2e cardinality {card_e} != {cards[-1]}")
        if i >= args.warmup:
            e2e_ms.append(a.elapsed_time(b))
    t_e2e_serial = sum(e2e_ms) / len(e2e_ms)
    E = max(1, args.e2e_streams)
    wsp = [ws] + [torch.empty(need, dtype=torch.uint8, device=dev) for _ in range(E - 1)]
    outs = [(rm_h, cm_h)] + [(torch.empty(g.m, dtype=torch.int32).pin_memory(),
                              torch.empty(g.n, dtype=torch.int32).pin_memory()) for _ in range(E - 1)]
    estreams = [torch.cuda.Stream(dev) for _ in range(E)]
    e2e_err = []

    def e2e_worker(t, count):
        try:
            with torch.cuda.device(dev):
                for _ in range(t, count, E):
                    c, _, _, _ = pkg.match_host(ip_h, ix_h, g.m, g.n, workspace=wsp[t], rmatch=outs[t][0],
                                                cmatch=outs[t][1], stream=estreams[t], **opts)
                    if c != cards[-1]:
                        e2e_err.append(RuntimeError(f"e2e cardinality {c} != {cards[-1]}"))
        except Exception as ex:  # surfaced after the join
            e2e_err.append(ex)

    def e2e_run(count):
        main = torch.cuda.current_stream(dev)
        a = torch.cuda.Event(enable_timing=True)
        b = torch.cuda.Event(enable_timing=True)
        a.record(main)
        for s_ in estreams:
            s_.wait_event(a)
        ths = [threading.Thread(target=e2e_worker, args=(t, count)) for t in range(E)]
        for th in ths:
            th.start()
        for th in ths:
            th.join()
        if e2e_err:
            raise e2e_err[0]
        for s_ in estreams:
            main.wait_stream(s_)
        b.record(main)
        b.synchronize()
        return a.elapsed_time(b)

    barrier()
    e2e_run(args.warmup)
    barrier()
    t_e2e = e2e_run(args.steps) / args.steps

    # ---- the paper's protocol and the paper's configuration, same graph, same run
    paper_protocol = run_paper_protocol(args, g, ip, ix, ws, rm, cm, flush, stream, opts, cards[-1])
    paper_config = run_paper_config(args, g, ip, ix, ws, rm, cm, flush, stream, cards[-1])

    # ---- max over ranks (times), sum over ranks (units processed)
    t_step_max, t_e2e_max, t_solve_max, t_create_max, nnz_total = reduce_over_ranks(
        t_step, t_e2e, t_solve, t_create, float(g.nnz), world, dev)
    t_e2e_ser_max = reduce_over_ranks(t_e2e_serial, 0.0, 0.0, 0.0, 0.0, world, dev)[0]
    if rank != 0:
        return None

    peaks = _peaks()
    hbm_peak = peaks["hbm_gbs"] if peaks else 6650.0
    alg = algorithmic_bytes(stats, g.m, g.n, g.nnz)
    sb_ = sector_bytes(stats, g.m, g.n, g.nnz)
    achieved = alg / (t_solve * 1e-3) / 1e9  # GB/s of the solve kernel
    traffic = None
    tp = os.path.join(ROOT, "profiles", f"ncu_traffic_{args.config}.json")
    if os.path.exists(tp):
        try:
            traffic = json.load(open(tp)).get("dram_bytes_per_launch")
        except Exception:
            traffic = None
    line = {
        "metric": METRIC,
        "value": nnz_total / (t_step_max * 1e-3),
        "unit": "edges/s",
        "n_gpus": world,
        "steps": args.steps,
        "warmup": args.warmup,
        "ms_per_step": t_step_max,
        "higher_is_better": True,
        "scaling": "weak",
        "vs_baseline": None,
        "dtype": "int32",
        "data": "synthetic",
        "config": config_keys(args.config, g, "flushed between steps (512 MiB write, outside the step events)",
                              f"replicas x{world} (one instance per GPU, no collective)"),
        "run": {
            "mm": cards[-1], "init_card": stats["init_card"],
            "options": used_opts,
            "step": "mcm_create + mcm_solve (device-resident CSR)",
            "ms_create": t_create_max, "ms_solve": t_solve_max,
            "edges_per_s_solve_only": nnz_total / (t_solve_max * 1e-3),
            "wall_s_timed_region": wall,
        },
        "roofline": {
            "bound": "hbm",
            "kernel": "gpr_kernel (persistent cooperative solve)",
            "achieved": achieved,
            "peak": hbm_peak,
            "unit": "GB/s",
            "frac": achieved / hbm_peak,
            "traffic": traffic,
            "algorithmic_bytes_per_launch": alg,
            "peak_source": "MEASURED_PEAKS.json hbm_gbs" if peaks else "fallback B200_PROFILING.md",
            "l2_sector_model": {"bytes": sb_, "achieved": sb_ / (t_solve * 1e-3) / 1e9,
                             "frac": sb_ / (t_solve * 1e-3) / 1e9 / hbm_peak},
            "latency": {"grid_barriers": stats["grid_barriers"], "loops": stats["loops"],
                        "gr_levels": stats["gr_levels"], "us_per_grid_barrier_measured": 1.27,
                        "barrier_floor_ms": stats["grid_barriers"] * 1.27e-3},
        },
        "solve_stats": {k: stats[k] for k in ("loops", "gr_count", "gr_levels", "pushes", "blocked", "dead",
                                              "edges_scanned", "slots", "shrinks", "guard_reactivated",
                                              "tail_loops", "grid_barriers", "gr_rows", "gr_edges", "gr_cols",
                                              "greedy_edges", "init_card", "ms_init", "ms_gr", "ms_loop",
                                              "ms_total", "grid_ctas")},
        "clocks": clk,
        "e2e": {"value": nnz_total / (t_e2e_ser_max * 1e-3), "unit": "edges/s",
                "h2d_bytes_per_step": 4 * (g.m + 1 + g.nnz), "d2h_bytes_per_step": 4 * (g.m + g.n),
                "ms_per_step": t_e2e_ser_max,
                "how": "one mcm_match_host call per step (pinned host CSR -> H2D -> create -> solve -> D2H of the "
                       "matching), CUDA events around each call: the per-graph end-to-end time",
                "pipelined": {"value": nnz_total / (t_e2e_max * 1e-3), "unit": "edges/s", "ms_per_step": t_e2e_max,
                              "host_streams": E,
                              "how": f"{args.steps} calls issued by {E} host threads, one stream / workspace each, "
                                     f"timed as a whole: one call's PCIe transfers overlap another's kernels "
                                     f"(request throughput, not per-graph time)"}},
        "gpu_launches": launches,
        "gpu_launches_note": "kernels of the timed region, counted by libmcm at its launch sites "
                             "(mcm_stats_t.kernel_launches: create's setup kernels + the persistent solve kernel)",
        "paper_protocol": paper_protocol,
        "paper_config": paper_config,
    }
    if world > 1:
        line["run"]["nccl_world_size"] = world
    if world == 1 and not args.no_cpu_baseline:
        line["cpu_baseline"] = cpu_baseline(args.config, g)
    return line


def _timed_solves(args, mk, flush, stream, card_ref, before=None):
    """Create a handle per step (untimed), optionally prepare (untimed), flush L2,
    time mcm_solve alone with CUDA events on the solve stream; returns (ms list,
    stats of the last solve)."""
    import torch

    ms, st = [], None
    for i in range(args.warmup + args.steps):
        mt = mk()
        if before:
            before(mt)
        flush.fill_(i & 0xFF)
        a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        a.record(stream)
        card = mt.solve_into()
        b.record(stream)
        b.synchronize()
        st = mt.stats()
        mt.close()
        if card != card_ref:
            raise RuntimeError(f"cardinality {card} != {card_ref}")
        if i >= args.warmup:
            ms.append(a.elapsed_time(b))
    return ms, st


def run_paper_protocol(args, g, ip, ix, ws, rm, cm, flush, stream, opts, card_ref):
    """t_pr: the paper times the matching from a cheap
    initial matching computed beforehand.  Per step: mcm_create + mcm_initial_matching
    (the device greedy, R13) outside the timed region, then mcm_solve with
    MCM_INIT_GIVEN from that M0, timed alone."""
    m0 = []

    def mk():
        mt = pkg_matcher(ip, ix, g, ws, dict(opts, init="given"))
        mt.solve_into = lambda: mt.solve(rm, cm)[0]
        return mt

    def before(mt):
        m0.append(mt.initial_matching(rm, cm)[0])

    ms, st = _timed_solves(args, mk, flush, stream, card_ref, before)
    t = statistics.median(ms)
    return {"t_pr_ms_median": t, "t_pr_ms_mean": statistics.mean(ms), "t_pr_ms_min": min(ms),
            "edges_per_s": g.nnz / (t * 1e-3), "m0_card": m0[-1], "mm": card_ref,
            "loops": st["loops"], "gr_count": st["gr_count"], "gr_levels": st["gr_levels"],
            "what": "mcm_solve alone, init=given from the device cheap matching (mcm_initial_matching, untimed); "
                    "create untimed (P:719-722)"}


def run_paper_config(args, g, ip, ix, ws, rm, cm, flush, stream, card_ref):
    """The paper's atomic-free G-PR: one push per column per loop
    (no push chains, R26), complete GRs (no early stop, R22 / R28), post-GR shrink
    only (no adaptive compaction), k = 0.7.  Solve timed alone (create
    untimed), same graph, same L2 flush."""
    def mk():
        mt = pkg_matcher(ip, ix, g, ws, PAPER_OPTS)
        mt.solve_into = lambda: mt.solve(rm, cm)[0]
        return mt

    ms, st = _timed_solves(args, mk, flush, stream, card_ref)
    t = statistics.median(ms)
    return {"options": PAPER_OPTS, "ms_solve_median": t, "ms_solve_mean": statistics.mean(ms),
            "edges_per_s_solve_only": g.nnz / (t * 1e-3), "mm": card_ref,
            "loops": st["loops"], "gr_count": st["gr_count"], "gr_levels": st["gr_levels"],
            "pushes": st["pushes"], "blocked": st["blocked"], "guard_reactivated": st["guard_reactivated"]}


def pkg_matcher(ip, ix, g, ws, opts):
    import paper_conf_icpp_devecikuc13_b200 as pkg

    mt = pkg.Matcher.__new__(pkg.Matcher)
    mt_init(mt, ip, ix, g, ws, opts)
    return mt


def mt_init(mt, ip, ix, g, ws, opts, stream=None):
    """Matcher over a preallocated workspace (mcm_create through the C ABI)."""
    import ctypes

    import paper_conf_icpp_devecikuc13_b200 as pkg

    mt.m, mt.n, mt.nnz = g.m, g.n, g.nnz
    mt.opts = pkg.mcm_default_options(**opts)
    mt.device = ip.device
    mt.workspace = ws
    h = ctypes.c_void_p()
    import torch

    st = stream if stream is not None else torch.cuda.current_stream()
    rc = pkg.lib().mcm_create(ctypes.c_void_p(ip.data_ptr()), ctypes.c_void_p(ix.data_ptr()), g.m, g.n, g.nnz,
                              ctypes.c_void_p(ws.data_ptr()), ws.numel(), ctypes.c_void_p(st.cuda_stream),
                              ctypes.byref(mt.opts), ctypes.byref(h))
    if rc != 0:
        raise pkg.MCMError(rc, "mcm_create")
    mt._h = h


def batch_partition(batch, world, rank):
    """C5: graph i of the batch goes to rank i mod world; no collective."""
    return [i for i in range(batch) if i % world == rank]


def batch_graphs(indices, scale=1.0):
    import synth

    return [synth.config("C5", scale, index=i) for i in indices]


def run_batch(args, rank, world, local_rank):
    """C5 (BASELINE configs[4]): a batch of args.batch independent 2^21 x 2^21 graphs;
    rank r solves graphs r, r+N, ... (no collective).  On one GPU the rank's graphs
    go round-robin to args.streams host threads, each with its own CUDA stream,
    workspace and handle, and each solve runs on 148 / streams CTAs -- several
    latency-bound solves share the GPU (one persistent kernel per stream).  One step
    = every graph of the rank created + solved; value = edges of all ranks' graphs /
    max over ranks of the step time."""
    import torch

    import paper_conf_icpp_devecikuc13_b200 as pkg
    import synth

    dev = torch.device("cuda", local_rank)
    torch.cuda.set_device(dev)
    mine = batch_partition(args.batch, world, rank)
    S = max(1, min(args.streams, len(mine)))
    sms = torch.cuda.get_device_properties(dev).multi_processor_count
    opts = dict(k=args.k, grid_ctas=args.solve_ctas if args.solve_ctas > 0 else max(1, sms // S))
    graphs = batch_graphs(mine)
    host = [(torch.from_numpy(g.indptr).pin_memory(), torch.from_numpy(g.indices).pin_memory()) for g in graphs]
    devg = [(a.to(dev), b.to(dev)) for a, b in host]
    streams = [torch.cuda.Stream(dev) for _ in range(S)]
    need = max(pkg.mcm_workspace_bytes(g.m, g.n, g.nnz, pkg.mcm_default_options(**opts)) for g in graphs)
    wss = [torch.empty(need, dtype=torch.uint8, device=dev) for _ in range(S)]
    rms = [torch.empty(max(g.m for g in graphs), dtype=torch.int32, device=dev) for _ in range(S)]
    cms = [torch.empty(max(g.n for g in graphs), dtype=torch.int32, device=dev) for _ in range(S)]
    flush = torch.empty(512 << 20, dtype=torch.uint8, device=dev)
    cards = [None] * len(graphs)
    stats = [None] * len(graphs)
    errors = []

    def worker(t):
        try:
            with torch.cuda.device(dev), torch.cuda.stream(streams[t]):
                for j in range(t, len(graphs), S):
                    g = graphs[j]
                    mt = pkg.Matcher.__new__(pkg.Matcher)
                    mt_init(mt, devg[j][0], devg[j][1], g, wss[t], opts, streams[t])
                    cards[j], _, _ = mt.solve(rms[t][:g.m], cms[t][:g.n], stream=streams[t])
                    stats[j] = mt.stats()
                    mt.close()
        except Exception as ex:  # surfaced after the join
            errors.append(ex)

    def worker_e2e(t):
        try:
            with torch.cuda.device(dev):
                rm_h = torch.empty(max(g.m for g in graphs), dtype=torch.int32).pin_memory()
                cm_h = torch.empty(max(g.n for g in graphs), dtype=torch.int32).pin_memory()
                for j in range(t, len(graphs), S):
                    g = graphs[j]
                    c, _, _, _ = pkg.match_host(host[j][0], host[j][1], g.m, g.n, workspace=wss[t], rmatch=rm_h[:g.m],
                                                cmatch=cm_h[:g.n], stream=streams[t], **opts)
                    if c != cards[j]:
                        errors.append(RuntimeError(f"e2e card {c} != {cards[j]} (graph {mine[j]})"))
        except Exception as ex:
            errors.append(ex)

    def step(fn):
        main = torch.cuda.current_stream(dev)
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        e0.record(main)
        for s_ in streams:
            s_.wait_event(e0)
        ths = [threading.Thread(target=fn, args=(t,)) for t in range(S)]
        for th in ths:
            th.start()
        for th in ths:
            th.join()
        if errors:
            raise errors[0]
        for s_ in streams:
            main.wait_stream(s_)
        e1.record(main)
        e1.synchronize()
        return e0.elapsed_time(e1)

    def barrier():
        if world > 1:
            torch.distributed.barrier()
        torch.cuda.synchronize(dev)

    for i in range(args.warmup):
        flush.fill_(i & 0xFF)
        step(worker)
    barrier()
    clocks = Clocks(local_rank)
    clocks.start()
    times = []
    for i in range(args.steps):
        flush.fill_(i & 0xFF)
        times.append(step(worker))
    barrier()
    clk = clocks.stop()
    for j, g in enumerate(graphs):  # parity against the closed form / oracle lives in tests; here: consistency
        if cards[j] is None or cards[j] < 0:
            raise RuntimeError(f"graph {mine[j]}: no result")
    e2e_t = []
    for i in range(args.warmup + args.steps):
        flush.fill_(i & 0xFF)
        barrier()
        t = step(worker_e2e)
        if i >= args.warmup:
            e2e_t.append(t)
    t_step = sum(times) / len(times)
    t_e2e = sum(e2e_t) / len(e2e_t)
    nnz_rank = float(sum(g.nnz for g in graphs))
    t_step_max, t_e2e_max, _, _, nnz_total = reduce_over_ranks(t_step, t_e2e, t_step, 0.0, nnz_rank, world, dev)
    if rank != 0:
        return None
    peaks = _peaks()
    hbm_peak = peaks["hbm_gbs"] if peaks else 6650.0
    alg = sum(algorithmic_bytes(st, g.m, g.n, g.nnz) for st, g in zip(stats, graphs))
    achieved = alg / (t_step * 1e-3) / 1e9
    line = {
        "metric": METRIC, "value": nnz_total / (t_step_max * 1e-3), "unit": "edges/s", "n_gpus": world,
        "steps": args.steps, "warmup": args.warmup, "ms_per_step": t_step_max, "higher_is_better": True,
        "scaling": "strong", "vs_baseline": None, "dtype": "int32", "data": "synthetic",
        "config": {"workload": f"C5: batch of {args.batch} x ({CONFIG_DESC['C5']})", "m": graphs[0].m,
                   "n": graphs[0].n, "nnz": int(nnz_total),
                   "l2": "flushed between steps (512 MiB write, outside the step events)",
                   "parallelism": f"batch over {world} GPU(s), graph i on rank i mod {world}, no collective"},
        "run": {"graphs_per_rank": len(graphs), "streams_per_gpu": S, "ctas_per_solve": opts["grid_ctas"],
                "nnz_rank0": int(nnz_rank), "cards_rank0": sorted(set(cards)), "k": args.k,
                "step": "every graph of the rank: mcm_create + mcm_solve (device-resident CSRs), S concurrent streams"},
        "roofline": {"bound": "hbm", "kernel": "gpr_kernel (all concurrent solves of a step)", "achieved": achieved,
                     "peak": hbm_peak, "unit": "GB/s", "frac": achieved / hbm_peak, "traffic": None,
                     "algorithmic_bytes_per_launch": alg // len(graphs),
                     "peak_source": "MEASURED_PEAKS.json hbm_gbs" if peaks else "fallback B200_PROFILING.md"},
        "solve_stats": {"loops_mean": statistics.mean(s_["loops"] for s_ in stats),
                        "gr_levels_mean": statistics.mean(s_["gr_levels"] for s_ in stats),
                        "ms_total_mean": statistics.mean(s_["ms_total"] for s_ in stats)},
        "clocks": clk,
        "e2e": {"value": nnz_total / (t_e2e_max * 1e-3), "unit": "edges/s",
                "h2d_bytes_per_step": int(sum(4 * (g.m + 1 + g.nnz) for g in graphs)),
                "d2h_bytes_per_step": int(sum(4 * (g.m + g.n) for g in graphs)), "ms_per_step": t_e2e_max},
        "gpu_launches": args.steps * sum(st_["kernel_launches"] for st_ in stats),
        "nccl_world_size": world,
    }
    if world == 1 and not args.no_cpu_baseline:
        line["cpu_baseline"] = cpu_baseline("C5", graphs[0])
        line["cpu_baseline"]["sample"] += " (graph 0 of the batch)"
    return line


def host_info():
    """nproc, the cores this process may use, the CPU model."""
    model = None
    try:
        for ln in open("/proc/cpuinfo"):
            if ln.startswith("model name"):
                model = ln.split(":", 1)[1].strip()
                break
    except OSError:
        pass
    try:
        allowed = sorted(os.sched_getaffinity(0))
    except AttributeError:
        allowed = list(range(os.cpu_count() or 1))
    return {"nproc": os.cpu_count(), "cores_allowed": len(allowed), "cpu_model": model}, allowed


def _pinned(fn, core, out, key):
    """Run fn() in this thread pinned to one core (ctypes releases the GIL, so two
    oracle calls run truly concurrently)."""
    try:
        os.sched_setaffinity(threading.get_native_id(), {core})
    except (AttributeError, OSError):
        pass
    t0 = time.perf_counter()
    r = fn()
    out[key] = (time.perf_counter() - t0, r)


def cpu_baseline(name, g, budget_s=60.0):
    """The oracle as it stands, on the host, rank 0 at N = 1: its sequential
    PR-FIFO (Alg. 1 + GR every 0.5(m+n) pushes, P:706-709 -- the paper's CPU
    comparison algorithm) and its Hopcroft-Karp, both from the same host cheap
    matching (computed once, timed separately, excluded like P:720-722), each
    single-threaded and pinned to its own core, the two running concurrently.  A
    reported baseline, not the target."""
    import oracle

    info, allowed = host_info()
    csc = oracle.transpose(g)
    t0 = time.perf_counter()
    _, rm0, cm0 = oracle.cheap_match(g, csc)
    t_cheap = time.perf_counter() - t0
    init = (rm0, cm0)
    runs = {"pr": [], "hk": []}
    cards = set()
    t_start = time.perf_counter()
    c_pr, c_hk = allowed[0], allowed[1 % len(allowed)]
    while True:
        out = {}
        ths = [threading.Thread(target=_pinned, args=(lambda: oracle.pr_fifo(g, k=0.5, init=init, csc=csc)[0], c_pr,
                                                      out, "pr")),
               threading.Thread(target=_pinned, args=(lambda: oracle.hopcroft_karp(g, init=init, csc=csc)[0], c_hk,
                                                      out, "hk"))]
        for th in ths:
            th.start()
        for th in ths:
            th.join()
        for k in ("pr", "hk"):
            runs[k].append(out[k][0])
            cards.add(out[k][1])
        if time.perf_counter() - t_start > budget_s * 0.5 or len(runs["pr"]) >= 3:
            break
    t_pr, t_hk = statistics.median(runs["pr"]), statistics.median(runs["hk"])
    if len(cards) != 1:
        raise RuntimeError(f"oracle disagreement {cards}")
    return {"value": g.nnz / t_pr, "unit": "edges/s", "cores": 2 if c_pr != c_hk else 1, "kind": "oracle",
            "sample": f"full {name} graph ({g.nnz} nnz), {len(runs['pr'])} run(s): PR-FIFO (value) and Hopcroft-Karp, "
                      f"single-threaded, concurrently on cores {c_pr} / {c_hk}, both from the host cheap matching",
            "pr_fifo_ms": t_pr * 1e3, "hopcroft_karp_ms": t_hk * 1e3, "hk_edges_per_s": g.nnz / t_hk,
            "cheap_match_ms": t_cheap * 1e3, "m0_card": int((rm0 >= 0).sum()), "card": cards.pop(), **info}


def run_reference(args, rank):
    if rank != 0:
        return None
    g = _graph(args.config, 0)
    times = []
    import oracle

    info, allowed = host_info()
    csc = oracle.transpose(g)
    for i in range(args.warmup + args.steps):
        t0 = time.perf_counter()
        oracle.pr_fifo(g, k=0.5, csc=csc)  # incl. the cheap matching it starts from
        dt = time.perf_counter() - t0
        if i >= args.warmup:
            times.append(dt)
    t = sum(times) / len(times)
    v = g.nnz / t
    return {
        "impl": "reference", "metric": METRIC, "value": v, "unit": "edges/s", "n_gpus": 1, "steps": args.steps,
        "warmup": args.warmup, "ms_per_step": t * 1e3, "higher_is_better": True, "scaling": "weak",
        "vs_baseline": None, "dtype": "int32", "data": "synthetic",
        "config": config_keys(args.config, g, "n/a (host run)", "host, 1 core (oracle)"),
        "cpu_baseline": {"value": v, "unit": "edges/s", "cores": 1, "kind": "oracle",
                         "sample": f"full {args.config} graph per step: cheap matching + sequential PR-FIFO "
                                   f"(k=0.5), single core", **info},
        "e2e": {"value": v, "unit": "edges/s", "h2d_bytes_per_step": 0, "d2h_bytes_per_step": 0},
    }


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--gpus", type=int, default=1)
    ap.add_argument("--steps", type=int, default=20)
    ap.add_argument("--warmup", type=int, default=3)
    ap.add_argument("--config", default="C4", choices=sorted(CONFIG_DESC))
    ap.add_argument("--impl", default="ours", choices=["ours", "reference"])
    ap.add_argument("--k", type=float, default=0.4)
    ap.add_argument("--no-cpu-baseline", action="store_true")
    ap.add_argument("--batch", type=int, default=64, help="C5: graphs in the batch")
    ap.add_argument("--streams", type=int, default=1,
                    help="C5: concurrent solve streams per GPU (the config says one; 2 measured 13 %% faster)")
    ap.add_argument("--e2e-streams", type=int, default=2,
                    help="e2e: host threads issuing mcm_match_host calls concurrently (one stream each)")
    ap.add_argument("--solve-ctas", type=int, default=0,
                    help="C5: CTAs per solve (0: SMs / streams); with streams > 1 and more CTAs than that, one "
                         "stream's creates run beside the other's solve")
    args = ap.parse_args()
    args.warmup = max(args.warmup, 3)
    world = int(os.environ.get("WORLD_SIZE", "1"))
    rank = int(os.environ.get("RANK", "0"))
    local_rank = int(os.environ.get("LOCAL_RANK", "0"))
    if args.impl == "reference":
        line = run_reference(args, rank)
        if line:
            print(json.dumps(line), flush=True)
        return
    if world > 1:
        import torch

        torch.cuda.set_device(local_rank)
        torch.distributed.init_process_group("nccl", device_id=torch.device("cuda", local_rank))
        if rank == 0:  # the driver's scaling run can check that NCCL saw every rank
            print(f"[bench] torch.distributed backend {torch.distributed.get_backend()}, world size "
                  f"{torch.distributed.get_world_size()}", file=sys.stderr, flush=True)
    line = (run_batch if args.config == "C5" else run_ours)(args, rank, world, local_rank)
    if line:
        print(json.dumps(line), flush=True)
    if world > 1:
        import torch

        torch.distributed.destroy_process_group()


if __name__ == "__main__":
    main()
