"""NEXT-4 experiment: the 1D row-partitioned GR with one
all-gather per BFS level (paper_conf_icpp_devecikuc13_b200/pgr.py) against the
solve's own single-GPU GR (mcm_global_relabel, complete GR: gr_early=0), on the
cheap matching M0 of each config (the first, widest GR of a solve) and on a
"late" matching -- the maximum one with 64 pairs removed, whose GR is the deep,
narrow BFS of a solve's last phase (C2: hundreds of levels).

    python tools/pgr_experiment.py C2 C3 C4                 # 1 process: parts 1, 2, 4, 8 on one GPU
    torchrun --nproc-per-node N tools/pgr_experiment.py C2  # N ranks, NCCL all-gather per level

Single process: the P parts run one after another on the one device (no
collective: each writes its slice into the shared buffer), which measures the
level kernels and the level count, not the exchange.  Under torchrun every rank
runs its part and the all-gather goes over NCCL; times are CUDA events on the
default stream, max over ranks.  Every run's labels are checked equal to the
single-GPU GR's (bit-exact)."""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402
import torch.distributed as dist  # noqa: E402

import synth  # noqa: E402
import paper_conf_icpp_devecikuc13_b200 as pkg  # noqa: E402
from paper_conf_icpp_devecikuc13_b200 import pgr  # noqa: E402


def timed(fn, reps=3):
    best = None
    for _ in range(reps):
        if dist.is_initialized():
            dist.barrier()
        torch.cuda.synchronize()
        a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        a.record()
        out = fn()
        b.record()
        torch.cuda.synchronize()
        ms = a.elapsed_time(b)
        if dist.is_initialized():
            t = torch.tensor([ms], device="cuda")
            dist.all_reduce(t, op=dist.ReduceOp.MAX)
            ms = float(t.item())
        best = ms if best is None or ms < best else best
    return best, out


def main():
    world = int(os.environ.get("WORLD_SIZE", "1"))
    rank = int(os.environ.get("RANK", "0"))
    if world > 1:
        torch.cuda.set_device(int(os.environ.get("LOCAL_RANK", "0")))
        dist.init_process_group("nccl", device_id=torch.device("cuda", int(os.environ.get("LOCAL_RANK", "0"))))
    names = [a for a in sys.argv[1:] if not a.startswith("-")] or ["C2", "C3", "C4"]
    if rank == 0:
        print("| config | parts | ranks | BFS levels | ms (best of 3) | us per level | single-GPU GR ms (complete) | "
              "labels equal |")
        print("|---|---|---|---|---|---|---|---|")
    for name in names:
        g = synth.config(name)
        ip, ix = torch.from_numpy(g.indptr).cuda(), torch.from_numpy(g.indices).cuda()
        mt = pkg.Matcher(ip, ix, g.m, g.n, gr_early=0)
        _, rm0, cm0 = mt.initial_matching()
        _, rmx, cmx = mt.solve()
        gen = torch.Generator().manual_seed(7)
        drop = torch.nonzero(rmx >= 0).flatten().cpu()
        drop = drop[torch.randperm(drop.numel(), generator=gen)[:64]].cuda()
        rml, cml = rmx.clone(), cmx.clone()
        cml[rml[drop].long()] = -1
        rml[drop] = -1
        if world > 1:  # the device greedy and the solve are nondeterministic: rank 0's matchings
            for t in (rm0, cm0, rml, cml):
                dist.broadcast(t, 0)
        for tag, rm, cm in (("M0", rm0, cm0), ("late", rml, cml)):
            run_case(name, tag, g, mt, rm, cm, world, rank)
        mt.close()
    if world > 1:
        dist.destroy_process_group()


def run_case(name, tag, g, mt, rm, cm, world, rank):
    t_ref, (ml, epr, epc, erf) = timed(lambda: mt.global_relabel(rm, cm))
    for P in ([world] if world > 1 else [1, 2, 4, 8]):
        parts = [rank] if world > 1 else list(range(P))

        def run():
            ops = pgr.DeviceParts(mt, rm, cm)
            return pgr.partitioned_relabel(ops, pgr.Collective(world > 1), g.m, g.n, P, parts)

        t, (pr, pc, pml, prf, levels) = timed(run)
        ok = bool(torch.equal(pr, epr) and torch.equal(pc, epc) and pml == ml and prf == erf)
        if rank == 0:
            print(f"| {name} {tag} | {P} | {world} | {levels} | {t:.2f} | {1e3 * t / max(levels, 1):.1f} | "
                  f"{t_ref:.2f} | {ok} |", flush=True)


if __name__ == "__main__":
    main()
