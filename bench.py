"""bench.py -- TeaLeaf CPPCG / CG on B200: one JSON line.

Workload (BASELINE.json metric and configs[3]): the crooked-pipe deck on a
4096 x 4096 mesh, CPPCG with a 10-step Chebyshev inner loop, fp64. A "step" is
one implicit timestep: a full tea_solve (presteps + Lanczos eigen-estimate +
CPPCG outer iterations) to ||r|| < eps ||r0||, every kernel of the hot path.
Timesteps advance u^n, so step k solves from the u of step k-1.

value       solver iterations/s (CG presteps + CPPCG outer iterations, tea_stats)
            over the K timed steps, device-timed (CUDA events), max over ranks.
e2e         same metric through the C ABI with HOST buffers: each step copies
            u^n host->device (tea_set_u, pinned), solves, copies u^{n+1} back
            (tea_fetch) inside the timed region.
roofline    the dominant kernel (the Chebyshev inner step):
            algorithmic bytes per launch / its mean launch duration from a
            profiled solve (CUDA events around each launch on the library's
            stream); peak = MEASURED_PEAKS.json hbm_gbs.
cpu_baseline the CPU oracle (oracle/, serial C, 1 thread) on a bounded prefix of
            the same timestep, same unit.

Usage: python bench.py [--gpus N] [--steps K] [--warmup W] [--impl reference]
       [--n 4096] [--method cppcg|cg] [--inner 10] [--eps 1e-12] [--halo-depth d]
For N > 1 launch with torchrun (one process per GPU, NCCL).
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

import numpy as np

ROOT = os.path.dirname(os.path.abspath(__file__))
sys.path.insert(0, ROOT)

HBM_FALLBACK = 6650.0  # B200_PROFILING.md fallback, GB/s


def peaks():
    p = os.path.join(ROOT, "MEASURED_PEAKS.json")
    if os.path.exists(p):
        d = json.load(open(p))
        return float(d["hbm_gbs"]), "measured"
    return HBM_FALLBACK, "fallback"


# ------------------------------------------------------------------ clocks
class ClockSampler:
    """nvidia-smi sampling during the timed region (B200_PROFILING.md clocks line)."""

    Q = ("clocks.sm,clocks.max.sm,clocks_event_reasons.active,"
         "clocks_event_reasons.hw_slowdown,clocks_event_reasons.hw_thermal_slowdown,"
         "clocks_event_reasons.sw_thermal_slowdown,clocks_event_reasons.sw_power_cap")

    def __init__(self, index=0):
        self.index = index
        self.rows = []
        self.proc = None
        self.th = None

    def start(self):
        try:
            self.proc = subprocess.Popen(
                ["nvidia-smi", "-i", str(self.index), "--query-gpu=" + self.Q,
                 "--format=csv,noheader,nounits", "-lms", "200"],
                stdout=subprocess.PIPE, stderr=subprocess.DEVNULL, text=True)
        except OSError:
            self.proc = None
            return
        self.th = threading.Thread(target=self._read, daemon=True)
        self.th.start()

    def _read(self):
        for line in self.proc.stdout:
            parts = [x.strip() for x in line.split(",")]
            if len(parts) >= 7:
                self.rows.append(parts)

    def stop(self):
        if self.proc is None:
            return {"sm_mhz": None, "sm_max_mhz": None, "reasons": ["nvidia-smi unavailable"]}
        time.sleep(0.25)
        self.proc.terminate()
        try:
            self.proc.wait(timeout=5)
        except subprocess.TimeoutExpired:
            self.proc.kill()
        self.th.join(timeout=2)
        sm = [float(r[0]) for r in self.rows if r[0].replace(".", "").isdigit()]
        smax = [float(r[1]) for r in self.rows if r[1].replace(".", "").isdigit()]
        names = ["hw_slowdown", "hw_thermal_slowdown", "sw_thermal_slowdown", "sw_power_cap"]
        reasons = set()
        for r in self.rows:
            for i, n in enumerate(names):
                if r[3 + i].lower().startswith("active"):
                    reasons.add(n)
        return {"sm_mhz": statistics.median(sm) if sm else None,
                "sm_max_mhz": max(smax) if smax else None,
                "reasons": sorted(reasons), "samples": len(self.rows)}


# ------------------------------------------------------------------ model bytes
def cheb_step_bytes(cells):
    """Chebyshev inner step (general): reads z_{i-1}, z_{i-2}, r, Kx, Ky; writes z_i."""
    return 6 * 8 * cells


def outer_bytes(cells, s):
    """One CPPCG outer iteration: spmv 8 + update/first-step 6 +
    second step 5 + 6 per further step."""
    if s == 1:
        return (8 + 6) * 8 * cells
    return (8 + 6 + 5 + 6 * (s - 2)) * 8 * cells


def cg_iter_bytes(cells):
    """One CG iteration: spmv 8 streams + update 3 streams."""
    return 11 * 8 * cells


def load_ncu_traffic(kernel_key, n):
    p = os.path.join(ROOT, "profiles", "ncu_traffic.json")
    if not os.path.exists(p):
        return None
    d = json.load(open(p))
    e = d.get(f"{kernel_key}@{n}")
    return None if e is None else float(e["dram_bytes_per_launch"])


# ------------------------------------------------------------------ reference arm
def run_reference(args):
    import oracle
    from paper_conf_cluster_mcintosh_smithm17_b200 import inputs

    rank = int(os.environ.get("RANK", "0"))
    if rank != 0:
        return 0
    oracle.build()
    deck = make_deck(args)
    method = {"cppcg": oracle.CPPCG, "cg": oracle.CG, "bjcg": oracle.BJCG,
              "cg1": oracle.CG1, "jacobi": oracle.JACOBI, "cheby": oracle.CHEBY,
              "cppcg1": oracle.CPPCG1}[args.method]
    sample_iters = args.ref_iters
    orun = oracle.run3 if args.nz > 1 else oracle.run
    for _ in range(args.warmup):  # untimed warm-up (page-in, caches)
        orun(deck, steps=1, method=method, eps=args.eps, max_iters=1, inner_steps=args.inner)
    t_all, its, mv = 0.0, 0, 0
    for _ in range(args.steps):
        t0 = time.perf_counter()
        _, st, _ = orun(deck, steps=1, method=method, eps=args.eps, max_iters=sample_iters,
                        inner_steps=args.inner)
        t_all += time.perf_counter() - t0
        its += st[0]["iterations"]
        mv += st[0]["matvecs"]
    value = its / t_all
    sample = (f"first {sample_iters} iterations of timestep 1 ("
              + (f"30 CG presteps + {sample_iters - 30} CPPCG outer" if args.method == "cppcg"
                 else METHOD_NAME[args.method]) + ") per step, serial C oracle")
    line = {
        "impl": "reference", "metric": metric_name(args), "value": value, "unit": "iterations/s",
        "n_gpus": args.gpus, "steps": args.steps, "warmup": args.warmup,
        "ms_per_step": 1e3 * t_all / args.steps, "higher_is_better": True,
        "scaling": "strong", "vs_baseline": None, "dtype": "f64", "data": "synthetic",
        "config": config(args),
        "cpu_baseline": {"value": value, "unit": "iterations/s", "cores": 1, "kind": "oracle",
                         "sample": sample, "matvecs_per_s": mv / t_all},
        "e2e": {"value": value, "unit": "iterations/s", "h2d_bytes_per_step": 0,
                "d2h_bytes_per_step": 0},
    }
    print(json.dumps(line), flush=True)
    return 0


METHOD_NAME = {"cppcg": "CPPCG", "cg": "CG", "bjcg": "block-Jacobi PCG",
               "cg1": "single-reduction CG", "jacobi": "Jacobi", "cheby": "Chebyshev",
               "cppcg1": "single-reduction CPPCG"}


def make_deck(args):
    from paper_conf_cluster_mcintosh_smithm17_b200 import inputs
    if args.nz > 1:
        return inputs.crooked_pipe3(args.n, args.n, args.nz)
    return inputs.crooked_pipe(args.n)


def mesh_str(args):
    return f"{args.n}x{args.n}" + (f"x{args.nz}" if args.nz > 1 else "")


def metric_name(args):
    return (f"solver iterations/s, {mesh_str(args)} {METHOD_NAME[args.method]}"
            f" (time-to-solution, HBM GB/s alongside)")


def config(args):
    return {"workload": f"crooked_pipe{'3' if args.nz > 1 else ''} {mesh_str(args)} "
                        f"{'CPPCG s=' + str(args.inner) if args.method == 'cppcg' else METHOD_NAME[args.method]}"
                        f" eps={args.eps:g} 1 timestep/step",
            "mesh": [args.n, args.n] + ([args.nz] if args.nz > 1 else []),
            "method": args.method, "inner_steps": args.inner,
            "eps": args.eps, "max_iters": args.max_iters, "halo_depth": args.halo_depth,
            "dt": 0.004, "kform": ("stored Kx, Ky, Kz (3D)" if args.nz > 1 else
                                    "stored Kx, Ky" if args.kform < 0 else "g = 1/rho on the fly"),
            "l2": "inputs larger than L2 (>= 12 fp64 fields x 8 B x cells > 126 MB)"
            if args.n * args.n * max(args.nz, 1) >= 2 ** 21 else
            "working set fits in L2 (no flush)"}


# ------------------------------------------------------------------ GPU arm
def cpu_baseline(args, deck):
    import oracle
    oracle.build()
    method = {"cppcg": oracle.CPPCG, "cg": oracle.CG, "bjcg": oracle.BJCG,
              "cg1": oracle.CG1, "jacobi": oracle.JACOBI, "cheby": oracle.CHEBY,
              "cppcg1": oracle.CPPCG1}[args.method]
    t0 = time.perf_counter()
    orun = oracle.run3 if args.nz > 1 else oracle.run
    _, st, _ = orun(deck, steps=1, method=method, eps=args.eps, max_iters=args.ref_iters,
                    inner_steps=args.inner)
    dt = time.perf_counter() - t0
    return {"value": st[0]["iterations"] / dt, "unit": "iterations/s", "cores": 1,
            "kind": "oracle",
            "sample": f"first {args.ref_iters} iterations of timestep 1 ("
                      + (f"{st[0]['presteps']} CG presteps + {st[0]['outer']} CPPCG outer"
                         if args.method == "cppcg" else METHOD_NAME[args.method])
                      + f"), serial C oracle, {dt:.1f} s",
            "matvecs_per_s": st[0]["matvecs"] / dt}


def factor(n):
    best = (1, n)
    for px in range(1, n + 1):
        if n % px == 0:
            py = n // px
            if abs(px - py) < abs(best[0] - best[1]) or (abs(px - py) == abs(best[0] - best[1])
                                                         and px < best[0]):
                best = (px, py)
    return best


def run_gpu(args):
    import torch

    import paper_conf_cluster_mcintosh_smithm17_b200 as tea
    from paper_conf_cluster_mcintosh_smithm17_b200 import inputs

    world = int(os.environ.get("WORLD_SIZE", "1"))
    rank = int(os.environ.get("RANK", "0"))
    local = int(os.environ.get("LOCAL_RANK", "0"))
    torch.cuda.set_device(local)
    dev = torch.device("cuda", local)
    dist_kw = None
    pg = None
    if world > 1:
        import torch.distributed as dist
        dist.init_process_group("nccl", device_id=dev)
        pg = dist
        nid = torch.zeros(128, dtype=torch.uint8, device=dev)
        if rank == 0:
            nid.copy_(torch.frombuffer(bytearray(tea.get_nccl_id()), dtype=torch.uint8))
        dist.broadcast(nid, 0)
        px, py = factor(world)
        dist_kw = dict(rank=rank, nranks=world, px=px, py=py, halo_depth=args.halo_depth,
                       nccl_id=bytes(nid.cpu().numpy().tobytes()))

    def barrier():
        torch.cuda.synchronize()
        if pg is not None:
            pg.barrier()
            torch.cuda.synchronize()

    def max_over_ranks(x):
        if pg is None:
            return x
        t = torch.tensor([x], dtype=torch.float64, device=dev)
        pg.all_reduce(t, op=pg.ReduceOp.MAX)
        return float(t.item())

    if args.blocks and world == 1:
        bpx, bpy = (int(v) for v in args.blocks.lower().split("x"))
        dist_kw = dict(rank=0, nranks=1, px=bpx, py=bpy, halo_depth=args.halo_depth)
    deck = make_deck(args)
    method = {"cppcg": tea.CPPCG, "cg": tea.CG, "bjcg": tea.BJCG,
              "cg1": tea.CG1, "jacobi": tea.JACOBI, "cheby": tea.CHEBY,
              "cppcg1": tea.CPPCG1}[args.method]
    cells = args.n * args.n * max(args.nz, 1)
    t = tea.Tea(tea.mesh_of(deck), deck.density, deck.energy, deck.dt, dist=dist_kw,
                tile_rows=args.tile_rows, tb_steps=args.tb_steps, loop_mode=args.loop_mode,
                persist=args.persist, overlap=args.overlap, kform=args.kform)
    stream = t.stream

    def solve():
        r = t.solve(method, args.eps, args.max_iters, args.inner)
        return r.stats

    for _ in range(args.warmup):
        solve()
    barrier()
    clk = ClockSampler(local)
    clk.start()
    l0 = t.launch_count()
    ev0 = torch.cuda.Event(enable_timing=True)
    ev1 = torch.cuda.Event(enable_timing=True)
    ev0.record(stream)
    stats = [solve() for _ in range(args.steps)]
    ev1.record(stream)
    ev1.synchronize()
    launches = t.launch_count() - l0
    clocks = clk.stop()
    ms = ev0.elapsed_time(ev1)
    ms = max_over_ranks(ms)
    iters = sum(s["iterations"] for s in stats)
    outer = sum(s["outer"] for s in stats)
    matvecs = sum(s["matvecs"] for s in stats)
    value = iters / (ms * 1e-3)
    if method == tea.CPPCG:
        model_bytes = sum(5 * 8 * cells + s["presteps"] * cg_iter_bytes(cells) +
                          outer_bytes(cells, args.inner) - 10 * 8 * cells +  # restart chain
                          s["outer"] * outer_bytes(cells, args.inner) for s in stats)
    elif method == tea.CPPCG1:
        # per outer: update 10 + q = A z 4 + the chain priced at one kernel per step
        chain_st = 4 if args.inner == 1 else 4 + 5 + 6 * (args.inner - 2)
        model_bytes = sum(5 * 8 * cells + s["presteps"] * cg_iter_bytes(cells) +
                          (chain_st + 4) * 8 * cells + s["outer"] * (10 + 4 + chain_st) * 8 * cells
                          for s in stats)
    elif method in (tea.JACOBI, tea.CHEBY):
        per = 5 if method == tea.JACOBI else 6
        model_bytes = len(stats) * 5 * 8 * cells + iters * per * 8 * cells
    elif method == tea.CG1:
        model_bytes = len(stats) * 9 * 8 * cells + iters * 12 * 8 * cells
    elif method == tea.BJCG:
        model_bytes = len(stats) * 10 * 8 * cells + iters * 15 * 8 * cells
    else:
        model_bytes = len(stats) * 5 * 8 * cells + iters * cg_iter_bytes(cells)

    # ---- e2e through the C ABI with host buffers (pinned)
    u_host = torch.empty(((args.nz,) if args.nz > 1 else ()) + (args.n, args.n),
                         dtype=torch.float64).pin_memory()
    u_np = u_host.numpy()
    t.fetch(u_np)
    barrier()
    e0 = time.perf_counter()
    e_iters = 0
    for _ in range(args.steps):
        t.set_u(u_np)
        e_iters += solve()["iterations"]
        t.fetch(u_np)
    torch.cuda.synchronize()
    e_dt = max_over_ranks(time.perf_counter() - e0)
    bx = cells // world  # host bytes this rank copies per step
    e2e = {"value": e_iters / e_dt, "unit": "iterations/s", "h2d_bytes_per_step": 8 * bx,
           "d2h_bytes_per_step": 8 * bx}
    t.close()

    # ---- roofline of the dominant kernel: profiled solve (events per launch)
    tp = tea.Tea(tea.mesh_of(deck), deck.density, deck.energy, deck.dt, dist=dist_kw,
                 profile=True, tile_rows=args.tile_rows, tb_steps=args.tb_steps,
                 check_interval=2, kform=args.kform)
    tp.set_u(u_np)
    pst = tp.solve(method, args.eps, args.max_iters, args.inner).stats
    kt = tp.kernel_times()
    tp.close()
    hbm, which = peaks()
    # dominant kernel class = the largest share of the profiled solve; its achieved
    # bandwidth = the library's algorithmic bytes for those launches / their time
    kkey = max(kt, key=lambda k: kt[k][0])
    kms, kn, kbytes = kt[kkey]
    avg_ms = kms / max(kn, 1)
    achieved = kbytes / (kms * 1e-3) / 1e9
    tot_ms = sum(v[0] for v in kt.values())
    roof = {"bound": "hbm", "achieved": achieved, "peak": hbm, "unit": "GB/s",
            "frac": achieved / hbm, "traffic": load_ncu_traffic(kkey, args.n),
            "kernel": kkey, "algorithmic_bytes_per_launch": kbytes / max(kn, 1),
            "avg_launch_us": avg_ms * 1e3, "launches_profiled": kn,
            "share_of_profiled_step": kms / tot_ms if tot_ms else None,
            "peak_source": f"MEASURED_PEAKS.json hbm_gbs ({which})",
            "kernel_ms": {k: round(v[0], 3) for k, v in kt.items() if v[1]},
            "kernel_gbs": {k: round(v[2] / (v[0] * 1e-3) / 1e9, 1) for k, v in kt.items()
                           if v[1] and v[2] > 0},
            "profiled_solve_model_gbs": sum(v[2] for v in kt.values()) / (tot_ms * 1e-3) / 1e9
            if tot_ms else None}

    line = {
        "metric": metric_name(args), "value": value, "unit": "iterations/s",
        "n_gpus": world, "steps": args.steps, "warmup": args.warmup,
        "ms_per_step": ms / args.steps, "higher_is_better": True, "scaling": "strong",
        "vs_baseline": None, "dtype": "f64", "data": "synthetic (crooked pipe deck, seeded)",
        "config": dict(config(args), parallelism=(
            f"{dist_kw['px']}x{dist_kw['py']} blocks" +
            (" in one process (device-copy halos)" if dist_kw and world == 1 else "")
            if dist_kw else "1 block")),
        "time_to_solution_s": ms * 1e-3 / args.steps,
        "iterations_per_step": iters / args.steps, "outer_per_step": outer / args.steps,
        "matvecs_per_s": matvecs / (ms * 1e-3),
        # library-accounted algorithmic bytes (fused passes counted as
        # what they move), per iteration from the profiled solve, over the timed region
        "hbm_gbs_model": (sum(v[2] for v in kt.values()) / max(pst["iterations"], 1)) * iters
        / (ms * 1e-3) / 1e9,
        # the same work priced at one kernel per Chebyshev step (6 streams / step):
        # an "effective bandwidth" that exceeds the HBM peak when fusion saves bytes
        "hbm_gbs_unfused_equiv": model_bytes / (ms * 1e-3) / 1e9,
        "e2e": e2e, "gpu_launches": launches, "clocks": clocks, "roofline": roof,
    }
    if rank == 0 and world == 1 and not args.no_cpu:
        line["cpu_baseline"] = cpu_baseline(args, deck)
    if rank == 0:
        print(json.dumps(line), flush=True)
    if pg is not None:
        pg.barrier()
        pg.destroy_process_group()
    return 0


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--gpus", type=int, default=1)
    ap.add_argument("--steps", type=int, default=5)
    ap.add_argument("--warmup", type=int, default=3)
    ap.add_argument("--impl", default="b200", choices=["b200", "reference"])
    ap.add_argument("--n", type=int, default=4096)
    ap.add_argument("--nz", type=int, default=0,
                    help="> 1: the 3D 7-point problem on n x n x nz (SURVEY NEXT-4)")
    ap.add_argument("--method", default="cppcg", choices=["cppcg", "cg", "bjcg", "cg1", "jacobi", "cheby",
                                                   "cppcg1"])
    ap.add_argument("--inner", type=int, default=10)
    ap.add_argument("--eps", type=float, default=1e-12)
    ap.add_argument("--max-iters", type=int, default=0,
                    help="0 = 100000 (Krylov methods) or 2000 (jacobi/cheby: a fixed-work "
                         "throughput run; they need O(kappa) iterations at 4096^2)")
    ap.add_argument("--halo-depth", type=int, default=0,
                    help="0 = auto: inner+1 for CPPCG (one deep exchange per outer, fused "
                         "passes on extended bounds), 1 otherwise")
    ap.add_argument("--blocks", default="",
                    help="PXxPY: run the px x py decomposition inside ONE process on one GPU "
                         "(the multi-GPU code path with device-copy halos instead of NCCL)")
    ap.add_argument("--tile-rows", type=int, default=0)
    ap.add_argument("--persist", type=int, default=0,
                    help="whole solve in one cooperative launch: 1 on, 0 (auto) or -1 off "
                         "(tea_opts.persist)")
    ap.add_argument("--overlap", type=int, default=0,
                    help="halo exchange of the fused passes overlapped with the interior on "
                         "a second stream: 1 on, -1 off, 0 auto = on across processes "
                         "(tea_opts.overlap)")
    ap.add_argument("--kform", type=int, default=0,
                    help="2D faces formed on the fly from g = 1/rho (1, auto 0) or read as stored "
                         "Kx, Ky (-1) (tea_opts.kform)")
    ap.add_argument("--tb-steps", type=int, default=0,
                    help="Chebyshev steps per fused HBM pass (0 auto=4, 1 = per-step kernels)")
    ap.add_argument("--loop-mode", type=int, default=0,
                    help="0 WHILE graph, 1 chunked graphs (ncu can profile), 2 eager")
    ap.add_argument("--ref-iters", type=int, default=31)
    ap.add_argument("--no-cpu", action="store_true")
    args = ap.parse_args()
    if args.warmup < 3:
        ap.error("--warmup must be >= 3")
    if args.halo_depth == 0:
        args.halo_depth = args.inner + 1 if args.method in ("cppcg", "cppcg1") else 1
    if args.max_iters == 0:
        args.max_iters = 2000 if args.method in ("jacobi", "cheby") else 100000
    if args.impl == "reference":
        return run_reference(args)
    return run_gpu(args)


if __name__ == "__main__":
    sys.exit(main())
