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
roofline    the dominant kernel = the kernel class with the largest share of the
            timed region's device time: algorithmic bytes per launch (DESIGN.md
            §4 model) / its mean launch duration, both taken INSIDE the timed
            WHILE-graph solves by the library's in-graph timing (tea_opts.trace:
            %globaltimer at each launch's start and at its last CTA's end;
            no-op launches after convergence and the finalising u update are
            not counted); peak = MEASURED_PEAKS.json hbm_gbs; traffic = ncu
            DRAM bytes per launch from profiles/ncu_traffic.json, used only when
            its recorded source hash matches the built library's sources.
cpu_baseline the CPU oracle (oracle/, serial C, 1 thread) timed on bounded
            samples of the same timestep (30 presteps; + the restart and 1 outer
            iteration; + 2 more outer iterations), its per-phase costs weighted by
            the GPU run's own iteration mix (like for like), and matvecs/s.

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


def source_hash():
    """sha256 (16 hex) of the CUDA library's sources: stamps ncu-derived numbers."""
    import hashlib
    h = hashlib.sha256()
    base = os.path.join(ROOT, "paper_conf_cluster_mcintosh_smithm17_b200", "csrc")
    for f in sorted(os.listdir(base)) + ["../../include/tea.h"]:
        if f.endswith((".cu", ".h")):
            h.update(open(os.path.join(base, f), "rb").read())
    return h.hexdigest()[:16]


def load_ncu_traffic(kernel_key, n):
    """ncu DRAM bytes per launch of kernel class `kernel_key` at mesh n, if captured from
    the current sources (profiles/ncu_traffic.json entries carry the source hash)."""
    p = os.path.join(ROOT, "profiles", "ncu_traffic.json")
    if not os.path.exists(p):
        return None, "no profiles/ncu_traffic.json"
    e = json.load(open(p)).get(f"{kernel_key}@{n}")
    if e is None:
        return None, f"no capture of {kernel_key}@{n}"
    if e.get("source_hash") != source_hash():
        return None, f"capture of {kernel_key}@{n} is from other sources ({e.get('source_hash')})"
    return float(e["dram_bytes_per_launch"]), f"profiles/ncu_traffic.json ({e.get('capture')})"


def cpu_info():
    info = {}
    try:
        for line in open("/proc/cpuinfo"):
            k, _, v = line.partition(":")
            k = k.strip()
            if k in ("model name", "cpu family", "model") and k not in info:
                info[k] = v.strip()
            if len(info) == 3:
                break
    except OSError:
        pass
    return {"cpu_model": f"{info.get('model name', 'unknown')} (family {info.get('cpu family', '?')}"
                         f" model {info.get('model', '?')})",
            "host_cores_available": len(os.sched_getaffinity(0)), "oracle_threads": 1}


# ------------------------------------------------------------------ oracle timing
TWO_PHASE = ("cppcg", "cppcg1", "cppcg1f", "cheby")
# iteration mix of one timestep of the headline workload on the GPU (4096^2 pipe CPPCG s=10,
# eps 1e-12, timesteps 6-25 of the bench: 30 presteps + 253.1 outer, profiles/r01j_bench.json;
# the oracle's counts agree within +-2, tests/test_gpu_parity.py): used by the reference arm,
# which cannot run the GPU, to weight its per-phase costs like the GPU arm's cpu_baseline
HEADLINE_MIX = (30.0, 253.1)


def oracle_phase_costs(args, deck):
    """Serial oracle costs of the phases of one timestep, measured on bounded samples:
    two-phase methods run 30 presteps, then 30 + restart + 1 outer, then + 2 more outer
    (t_pre per prestep, t_restart = eigen-estimate + restart chain, t_outer per outer);
    one-phase methods run 20 iterations. Solve time only (faces precomputed)."""
    import oracle
    oracle.build()
    method = {"cppcg": oracle.CPPCG, "cg": oracle.CG, "bjcg": oracle.BJCG,
              "cg1": oracle.CG1, "jacobi": oracle.JACOBI, "cheby": oracle.CHEBY,
              "cppcg1": oracle.CPPCG1, "cppcg1f": oracle.CPPCG1F}[args.method]
    if args.nz > 1:
        rx, ry, rz = oracle.mesh_r3(deck)
        K = oracle.face_coefficients3(deck.nx, deck.ny, deck.nz, rx, ry, rz, deck.density)

        def solve(its):
            return oracle.solve3(*K, deck.density * deck.energy, None, method, args.eps, its,
                                 args.inner)
    else:
        rx, ry = oracle.mesh_r(deck)
        K = oracle.face_coefficients(deck.nx, deck.ny, rx, ry, deck.density)

        def solve(its):
            return oracle.solve(*K, deck.density * deck.energy, None, method, args.eps, its,
                                args.inner)

    def timed(its):
        t0 = time.perf_counter()
        r = solve(its)
        return time.perf_counter() - t0, r.stats

    if args.method in TWO_PHASE:
        # the per-outer cost from a 2-outer difference: a 1-outer difference of two ~7 s runs
        # was noise-dominated at 4096^2 (0.44 vs 0.92 s/outer in two runs on one box, round 2)
        t30, s30 = timed(30)
        t31, s31 = timed(31)
        t33, s33 = timed(33)
        t_outer = (t33 - t31) / 2
        c = {"t_pre": t30 / 30, "t_restart": max(t31 - t30 - t_outer, 0.0), "t_outer": t_outer,
             "sample_s": t30 + t31 + t33, "matvecs_per_s": (s30["matvecs"] + s31["matvecs"] +
                                                          s33["matvecs"]) / (t30 + t31 + t33),
             "sample": "30 presteps; 30 presteps + restart + 1 outer; + 2 more outer"}
    else:
        t20, s20 = timed(20)
        c = {"t_it": t20 / 20, "sample_s": t20, "matvecs_per_s": s20["matvecs"] / t20,
             "sample": "20 iterations"}
    return c


def cpu_time_for_mix(c, presteps, outer, iters):
    """Oracle seconds for one timestep with the given iteration mix (per-phase costs)."""
    if "t_pre" in c:
        return presteps * c["t_pre"] + (c["t_restart"] if outer > 0 else 0.0) + outer * c["t_outer"]
    return iters * c["t_it"]


# ------------------------------------------------------------------ reference arm
def run_reference(args):
    """The reference arm for this tier: the CPU oracle as it stands, 1 thread, on the same
    workload. Warm-up 1 measures its per-phase costs (oracle_phase_costs); each timed step
    re-times the 31-iteration sample (30 presteps + restart + 1 outer) and is charged the
    CPU time of a full timestep of the headline's iteration mix scaled by it."""
    rank = int(os.environ.get("RANK", "0"))
    if rank != 0:
        return 0
    import oracle
    oracle.build()
    deck = make_deck(args)
    method = {"cppcg": oracle.CPPCG, "cg": oracle.CG, "bjcg": oracle.BJCG,
              "cg1": oracle.CG1, "jacobi": oracle.JACOBI, "cheby": oracle.CHEBY,
              "cppcg1": oracle.CPPCG1, "cppcg1f": oracle.CPPCG1F}[args.method]
    orun = oracle.run3 if args.nz > 1 else oracle.run
    costs = oracle_phase_costs(args, deck)  # (part of the warm-up)
    two = "t_pre" in costs
    mix = (HEADLINE_MIX if (args.method == "cppcg" and args.n == 4096 and args.inner == 10
                            and args.nz <= 1) else None)
    sample_iters = 31 if two else 20
    t_sample_warm = None
    for _ in range(max(args.warmup - 1, 1)):
        t0 = time.perf_counter()
        orun(deck, steps=1, method=method, eps=args.eps, max_iters=sample_iters,
             inner_steps=args.inner)
        t_sample_warm = time.perf_counter() - t0
    t_all, t_charged, its, mv = 0.0, 0.0, 0.0, 0
    for _ in range(args.steps):
        t0 = time.perf_counter()
        _, st, _ = orun(deck, steps=1, method=method, eps=args.eps, max_iters=sample_iters,
                        inner_steps=args.inner)
        dt = time.perf_counter() - t0
        t_all += dt
        mv += st[0]["matvecs"]
        if mix is not None:
            t_charged += cpu_time_for_mix(costs, mix[0], mix[1], 0) * dt / t_sample_warm
            its += mix[0] + mix[1]
        else:
            t_charged += dt
            its += st[0]["iterations"]
    value = its / t_charged
    sample = (f"{sample_iters} iterations of timestep 1 per step (serial C oracle, 1 thread)"
              + (f", charged as a full timestep of the GPU's iteration mix ({mix[0]:g} presteps"
                 f" + {mix[1]:g} outer) from the oracle's per-phase costs ({costs['sample']}:"
                 f" {costs['t_pre']:.3f} s/prestep, restart {costs['t_restart']:.2f} s,"
                 f" {costs['t_outer']:.2f} s/outer)" if mix else ""))
    line = {
        "impl": "reference", "metric": metric_name(args), "value": value, "unit": "iterations/s",
        "n_gpus": args.gpus, "steps": args.steps, "warmup": args.warmup,
        "ms_per_step": 1e3 * t_all / args.steps, "higher_is_better": True,
        "scaling": "strong", "vs_baseline": None, "dtype": "f64", "data": "synthetic",
        "config": config(args),
        "cpu_baseline": dict({"value": value, "unit": "iterations/s", "cores": 1,
                              "kind": "oracle", "sample": sample,
                              "matvecs_per_s": mv / t_all}, **cpu_info()),
        "e2e": {"value": value, "unit": "iterations/s", "h2d_bytes_per_step": 0,
                "d2h_bytes_per_step": 0},
    }
    print(json.dumps(line), flush=True)
    return 0


METHOD_NAME = {"cppcg": "CPPCG", "cg": "CG", "bjcg": "block-Jacobi PCG",
               "cg1": "single-reduction CG", "jacobi": "Jacobi", "cheby": "Chebyshev",
               "cppcg1": "single-reduction CPPCG",
               "cppcg1f": "single-reduction CPPCG (fused form)"}


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
def cpu_baseline(args, deck, stats):
    """The oracle (1 thread) like for like: its measured per-phase costs weighted by this
    run's own iteration mix (presteps / outer iterations per timestep, averaged)."""
    c = oracle_phase_costs(args, deck)
    k = len(stats)
    pre = sum(s["presteps"] for s in stats) / k
    outer = sum(s["outer"] for s in stats) / k
    iters = sum(s["iterations"] for s in stats) / k
    t_step = cpu_time_for_mix(c, pre, outer, iters)
    mix = (f"{pre:g} presteps + {outer:g} outer" if "t_pre" in c else f"{iters:g} iterations")
    return dict({"value": iters / t_step, "unit": "iterations/s", "cores": 1, "kind": "oracle",
                 "sample": f"serial C oracle timed on {c['sample']} of timestep 1 "
                           f"({c['sample_s']:.1f} s); per-phase costs weighted by this run's "
                           f"mix per timestep ({mix}): {t_step:.1f} s per timestep "
                           "(extrapolated)",
                 "matvecs_per_s": c["matvecs_per_s"],
                 "phase_costs_s": {k2: round(v, 4) for k2, v in c.items()
                                   if k2.startswith("t_")}}, **cpu_info())


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
              "cppcg1": tea.CPPCG1, "cppcg1f": tea.CPPCG1F}[args.method]
    cells = args.n * args.n * max(args.nz, 1)
    t = tea.Tea(tea.mesh_of(deck), deck.density, deck.energy, deck.dt, dist=dist_kw,
                tile_rows=args.tile_rows, tb_steps=args.tb_steps, tb_rows=args.tb_rows,
                loop_mode=args.loop_mode,
                persist=args.persist, overlap=args.overlap, kform=args.kform,
                trace=not args.no_trace)
    stream = t.stream

    def solve():
        r = t.solve(method, args.eps, args.max_iters, args.inner)
        return r.stats

    for _ in range(args.warmup):
        solve()
    barrier()
    if not args.no_trace:
        t.trace(reset=True)  # in-graph kernel timing: the timed region only
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

    tr = [] if args.no_trace else t.trace(reset=True)

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

    # ---- roofline of the dominant kernel, from the in-graph timing of the timed region:
    # per (kernel class, algorithmic bytes per launch) slot, the launches that did their
    # work and their summed device time; dominant = the largest share of the kernel time
    hbm, which = peaks()
    cls = {}
    for kname, bpl, n, kms in tr:
        e = cls.setdefault(kname, [0.0, 0, 0.0])
        e[0] += kms
        e[1] += n
        e[2] += bpl * n
    roof = None
    if cls:
        tot_ms = sum(v[0] for v in cls.values())
        kkey = max(cls, key=lambda k: cls[k][0])
        kms, kn, kbytes = cls[kkey]
        traffic, traffic_src = load_ncu_traffic(kkey, args.n)
        achieved = kbytes / (kms * 1e-3) / 1e9
        roof = {"bound": "hbm", "achieved": achieved, "peak": hbm, "unit": "GB/s",
                "frac": achieved / hbm, "traffic": traffic, "traffic_source": traffic_src,
                "kernel": kkey, "algorithmic_bytes_per_launch": kbytes / max(kn, 1),
                "avg_launch_us": kms / max(kn, 1) * 1e3, "launches_timed": kn,
                "share_of_kernel_time": kms / tot_ms, "kernel_time_of_step": tot_ms / ms,
                "timing": "in-graph (tea_opts.trace: %globaltimer at launch start / last CTA "
                          "end), the K timed WHILE-graph timesteps",
                "peak_source": f"MEASURED_PEAKS.json hbm_gbs ({which})",
                "kernel_ms": {k: round(v[0], 3) for k, v in cls.items()},
                "kernel_avg_us": {k: round(v[0] / max(v[1], 1) * 1e3, 1) for k, v in cls.items()},
                "kernel_gbs": {k: round(v[2] / (v[0] * 1e-3) / 1e9, 1) for k, v in cls.items()
                               if v[2] > 0 and v[0] > 0},
                "model_gbs_timed_region": sum(v[2] for v in cls.values()) / (ms * 1e-3) / 1e9}

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
        # library-accounted algorithmic bytes of the launches timed in-graph (
        # fused passes counted as what they move) over the timed region
        "hbm_gbs_model": roof["model_gbs_timed_region"] if roof else None,
        # the same work priced at one kernel per Chebyshev step (6 streams / step):
        # an "effective bandwidth" that exceeds the HBM peak when fusion saves bytes
        "hbm_gbs_unfused_equiv": model_bytes / (ms * 1e-3) / 1e9,
        "e2e": e2e, "gpu_launches": launches, "clocks": clocks, "roofline": roof,
    }
    # the same workload by the single-reduction CPPCG in fused form (TEA_CPPCG1F, SURVEY NEXT-2:
    # one reduction and two fused kernels per outer iteration), same steps and timing
    if args.method == "cppcg" and not args.no_variants:
        tv = tea.Tea(tea.mesh_of(deck), deck.density, deck.energy, deck.dt, dist=dist_kw,
                     tile_rows=args.tile_rows, tb_steps=args.tb_steps, tb_rows=args.tb_rows,
                     loop_mode=args.loop_mode, persist=args.persist, overlap=args.overlap,
                     kform=args.kform, trace=not args.no_trace)
        for _ in range(args.warmup):
            tv.solve(tea.CPPCG1F, args.eps, args.max_iters, args.inner)
        barrier()
        if not args.no_trace:
            tv.trace(reset=True)
        v0 = torch.cuda.Event(enable_timing=True)
        v1 = torch.cuda.Event(enable_timing=True)
        v0.record(tv.stream)
        vst = [tv.solve(tea.CPPCG1F, args.eps, args.max_iters, args.inner).stats
               for _ in range(args.steps)]
        v1.record(tv.stream)
        v1.synchronize()
        vms = max_over_ranks(v0.elapsed_time(v1))
        vtr = [] if args.no_trace else tv.trace()
        tv.close()
        vcls = {}
        for kname, bpl, n, kms in vtr:
            e = vcls.setdefault(kname, [0.0, 0])
            e[0] += kms
            e[1] += n
        line["variants"] = {"cppcg1f": {
            "method": "single-reduction CPPCG, fused form (TEA_CPPCG1F)",
            "value": sum(x["iterations"] for x in vst) / (vms * 1e-3), "unit": "iterations/s",
            "ms_per_step": vms / args.steps,
            "iterations_per_step": sum(x["iterations"] for x in vst) / args.steps,
            "kernel_avg_us": {k: round(v[0] / max(v[1], 1) * 1e3, 1) for k, v in vcls.items()}}}
    if rank == 0 and world == 1 and not args.no_cpu:
        line["cpu_baseline"] = cpu_baseline(args, deck, stats)
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
                                                   "cppcg1", "cppcg1f"])
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
    ap.add_argument("--tb-rows", type=int, default=0, help="output rows per fused-pass tile (0 auto)")
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
    ap.add_argument("--no-trace", action="store_true",
                    help="time without the in-graph kernel timing (no roofline block)")
    ap.add_argument("--no-cpu", action="store_true")
    ap.add_argument("--no-variants", action="store_true",
                    help="skip the CPPCG1F line of the headline run")
    args = ap.parse_args()
    if args.warmup < 3:
        ap.error("--warmup must be >= 3")
    if args.halo_depth == 0:
        args.halo_depth = args.inner + 1 if args.method in ("cppcg", "cppcg1", "cppcg1f") else 1
    if args.max_iters == 0:
        args.max_iters = 2000 if args.method in ("jacobi", "cheby") else 100000
    if args.impl == "reference":
        return run_reference(args)
    return run_gpu(args)


if __name__ == "__main__":
    sys.exit(main())
