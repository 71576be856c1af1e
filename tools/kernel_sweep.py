"""Per-kernel timing sweep (profile mode: CUDA events around every launch).

python tools/kernel_sweep.py --n 4096 --tile-rows 8,16,32,64 [--iters 50] [--method cppcg]
Prints, per tile height, the mean launch time and algorithmic GB/s of each kernel.
"""
import argparse
import json
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))

STREAMS = {"residual": 5, "spmv": 8, "update": 3, "cheb_first": 6, "cheb_step": 6,
           "cheb_last": 6}


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--n", type=int, default=4096)
    ap.add_argument("--tile-rows", default="0")
    ap.add_argument("--iters", type=int, default=50)
    ap.add_argument("--method", default="cppcg")
    ap.add_argument("--inner", type=int, default=10)
    ap.add_argument("--once", action="store_true", help="one solve, no profiling (for ncu)")
    args = ap.parse_args()
    import torch
    import paper_conf_cluster_mcintosh_smithm17_b200 as tea
    from paper_conf_cluster_mcintosh_smithm17_b200 import inputs
    deck = inputs.crooked_pipe(args.n)
    method = tea.CPPCG if args.method == "cppcg" else tea.CG
    cells = args.n * args.n
    out = {}
    for ty in [int(x) for x in args.tile_rows.split(",")]:
        t = tea.Tea(tea.mesh_of(deck), deck.density, deck.energy, deck.dt,
                    profile=not args.once, tile_rows=ty, loop_mode=2 if args.once else 0)
        t.solve(method, 0.0, args.iters, args.inner, raise_on_error=False)
        if args.once:
            t.close()
            return
        kt = t.kernel_times()
        t.close()
        row = {}
        for k, (ms, n, *_) in kt.items():
            if n == 0:
                continue
            us = 1e3 * ms / n
            gbs = STREAMS.get(k, 0) * 8 * cells / (us * 1e-6) / 1e9 if k in STREAMS else None
            row[k] = {"us": round(us, 2), "n": n, "GBs": round(gbs, 1) if gbs else None}
        out[ty] = row
        print(f"tile_rows={ty}: " + "  ".join(
            f"{k}={v['us']}us/{v['GBs']}GB/s" for k, v in row.items() if v["GBs"]), flush=True)
    print(json.dumps(out))


if __name__ == "__main__":
    main()
