"""Solve-time vs kernel-time probe: fixed-iteration CPPCG solves in each loop mode.

python tools/gap_probe.py --n 4096 --iters 130
"""
import argparse
import os
import sys
import time

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--n", type=int, default=4096)
    ap.add_argument("--iters", type=int, default=130)
    ap.add_argument("--inner", type=int, default=10)
    ap.add_argument("--method", default="cppcg")
    ap.add_argument("--tile-rows", default="0")
    args = ap.parse_args()
    import torch
    import paper_conf_cluster_mcintosh_smithm17_b200 as tea
    from paper_conf_cluster_mcintosh_smithm17_b200 import inputs
    deck = inputs.crooked_pipe(args.n)
    method = tea.CPPCG if args.method == "cppcg" else tea.CG
    for ty in [int(x) for x in args.tile_rows.split(",")]:
        res = {}
        for mode, ci in ((0, 0), (1, 16), (1, 64), (2, 16)):
            t = tea.Tea(tea.mesh_of(deck), deck.density, deck.energy, deck.dt, loop_mode=mode,
                        check_interval=ci, tile_rows=ty)
            t.solve(method, 0.0, args.iters, args.inner, raise_on_error=False)  # warm / capture
            ts = []
            for _ in range(3):
                t.set_u(deck.density * deck.energy)
                r = t.solve(method, 0.0, args.iters, args.inner, raise_on_error=False)
                ts.append(r.stats["seconds"])
            l = t.launch_count()
            t.close()
            res[(mode, ci)] = min(ts)
        # profiled (eager + events): pure kernel time
        t = tea.Tea(tea.mesh_of(deck), deck.density, deck.energy, deck.dt, profile=True,
                    check_interval=2, tile_rows=ty)
        t.solve(method, 0.0, args.iters, args.inner, raise_on_error=False)
        kt = t.kernel_times(reset=True)
        t.set_u(deck.density * deck.energy)
        t.solve(method, 0.0, args.iters, args.inner, raise_on_error=False)
        kt = t.kernel_times()
        t.close()
        ksum = sum(v[0] for v in kt.values()) * 1e-3
        print(f"tile_rows={ty} n={args.n} iters={args.iters}: " +
              " ".join(f"mode{m}/ci{c}={v*1e3:.2f}ms" for (m, c), v in res.items()) +
              f" kernel_sum={ksum*1e3:.2f}ms  " +
              " ".join(f"{k}={1e3*v[0]/max(v[1],1):.1f}us(x{v[1]})" for k, v in kt.items() if v[1]),
              flush=True)


if __name__ == "__main__":
    main()
