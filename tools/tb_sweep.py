"""Fused-pass sweep: fixed-iteration CPPCG (30 presteps + K outer) timed in graph mode
for tb_steps x tb_rows, plus a profiled solve for per-class GB/s.

python tools/tb_sweep.py --n 4096 --steps 1,2,3,4,5 --rows 0
"""
import argparse
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--n", type=int, default=4096)
    ap.add_argument("--iters", type=int, default=130)
    ap.add_argument("--inner", type=int, default=10)
    ap.add_argument("--steps", default="1,2,3,4,5")
    ap.add_argument("--rows", default="0")
    args = ap.parse_args()
    import paper_conf_cluster_mcintosh_smithm17_b200 as tea
    from paper_conf_cluster_mcintosh_smithm17_b200 import inputs
    deck = inputs.crooked_pipe(args.n)
    u0 = deck.density * deck.energy
    for tb in [int(x) for x in args.steps.split(",")]:
        for rows in [int(x) for x in args.rows.split(",")]:
            t = tea.Tea(tea.mesh_of(deck), deck.density, deck.energy, deck.dt, tb_steps=tb,
                        tb_rows=rows)
            t.solve(tea.CPPCG, 0.0, args.iters, args.inner, raise_on_error=False)
            best = 1e9
            for _ in range(3):
                t.set_u(u0)
                r = t.solve(tea.CPPCG, 0.0, args.iters, args.inner, raise_on_error=False)
                best = min(best, r.stats["seconds"])
            t.close()
            t = tea.Tea(tea.mesh_of(deck), deck.density, deck.energy, deck.dt, tb_steps=tb,
                        tb_rows=rows, profile=True, check_interval=2)
            t.solve(tea.CPPCG, 0.0, args.iters, args.inner, raise_on_error=False)
            kt = t.kernel_times()
            t.close()
            outer = args.iters - 30
            print(f"n={args.n} tb={tb} rows={rows}: solve={best*1e3:.2f}ms "
                  f"per_outer~{(best*1e3 - 30*0.26*(args.n/4096)**2)/outer*1e3:.0f}us  " +
                  "  ".join(f"{k}={1e3*v[0]/v[1]:.1f}us/{v[2]/(v[0]*1e-3)/1e9:.0f}GB/s(x{v[1]})"
                            for k, v in kt.items() if v[1] and v[2] > 0), flush=True)


if __name__ == "__main__":
    main()
