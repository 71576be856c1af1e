"""Small solves of every path, for compute-sanitizer (memcheck / racecheck / synccheck /
initcheck). Eager launches (loop mode 2) so every kernel is visible to the tool.

compute-sanitizer --tool memcheck --error-exitcode 9 python tools/sanitize.py
"""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))


def main():
    import paper_conf_cluster_mcintosh_smithm17_b200 as tea
    from paper_conf_cluster_mcintosh_smithm17_b200 import inputs
    cases = [
        (inputs.crooked_pipe(96, 70), None, dict(tb_steps=1)),
        (inputs.crooked_pipe(96, 70), None, dict(tb_steps=5)),      # fused passes forced on
        (inputs.random_fields(67, 45, 3), dict(px=2, py=2, halo_depth=3, nranks=1), {}),
        (inputs.crooked_pipe3(20, 18, 9), None, {}),
        # persistent solver (one cooperative launch; needs the device-loop mode)
        (inputs.crooked_pipe(96, 70), None, dict(persist=1, loop_mode=0)),
        (inputs.random_fields(300, 41, 5), None, dict(persist=1, loop_mode=0, tile_rows=1)),
        # fused passes across blocks with the halo exchange overlapped (second stream)
        (inputs.random_fields(90, 60, 4), dict(px=2, py=2, halo_depth=11, nranks=1),
         dict(tb_steps=5, overlap=1, _s=10, _methods=(1, 6, 7))),
        # single-reduction CPPCG, fused form: one block (pre / post passes, s = 10 and 4)
        (inputs.crooked_pipe(96, 70), None, dict(tb_steps=5, _s=10, _methods=(7,))),
        (inputs.random_fields(70, 50, 6), None, dict(tb_steps=5, _s=4, _methods=(7,))),
        (inputs.random_fields(70, 50, 6), dict(px=2, py=1, halo_depth=2, nranks=1),
         dict(_s=6, _methods=(7,))),
    ]
    for deck, dist, kw in cases:
        kw = dict(kw)
        s = kw.pop("_s", 4)
        methods = kw.pop("_methods", (0, 1, 2, 3, 4, 5, 6, 7))
        for method in methods:
            if getattr(deck, "nz", 1) > 1 and method == 2:
                continue
            if kw.get("persist") and method not in (0, 1):
                continue
            kw = dict(dict(loop_mode=2, check_interval=4), **kw)
            t = tea.Tea(tea.mesh_of(deck), deck.density, deck.energy, deck.dt, dist=dist,
                        presteps=10, **kw)
            r = t.solve(method, 1e-10, 60, s, raise_on_error=False)
            t.fetch()
            t.close()
            print(deck.name, dist, kw, method, r.status, r.stats["iterations"], flush=True)


if __name__ == "__main__":
    main()
