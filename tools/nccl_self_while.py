"""Diagnostic: NCCL kernels (1-rank communicator, TEA_NCCL_SELF=1) inside the WHILE-conditional
graph body (TEA_NCCL_SELF_WHILE=1 keeps loop mode 0) vs chunked graphs and the device-copy
transport. Prints whether capture/instantiation/run succeed and whether the fields agree."""
import os
import sys
import time

import numpy as np

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_cluster_mcintosh_smithm17_b200 as tea  # noqa: E402
from paper_conf_cluster_mcintosh_smithm17_b200 import inputs  # noqa: E402

deck = inputs.crooked_pipe(1024)


def run(env, name, d):
    for k in ("TEA_NCCL_SELF", "TEA_NCCL_SELF_WHILE"):
        os.environ.pop(k, None)
    os.environ.update(env)
    t = tea.Tea(tea.mesh_of(deck), deck.density, deck.energy, deck.dt,
                dist=dict(rank=0, nranks=1, px=2, py=2, halo_depth=d))
    m = getattr(tea, name)
    try:
        t.solve(method=m, eps=1e-12, max_iters=20000, inner_steps=10)  # warm-up
        t.set_u(deck.density * deck.energy)
        t0 = time.perf_counter()
        r = t.solve(method=m, eps=1e-12, max_iters=20000, inner_steps=10, raise_on_error=False)
        dt = time.perf_counter() - t0
        u = t.fetch()
    finally:
        t.close()  # a failed context aborts its communicators (tea_finalize)
    return u, r, dt


for name, d in (("CPPCG", 11), ("CG", 1), ("CPPCG1F", 11)):
    base = run({}, name, d)
    for label, env in (("nccl-self chunked", {"TEA_NCCL_SELF": "1"}),
                       ("nccl-self WHILE", {"TEA_NCCL_SELF": "1", "TEA_NCCL_SELF_WHILE": "1"})):
        try:
            u, r, dt = run(env, name, d)
            print(f"{name:8s} {label:18s} status {r.status} its {r.stats['iterations']} "
                  f"(copy {base[1].stats['iterations']}) bitwise {np.array_equal(u, base[0])} "
                  f"{dt * 1e3:.1f} ms (device-copy {base[2] * 1e3:.1f} ms)", flush=True)
        except Exception as e:  # noqa: BLE001
            print(f"{name:8s} {label:18s} FAILED: {e!r}"[:400], flush=True)
