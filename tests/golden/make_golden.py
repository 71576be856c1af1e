"""Write tests/golden/oracle_*.npz -- expected values for the full-size GPU parity
tests, computed by the CPU oracle ONLY (oracle/, never the CUDA path).

Each file holds, for one workload (crooked pipe, reading c12): the iteration
counts and stats of the oracle run, sum/min/max of u^{n+1}, and u at a seeded
sample of cells (plus the four corners and edge midpoints, which sit on the
ragged tails of the GPU tiles). Run from the repo root:

    python tests/golden/make_golden.py            # ~2-3 minutes on one core
"""
import os
import sys
import time

import numpy as np

ROOT = os.path.dirname(os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
sys.path.insert(0, ROOT)

import oracle  # noqa: E402
from paper_conf_cluster_mcintosh_smithm17_b200 import inputs  # noqa: E402

OUT = os.path.dirname(os.path.abspath(__file__))

CASES = {
    # name: (n, method, eps, max_iters, inner_steps)
    "pipe1024_cg": (1024, oracle.CG, 1e-12, 20000, 10),
    "pipe1024_cppcg": (1024, oracle.CPPCG, 1e-12, 20000, 10),
    "pipe4096_cg_fixed50": (4096, oracle.CG, 0.0, 50, 10),
    "pipe4096_cppcg_fixed33": (4096, oracle.CPPCG, 0.0, 33, 10),
}


def sample_idx(n, k=1024, seed=1234):
    rng = np.random.default_rng(seed)
    flat = rng.choice(n * n, size=k, replace=False)
    extra = []
    for kk in (0, n // 2, n - 1):
        for jj in (0, 1, n // 2, n - 2, n - 1):
            extra.append(kk * n + jj)
    return np.unique(np.concatenate([flat, np.array(extra)]))


def main(names):
    for name in names:
        n, method, eps, max_iters, s = CASES[name]
        t0 = time.time()
        deck = inputs.crooked_pipe(n)
        u, stats, status = oracle.run(deck, steps=1, method=method, eps=eps,
                                      max_iters=max_iters, inner_steps=s)
        idx = sample_idx(n)
        st = stats[0]
        np.savez(os.path.join(OUT, f"oracle_{name}.npz"), n=n, method=method, eps=eps,
                 max_iters=max_iters, inner_steps=s, status=status[0],
                 iterations=st["iterations"], presteps=st["presteps"], outer=st["outer"],
                 r0=st["r0"], rnorm=st["rnorm"], eig_min=st["eig_min"], eig_max=st["eig_max"],
                 sum=u.sum(), umin=u.min(), umax=u.max(), idx=idx, vals=u.ravel()[idx])
        print(f"{name}: {time.time() - t0:.1f}s its={st['iterations']} status={status[0]}",
              flush=True)


if __name__ == "__main__":
    main(sys.argv[1:] or list(CASES))
