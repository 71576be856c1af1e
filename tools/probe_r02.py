"""Round-2 probes (gpurun): host resources, NCCL two ranks on one GPU, CUPTI kernel records
inside the WHILE graph (torch.profiler), and the pointwise error of the random-deck cases."""
import json, os, subprocess, sys, time
import numpy as np
ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
out = {}
def sh(c):
    return subprocess.run(c, shell=True, capture_output=True, text=True).stdout
out["free"] = sh("free -g")
out["nproc"] = sh("nproc")
out["affinity"] = len(os.sched_getaffinity(0))
out["lscpu"] = sh("lscpu | head -20")
print(json.dumps(out, indent=1), flush=True)

import torch
import paper_conf_cluster_mcintosh_smithm17_b200 as tea
from paper_conf_cluster_mcintosh_smithm17_b200 import inputs
import oracle
oracle.build()

# --- random decks: pointwise vs normwise, and the residual bound (lambda_min(A) >= 1)
def run_g(deck, **kw):
    sk = {k: kw.pop(k) for k in ("method", "eps", "max_iters", "inner_steps") if k in kw}
    tt = tea.Tea(tea.mesh_of(deck), deck.density, deck.energy, deck.dt, **kw)
    r = tt.solve(**sk)
    u = tt.fetch(); tt.close()
    return u, r.stats
for (nx, ny, seed, dt, method, eps, its) in [(300, 200, 3, 0.004, 0, 1e-13, 20000), (1000, 777, 3, 0.004, 1, 1e-13, 20000),
                                             (257, 65, 3, 0.004, 0, 1e-13, 20000), (300, 200, 7, 0.04, 0, 0.0, 7),
                                             (300, 200, 7, 0.04, 1, 0.0, 33), (1, 97, 4, 0.04, 1, 0.0, 33),
                                             (95, 1, 4, 0.04, 1, 0.0, 33), (300, 203, 8, 0.04, 6, 0.0, 37)]:
    d = inputs.random_fields(nx, ny, seed, dt=dt)
    kw = dict(method=method, eps=eps, max_iters=its, inner_steps=7)
    uo, so, _ = oracle.run(d, steps=1, **kw)
    so = so[0]
    ug, sg = run_g(d, **kw)
    rx, ry = oracle.mesh_r(d)
    Kx, Ky = oracle.face_coefficients(nx, ny, rx, ry, d.density)
    u0 = d.density * d.energy
    rg = np.linalg.norm(u0 - oracle.apply_A(Kx, Ky, ug)); ro = np.linalg.norm(u0 - oracle.apply_A(Kx, Ky, uo))
    du = np.abs(ug - uo)
    print(f"random {nx}x{ny} m{method} eps={eps} its={sg['iterations']}/{so['iterations']} "
          f"pointwise={np.max(du/np.abs(uo)):.3e} normwise={du.max()/np.abs(uo).max():.3e} "
          f"maxabs={du.max():.3e} bound(rg+ro)={rg+ro:.3e} umin={np.abs(uo).min():.3e} umax={np.abs(uo).max():.3e}", flush=True)
