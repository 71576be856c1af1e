"""Fixed-iteration solves saved to an .npz (bitwise A/B of library variants: run under each
TEA_B200_LIB, then compare the files). python tools/dump_u.py OUT.npz"""
import os
import sys

import numpy as np

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_cluster_mcintosh_smithm17_b200 as tea  # noqa: E402
from paper_conf_cluster_mcintosh_smithm17_b200 import inputs  # noqa: E402

out = {}
cases = [("pipe1024", inputs.crooked_pipe(1024), {}, tea.CPPCG),
         ("pipe1024_f1", inputs.crooked_pipe(1024), {}, tea.CPPCG1F),
         ("rand777x515", inputs.random_fields(777, 515, seed=3), {}, tea.CPPCG),
         ("pipe1024_2x4", inputs.crooked_pipe(1024),
          dict(dist=dict(rank=0, nranks=1, px=2, py=4, halo_depth=11)), tea.CPPCG),
         ("pipe1024_2x4_f1", inputs.crooked_pipe(1024),
          dict(dist=dict(rank=0, nranks=1, px=2, py=4, halo_depth=11)), tea.CPPCG1F),
         ("pipe600_rows16", inputs.crooked_pipe(600, 500), dict(tb_steps=5, tb_rows=16), tea.CPPCG)]
for name, deck, kw, m in cases:
    t = tea.Tea(tea.mesh_of(deck), deck.density, deck.energy, deck.dt, **kw)
    r = t.solve(method=m, eps=0.0, max_iters=60, inner_steps=10, raise_on_error=False)
    out[name] = t.fetch()
    out[name + "_its"] = np.array(r.stats["iterations"])
    t.close()
np.savez(sys.argv[1], **out)
print("saved", sys.argv[1], {k: v.shape for k, v in out.items() if v.ndim})
