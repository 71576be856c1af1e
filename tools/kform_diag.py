"""Where do kform 1 and -1 differ? (diagnostic; run under gpurun)"""
import os, sys
import numpy as np
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_cluster_mcintosh_smithm17_b200 as tea
from paper_conf_cluster_mcintosh_smithm17_b200 import inputs


def run(deck, kform, **kw):
    s = {k: kw.pop(k) for k in ("method", "eps", "max_iters", "inner_steps")}
    t = tea.Tea(tea.mesh_of(deck), deck.density, deck.energy, deck.dt, kform=kform, **kw)
    r = t.solve(raise_on_error=False, **s)
    u = t.fetch()
    t.close()
    return u, r


deck = inputs.crooked_pipe(128, 128)
for method, its, extra in [(1, 30, {}), (1, 31, {}), (1, 32, {}), (5, 10, dict(presteps=10)),
                           (5, 11, dict(presteps=10)), (5, 12, dict(presteps=10)),
                           (4, 3, dict(presteps=10))]:
    for tb in (1,):
        kw = dict(method=method, eps=0.0, max_iters=its, inner_steps=6, tb_steps=tb, persist=-1,
                  loop_mode=2, **extra)
        a, ra = run(deck, 1, **dict(kw))
        b, rb = run(deck, -1, **dict(kw))
        d = np.abs(a - b)
        i = np.unravel_index(np.argmax(d), d.shape)
        print(f"method {method} its {its}: status {ra.status}/{rb.status} it {ra.stats['iterations']}"
              f"/{rb.stats['iterations']} maxdiff {d.max():.3e} at {i} ndiff {(d > 0).sum()} "
              f"nan {np.isnan(a).sum()}/{np.isnan(b).sum()} rel {(d / np.abs(b)).max():.3e}",
              flush=True)
