import sys, os; sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np, oracle
sys.path.insert(0,'.')
import paper_conf_cluster_mcintosh_smithm17_b200 as tea
from paper_conf_cluster_mcintosh_smithm17_b200 import inputs
for (nx,ny) in [(1,97),(2,97),(97,1),(300,200),(4,33)]:
    deck = inputs.random_fields(nx, ny, 4, dt=0.04)
    for mi in (31, 33, 40):
        u_o, st_o, _ = oracle.run(deck, steps=1, method=1, eps=0.0, max_iters=mi, inner_steps=7)
        res=[]
        for tb in (1,2,3,4,5):
            t = tea.Tea(tea.mesh_of(deck), deck.density, deck.energy, deck.dt, tb_steps=tb)
            r = t.solve(1, 0.0, mi, 7); u=t.fetch(); t.close()
            res.append(float(np.max(np.abs(u-u_o))/np.max(np.abs(u_o))))
        print(nx,ny,mi,"rnorm_ora=%.3e"%st_o[0]['rnorm'], "r0=%.3e"%st_o[0]['r0'], " ".join("tb%d=%.2e"%(i+1,e) for i,e in enumerate(res)), flush=True)
