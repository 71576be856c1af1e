import ctypes, sys
sys.path.insert(0, '.')
import torch
torch.cuda.init()
L = ctypes.CDLL("paper_conf_cluster_mcintosh_smithm17_b200/libtea_b200.so")
f = getattr(L, "_ZN3tea12tb_auto_rowsEiii")
f.restype = ctypes.c_int
for (nl, w, h) in [(5, 2060, 1036), (5, 2050, 1026), (5, 4096, 4096), (5, 1024, 1024), (6, 4096, 4096), (5, 16384, 16384)]:
    print(nl, w, h, f(nl, w, h))
