"""Instruction mix of the main (largest) loop of kernels in the built library (SASS):
python tools/sass_loop.py [lib.so] [name-substring ...]"""
import collections
import re
import subprocess
import sys

lib = sys.argv[1] if len(sys.argv) > 1 and sys.argv[1].endswith(".so") else \
    "paper_conf_cluster_mcintosh_smithm17_b200/libtea_b200.so"
pats = [a for a in sys.argv[1:] if not a.endswith(".so")] or ["k_cheb_tbILi5ELb0ELb0ELb1ELb1ELb0ELb0E",
                                                            "k_cheb_tbILi5ELb1ELb1ELb0ELb1ELb0ELb0E"]
txt = subprocess.run(["cuobjdump", "-sass", lib], capture_output=True, text=True).stdout
for p in re.split(r"\n\s+Function : ", txt):
    name = p.split("\n", 1)[0]
    if not any(q in name for q in pats):
        continue
    ins = []
    for l in p.split("\n"):
        m = re.search(r"/\*([0-9a-f]{4,6})\*/\s+(.*?);", l)
        if m:
            ins.append((int(m.group(1), 16), m.group(2).strip()))
    back = []
    for a, t in ins:
        m = re.search(r"BRA\s+(?:\S+\s+)?0x([0-9a-f]+)", t)
        if m and int(m.group(1), 16) < a:
            back.append((a, int(m.group(1), 16)))
    if not back:
        continue
    a, b = max(back, key=lambda x: x[0] - x[1])
    body = [t for x, t in ins if b <= x <= a]
    def op(t):
        t = re.sub(r"^@!?U?P\w+\s+", "", t)
        return t.split()[0].split(".")[0]
    c = collections.Counter(op(t) for t in body)
    dp = c["DFMA"] + c["DMUL"] + c["DADD"]
    print(f"{name[:60]} total {len(ins)} loop {len(body)} (DP {dp})")
    print("  ", sorted(c.items(), key=lambda x: -x[1])[:22])
