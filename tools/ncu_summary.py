"""Summarise a tools/profile.sh capture into profiles/: launch-list table, full-set metrics
per kernel, and the DRAM bytes per launch that bench.py reports as roofline.traffic.

python tools/ncu_summary.py r01e            # reads gpurun_out/prof_r01e/
"""
import csv
import io
import json
import os
import subprocess
import sys
from collections import defaultdict

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)


def raw_rows(rep):
    out = subprocess.check_output(["ncu", "-i", rep, "--page", "raw", "--csv"],
                                  stderr=subprocess.DEVNULL).decode()
    rows = list(csv.reader(io.StringIO(out)))
    h = rows[0]
    return [dict(zip(h, r)) for r in rows[2:]]


def f(d, k):
    try:
        return float(d.get(k, "") or "nan")
    except ValueError:
        return float("nan")


def short(name):
    return name.split("(")[0].strip()


def full_set(rep):
    res = []
    for d in raw_rows(rep):
        rd, wr = f(d, "dram__bytes_read.sum"), f(d, "dram__bytes_write.sum")
        # ncu reports MB in the raw page for these; normalise to bytes
        unit = 1e6 if rd < 1e5 else 1.0
        stalls = {k[len("smsp__average_warps_issue_stalled_"):-len("_per_issue_active.ratio")]: f(d, k)
                  for k in d if k.startswith("smsp__average_warps_issue_stalled_")
                  and k.endswith("_per_issue_active.ratio")}
        top = sorted(((v, k) for k, v in stalls.items() if v == v), reverse=True)[:4]
        res.append({
            "kernel": short(d["Kernel Name"]),
            "grid": d.get("Grid Size") or d.get("launch__grid_size"),
            "us": f(d, "gpu__time_duration.sum"),
            "dram_read_bytes": rd * unit,
            "dram_write_bytes": wr * unit,
            "l1tex_lsu_wavefronts_pct": f(d, "l1tex__data_pipe_lsu_wavefronts.avg.pct_of_peak_sustained_elapsed"),
            "shared_wavefronts": f(d, "l1tex__data_pipe_lsu_wavefronts_mem_shared.sum"),
            "issue_active_pct": f(d, "smsp__issue_active.avg.pct_of_peak_sustained_active"),
            "fp64_pipe_pct": f(d, "sm__pipe_fp64_cycles_active.avg.pct_of_peak_sustained_active"),
            "warps_active_pct": f(d, "sm__warps_active.avg.pct_of_peak_sustained_active"),
            "regs": f(d, "launch__registers_per_thread"),
            "top_stalls_per_issue": {k: round(v, 3) for v, k in top},
        })
    return res


def launch_list(path, limit=3000):
    txt = open(path).read()
    i = txt.find('"ID"')
    rows = list(csv.reader(io.StringIO(txt[i:])))
    h = rows[0]
    ki, mi, vi = h.index("Kernel Name"), h.index("Metric Name"), h.index("Metric Value")
    agg = defaultdict(lambda: [0, 0.0])
    for r in rows[1:limit + 1]:
        if len(r) <= vi or r[mi] != "gpu__time_duration.sum":
            continue
        v = float(r[vi].replace(",", ""))
        a = agg[short(r[ki])]
        a[0] += 1
        a[1] += v
    return agg


def main():
    tag = sys.argv[1]
    n = int(sys.argv[2]) if len(sys.argv) > 2 else 4096
    src = os.path.join(ROOT, "gpurun_out", f"prof_{tag}")
    prof = os.path.join(ROOT, "profiles")
    full = []
    for rep in ("full_tb.ncu-rep", "full_spmv.ncu-rep"):
        p = os.path.join(src, rep)
        if os.path.exists(p):
            full += full_set(p)
    json.dump(full, open(os.path.join(prof, f"{tag}_ncu_full_summary.json"), "w"), indent=1)
    ll = os.path.join(src, "launches.csv")
    agg = launch_list(ll) if os.path.exists(ll) else {}
    if os.path.exists(ll):
        subprocess.call(["cp", ll, os.path.join(prof, f"{tag}_launches_bench{n}.csv")])
    # the same launch list with --cache-control none (L2 not flushed between kernels: each
    # kernel pays the write-back of its predecessor's dirty lines, as inside the bench)
    llw = os.path.join(src, "launches_warm.csv")
    aggw = launch_list(llw) if os.path.exists(llw) else {}
    if os.path.exists(llw):
        subprocess.call(["cp", llw, os.path.join(prof, f"{tag}_launches_warm_bench{n}.csv")])
    import bench
    shash = bench.source_hash()
    # traffic per launch for bench.py: average over the captured launches of each class
    # kernel class of a full-set entry: template-argument prefixes of the headline's kernels
    # (the argument lists grew over the rounds: <M, FIRST, FUSE, LAST[, KG[, PRE, POST[, UPD]]]>)
    prefixes = [("k_cheb_tb<5, 1, 1, 0", "tb_first"), ("k_cheb_tb<5, 0, 0, 1", "tb_last"),
                ("k_spmv<0", "spmv"), ("k_spmv", "spmv")]

    def cls_of(name):
        for pre, c in prefixes:
            if name.startswith(pre):
                return c
        return None
    tp = os.path.join(prof, "ncu_traffic.json")
    traffic = json.load(open(tp))
    per = defaultdict(list)
    for k in full:
        name = k["kernel"].replace("void ", "")
        if cls_of(name):
            per[cls_of(name)].append((k["dram_read_bytes"] + k["dram_write_bytes"], k["kernel"]))
    for cls, v in per.items():
        ent = traffic.setdefault(f"{cls}@{n}", {})
        ent["dram_bytes_per_launch"] = int(sum(x for x, _ in v) / len(v))
        # algorithmic bytes of the form profiled (faces from g: DESIGN.md §4.13)
        ent["algorithmic_bytes_per_launch"] = {"spmv": 7, "tb_first": 6, "tb_last": 5}[cls] * 8 * n * n
        ent["kernel"] = v[0][1]
        ent["round"] = tag[1:] if tag.startswith("r") else tag
        ent["source_hash"] = shash
        ent["capture"] = f"ncu --set full, gpurun_out/prof_{tag}" + (f", summary {sys.argv[3]}" if len(sys.argv) > 3 else "")
    json.dump(traffic, open(tp, "w"), indent=1)
    tot = sum(a[1] for a in agg.values()) or 1.0
    totw = sum(a[1] for a in aggw.values()) or 1.0
    lines = [f"source hash {shash}", "",
             "| kernel | launches | mean us (cold L2) | share | mean us (warm L2) | share |",
             "|---|---|---|---|---|---|"]
    for k, (c, s) in sorted(agg.items(), key=lambda x: -x[1][1]):
        cw, sw = aggw.get(k, (0, 0.0))
        mw = ((sw / cw / 1e3 if s > 1e4 else sw / cw) if cw else float("nan"))
        lines.append(f"| {k} | {c} | {s / c / 1e3 if s > 1e4 else s / c:.1f} | {s / tot:.3f} | "
                     f"{mw:.1f} | {sw / totw:.3f} |")
    lines += ["", "| kernel | us | DRAM MB (r+w) | L1TEX lsu wavefronts % | issue % | fp64 pipe % |"
              " warps active % | regs | top stalls (per issue) |", "|---|---|---|---|---|---|---|---|---|"]
    for k in full:
        lines.append(f"| {k['kernel']} | {k['us']:.1f} | {(k['dram_read_bytes'] + k['dram_write_bytes']) / 1e6:.1f}"
                     f" | {k['l1tex_lsu_wavefronts_pct']:.1f} | {k['issue_active_pct']:.1f} | "
                     f"{k['fp64_pipe_pct']:.1f} | {k['warps_active_pct']:.1f} | {k['regs']:.0f} | "
                     + ", ".join(f"{a} {b}" for a, b in k["top_stalls_per_issue"].items()) + " |")
    print("\n".join(lines))


if __name__ == "__main__":
    main()
