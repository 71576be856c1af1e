"""Build alternative copies of the C-ABI library with compile-time knobs (measurement only).

python tools/build_variants.py NAME:-DFOO=1,-DBAR=2 ...   -> build_variants/NAME.so
Run a tool against one with TEA_B200_LIB=build_variants/NAME.so.
"""
import os
import subprocess
import sys
from concurrent.futures import ThreadPoolExecutor

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
from paper_conf_cluster_mcintosh_smithm17_b200 import _build  # noqa: E402


def one(spec):
    name, _, flags = spec.partition(":")
    out = os.path.join(ROOT, "build_variants", name + ".so")
    cmd = _build.nvcc_cmd(out, [f for f in flags.split(",") if f])
    subprocess.run(cmd, check=True)
    return out


if __name__ == "__main__":
    os.makedirs(os.path.join(ROOT, "build_variants"), exist_ok=True)
    with ThreadPoolExecutor(4) as ex:
        for o in ex.map(one, sys.argv[1:]):
            print("built", o)
