"""bench.py contract checks that run without a GPU: the reference arm (the CPU oracle,
per the tier rules) prints one JSON line with the required keys; argument checks."""
import json
import os
import subprocess
import sys

import pytest

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def run(*args, env=None):
    out = subprocess.run([sys.executable, os.path.join(ROOT, "bench.py"), *args],
                         capture_output=True, text=True, timeout=300, cwd=ROOT, env=env)
    return out


@pytest.mark.parametrize("extra", [["--method", "cppcg"], ["--method", "cg", "--nz", "16"],
                                   ["--method", "bjcg"], ["--method", "jacobi"]])
def test_reference_arm_json(extra):
    out = run("--impl", "reference", "--n", "48", "--steps", "1", "--warmup", "3", *extra)
    assert out.returncode == 0, out.stderr
    line = json.loads(out.stdout.strip().splitlines()[-1])
    for k in ("metric", "value", "unit", "n_gpus", "steps", "warmup", "ms_per_step",
              "higher_is_better", "scaling", "dtype", "config", "cpu_baseline", "e2e"):
        assert k in line, k
    assert line["impl"] == "reference" and line["value"] > 0
    assert line["cpu_baseline"]["kind"] == "oracle" and line["cpu_baseline"]["cores"] == 1
    assert line["cpu_baseline"]["oracle_threads"] == 1 and "cpu_model" in line["cpu_baseline"]
    assert line["e2e"]["h2d_bytes_per_step"] == 0
    assert "workload" in line["config"]


def test_reference_arm_nonzero_rank_exits_quietly():
    env = dict(os.environ, RANK="1", WORLD_SIZE="2")
    out = run("--impl", "reference", "--n", "32", "--steps", "1", "--warmup", "3", env=env)
    assert out.returncode == 0 and out.stdout.strip() == ""


def test_warmup_must_be_at_least_3():
    out = run("--impl", "reference", "--n", "32", "--steps", "1", "--warmup", "2")
    assert out.returncode != 0


def test_headline_reference_weights_the_gpu_mix():
    """The 4096^2 CPPCG reference arm charges each step a full timestep of the headline's
    iteration mix (like for like with the GPU arm's iterations/s), from per-phase costs."""
    import bench
    c = {"t_pre": 0.1, "t_restart": 1.0, "t_outer": 1.2}
    t = bench.cpu_time_for_mix(c, 30, 253.1, 0)
    assert t == pytest.approx(30 * 0.1 + 1.0 + 253.1 * 1.2)
    assert bench.cpu_time_for_mix({"t_it": 0.5}, 0, 0, 40) == pytest.approx(20.0)
