"""Golden pins from an independent computation (SURVEY.md Appendix [S2], [S3]).

The survey ran its own numpy CG / CPPCG on the crooked-pipe deck before
oracle/ existed; its iteration counts, extrema and Ritz values are fixed here
(tests/golden/survey_appendix.json, with the citation inside). Iteration counts
are allowed +-2 (BASELINE.json north_star), the rest to the printed precision.
"""
import json
import os

import numpy as np
import pytest

from paper_conf_cluster_mcintosh_smithm17_b200 import inputs

G = json.load(open(os.path.join(os.path.dirname(__file__), "golden", "survey_appendix.json")))


def test_s2_cg_128_ten_steps(ora):
    g = G["S2_cg_128_10steps"]
    u, stats, status = ora.run(inputs.crooked_pipe(128), steps=10, method=0, eps=g["eps"])
    assert status == [0] * 10
    its = [s["iterations"] for s in stats]
    assert np.abs(np.array(its) - np.array(g["iterations"])).max() <= 2
    assert u.max() == pytest.approx(g["u_max_final"], abs=5e-4)
    assert u.min() == pytest.approx(g["u_min_final"], abs=5e-4)


@pytest.mark.parametrize("n", [128, 256])
def test_s3_cppcg_counts(ora, n):
    g = G["S3_cppcg_s10"][str(n)]
    d = inputs.crooked_pipe(n)
    _, st, status = ora.run(d, steps=1, method=1, eps=1e-15, inner_steps=10)
    assert status == [0]
    assert abs(st[0]["outer"] - g["outer"]) <= 2
    assert abs(st[0]["matvecs"] - g["matvecs"]) <= 2 * 11
    _, st_cg, _ = ora.run(d, steps=1, method=0, eps=1e-15)
    assert abs(st_cg[0]["iterations"] - g["cg_iterations"]) <= 2


def test_s3_cppcg_s5_and_ritz(ora):
    d = inputs.crooked_pipe(128)
    _, st, _ = ora.run(d, steps=1, method=1, eps=1e-15, inner_steps=5)
    g = G["S3_cppcg_s5_128"]
    assert abs(st[0]["outer"] - g["outer"]) <= 2
    _, st, _ = ora.run(d, steps=1, method=1, eps=1e-15, inner_steps=10)
    assert st[0]["eig_max"] == pytest.approx(G["S1_lmax_after_margin_128"], abs=0.005)
    assert st[0]["ritz_max"] <= G["S2_cg_128_10steps"]["gershgorin"]


@pytest.mark.slow
def test_s3_cppcg_512_ritz_min(ora):
    d = inputs.crooked_pipe(512)
    _, st, _ = ora.run(d, steps=1, method=1, eps=1e-15, inner_steps=10)
    g = G["S3_cppcg_s10"]["512"]
    assert abs(st[0]["outer"] - g["outer"]) <= 2
    assert st[0]["ritz_min"] == pytest.approx(g["ritz_min_step1"], abs=0.005)
