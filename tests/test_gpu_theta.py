"""theta MLE on the GPU (Eq. 25-26, Alg. 2,
5.2.3 L1417-1436) against the oracle on PRESCRIBED sample sets loaded with
mpcgs_load_samples: S20's bimodal relative likelihood (the global mode flips
with theta0), a two-cluster set with interior modes, a coarse GPU grid, and
Table 2's largest sample count M = 1e6.  Tolerance: theta-hat 1e-6 relative
(north star), ln L(theta) 1e-10."""
import time

import numpy as np
import pytest

import synth

pytestmark = pytest.mark.gpu


@pytest.fixture(scope="module")
def P():
    import torch

    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    import paper_conf_ipps_davistzw17_b200 as pkg

    pkg.lib()
    return pkg


def _ctx(P, n, M):
    codes = synth.random_alignment(n, 12, np.random.default_rng(n))
    return P.Context(synth.to_strings(codes), 1.0, max_proposals=4, max_samples=M)


@pytest.mark.parametrize("theta0", [2.1, 2.14, 2.145, 2.15, 2.16, 2.2])
@pytest.mark.parametrize("G", [256, 16])
def test_bimodal_global_mode(P, orc, theta0, G):
    """S20: S = {1, 100}, n = 11: ln L has maxima near theta = 0.1 and theta = 10 whose
    heights cross near theta0 = 2.145; theta-hat must be the global one."""
    S = np.array([1.0, 100.0])
    ctx = _ctx(P, 11, 16)
    ctx.mpcgs_load_samples(S, theta0)
    th = ctx.mpcgs_estimate_theta(G)
    want = orc.theta_hat(S, 11, theta0)
    assert abs(th - want) <= 1e-6 * want, (th, want)
    assert (want < 1.0) == (theta0 >= 2.15)
    for t in (0.1, 1.0, 10.0, th):
        assert abs(ctx.mpcgs_log_rel_likelihood(t) - orc.log_rel_likelihood(S, 11, theta0, t)) <= 1e-10


@pytest.mark.parametrize("theta0", [0.5, 1.0, 3.0])
def test_two_cluster_interior_modes(P, orc, theta0):
    rng = np.random.default_rng(int(theta0 * 10))
    n = 8
    S = np.concatenate([rng.gamma(n - 1, 0.1, 300), rng.gamma(n - 1, 2.0, 300)])
    ctx = _ctx(P, n, 1000)
    ctx.mpcgs_load_samples(S, theta0)
    th, gt, gl = ctx.mpcgs_estimate_theta(256, curve=True)
    want = orc.theta_hat(S, n, theta0)
    assert abs(th - want) <= 1e-6 * want, (th, want)
    # the grid curve is Eq. 25 at the grid points
    for k in (0, 77, 255):
        assert abs(gl[k] - orc.log_rel_likelihood(S, n, theta0, gt[k])) <= 1e-9 * max(1.0, abs(gl[k]))
    # stationarity (Appendix B): theta-hat = S_w(theta-hat) / (n-1)
    assert abs(orc.weighted_mean_S(S, theta0, th) / (n - 1) / th - 1) <= 1e-9


def test_theta_hat_one_million_samples(P, orc):
    """Table 2's largest M (L1544-1551): 1e6 samples, theta-hat vs the oracle; the device
    time of mpcgs_estimate_theta is printed (a7 is a small part of a run, L1558-1559)."""
    M, n, theta0 = 1_000_000, 24, 0.01
    rng = np.random.default_rng(11)
    S = rng.gamma(n - 1, 0.012, M) * np.exp(rng.normal(0, 0.2, M))
    ctx = _ctx(P, n, M)
    ctx.mpcgs_load_samples(S, theta0)
    ctx.mpcgs_estimate_theta(256)  # warm
    t0 = time.perf_counter()
    th = ctx.mpcgs_estimate_theta(256)
    dt = time.perf_counter() - t0
    want = orc.theta_hat(S, n, theta0, G=256)
    assert abs(th - want) <= 1e-6 * want, (th, want)
    for t in (0.5 * th, th, 2 * th):
        assert abs(ctx.mpcgs_log_rel_likelihood(t) - orc.log_rel_likelihood(S, n, theta0, t)) <= 1e-9 * max(
            1.0, abs(orc.log_rel_likelihood(S, n, theta0, t)))
    print(f"theta-hat over M = 1e6 samples: {dt * 1e3:.2f} ms (host wall, grid 256 + Newton)")


def test_load_samples_errors_and_degenerate(P):
    ctx = _ctx(P, 5, 8)
    with pytest.raises(P.MpcgsError):
        ctx.mpcgs_load_samples(np.ones(9), 1.0)          # above capacity
    with pytest.raises(P.MpcgsError):
        ctx.mpcgs_load_samples(np.array([1.0, -2.0]), 1.0)
    with pytest.raises(P.MpcgsError):
        ctx.mpcgs_load_samples(np.array([1.0]), 0.0)
    ctx.mpcgs_load_samples(np.array([3.2, 3.2, 3.2]), 0.7)   # all S equal: theta-hat = S/(n-1)
    assert ctx.mpcgs_estimate_theta(64) == pytest.approx(0.8, rel=1e-15)
    g = ctx.mpcgs_get_samples()
    assert np.all(g["step"] == -1) and np.all(g["slot"] == -1)
