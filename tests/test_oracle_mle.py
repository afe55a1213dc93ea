"""Pins of the oracle's relative likelihood and MLE (PAPER.md
Eq. 25-26, 5.1.5 L1306-1311, Alg. 2) and of its UPGMA G0
(5.1.3 L1287-1295).
"""
import numpy as np

import synth


def test_rel_likelihood_is_one_at_theta0(orc):
    S = np.array([0.3, 1.2, 2.5])
    assert abs(orc.log_rel_likelihood(S, 7, 0.4, 0.4)) < 1e-15


def test_single_sample_closed_form(orc):
    for S, n in [(3.7, 5), (0.01, 12), (250.0, 64)]:
        assert np.isclose(orc.theta_hat(np.array([S]), n, 0.01), S / (n - 1), rtol=1e-15)
        assert np.isclose(orc.theta_hat(np.full(50, S), n, 1.3), S / (n - 1), rtol=1e-15)


def test_bracket_stationarity_and_em_monotone(orc):
    rng = np.random.default_rng(12)
    for n, theta0 in [(12, 0.01), (24, 0.5), (5, 2.0)]:
        S = rng.gamma(n - 1, 0.8, size=300) * rng.uniform(0.5, 2.0)
        th = orc.theta_hat(S, n, theta0)
        assert S.min() / (n - 1) <= th <= S.max() / (n - 1)
        # stationary point of ln L: theta = S_w(theta) / (n-1)
        assert np.isclose(orc.em_map(S, n, theta0, th), th, rtol=1e-10)
        # it is the maximum on a dense independent scan
        grid = np.exp(np.linspace(np.log(S.min() / (n - 1)), np.log(S.max() / (n - 1)), 20001))
        ll = np.array([orc.log_rel_likelihood(S, n, theta0, t) for t in grid[::50]])
        assert orc.log_rel_likelihood(S, n, theta0, th) >= ll.max() - 1e-12
        # EM never decreases ln L (Appendix B)
        for t in grid[::2000]:
            assert orc.log_rel_likelihood(S, n, theta0, orc.em_map(S, n, theta0, t)) >= \
                orc.log_rel_likelihood(S, n, theta0, t) - 1e-12
        # the paper's local gradient ascent (Alg. 2, literal) agrees when theta0 is
        # near the mode; started 200x away it drifts off (why S20 uses a bracket)
        if theta0 > 0.1:
            assert np.isclose(orc.theta_alg2(S, n, theta0), th, rtol=3e-3)


def test_bimodal_curve_global_mode(orc):
    """S20: S = {1, 100}, n = 11, theta0 near 2.15 has two local maxima of
    nearly equal height; the estimate must be the global one."""
    S = np.array([1.0, 100.0])
    n = 11
    for theta0 in [2.1, 2.15, 2.2]:
        grid = np.exp(np.linspace(np.log(0.05), np.log(20.0), 200001))
        # Eq. 25-26 evaluated directly with numpy for the scan
        e = (n - 1) * np.log(theta0 / grid)[:, None] - S[None, :] * (1 / grid - 1 / theta0)[:, None]
        ll = np.logaddexp(e[:, 0], e[:, 1]) - np.log(2)
        g = grid[np.argmax(ll)]
        th = orc.theta_hat(S, n, theta0)
        assert np.isclose(th, g, rtol=1e-3), (theta0, th, g)
        # two separated local maxima exist
        d = np.diff(np.sign(np.diff(ll)))
        assert np.sum(d < 0) == 2


def test_upgma_hand_example(orc):
    # d(0,1)=1, d(2,3)=2, d(0,2)=d(0,3)=d(1,2)=d(1,3)=5 over 6 sites
    codes = np.array([
        [0, 0, 0, 0, 0, 0],
        [1, 0, 0, 0, 0, 0],
        [2, 2, 2, 2, 2, 0],
        [2, 2, 2, 2, 1, 1],
    ], np.uint8)
    theta0 = 0.1
    parent, age = orc.upgma(codes, theta0)
    assert list(parent) == [4, 4, 5, 5, 6, 6, -1]
    # heights theta0 * D / 2 with D = 1, 2, mean(5, 5, 6, 5) ... recomputed by hand
    d01, d23 = 1, 2
    dx = np.mean([np.sum(codes[a] != codes[b]) for a in (0, 1) for b in (2, 3)])
    assert np.allclose(age[4:], [theta0 * d01 / 2, theta0 * d23 / 2, theta0 * dx / 2])


def test_upgma_identical_sequences_strictly_increasing(orc):
    codes = np.zeros((5, 10), np.uint8)
    parent, age = orc.upgma(codes, 0.01)
    assert orc.check_tree(parent, age) == 0
    for v in range(9):
        if parent[v] >= 0:
            assert age[parent[v]] > age[v]


def test_synthetic_workload_shapes():
    for name, (n, L) in {"c1": (4, 100), "c2": (12, 1000)}.items():
        wl = synth.workload(name)
        assert wl["codes"].shape == (n, L)
        assert wl["codes"].dtype == np.uint8 and wl["codes"].max() <= 3


# ------------------------------------------------------------------ multiple loci
def test_loci_one_locus_is_single_locus(orc):
    rng = np.random.default_rng(2)
    S = rng.gamma(3.0, 0.02, 500)
    assert orc.theta_hat_loci([S], [12], [0.01]) == orc.theta_hat(S, 12, 0.01)
    for th in (0.003, 0.01, 0.05):
        assert orc.log_rel_likelihood_loci([S], [12], [0.01], th) == orc.log_rel_likelihood(S, 12, 0.01, th)


def test_loci_degenerate_closed_form(orc):
    """One value of S per locus: ln L = sum_l (n_l-1) ln(theta0_l/theta) - S_l (1/theta - 1/theta0_l),
    maximised at sum_l S_l / sum_l (n_l - 1) (differentiate); the grid + bisection must find it."""
    S_list = [np.full(7, 0.3), np.full(3, 1.1), np.full(5, 0.05)]
    n_list, t0 = [5, 12, 4], [0.01, 0.02, 0.005]
    want = (0.3 + 1.1 + 0.05) / (4 + 11 + 3)
    assert abs(orc.theta_hat_loci(S_list, n_list, t0) - want) <= 1e-13 * want


def test_loci_product_stationarity_and_duplication(orc):
    rng = np.random.default_rng(9)
    S_list = [rng.gamma(4.0, 0.01, 300), rng.gamma(2.0, 0.05, 200)]
    n_list, t0 = [8, 16], [0.01, 0.03]
    th = orc.theta_hat_loci(S_list, n_list, t0)
    # the joint likelihood is the product over loci (independent genealogies, one theta)
    for x in (0.5 * th, th, 2 * th):
        parts = sum(orc.log_rel_likelihood(S, n, a, x) for S, n, a in zip(S_list, n_list, t0))
        assert np.isclose(orc.log_rel_likelihood_loci(S_list, n_list, t0, x), parts, rtol=1e-14)
    # stationarity: sum_l S_w,l(theta-hat) = theta-hat sum_l (n_l - 1)
    sw = sum(orc.weighted_mean_S(S, a, th) for S, a in zip(S_list, t0))
    assert abs(sw - th * sum(n - 1 for n in n_list)) <= 1e-9 * sw
    # bracket, and a duplicated locus set leaves the argmax unchanged
    lo = sum(S.min() for S in S_list) / sum(n - 1 for n in n_list)
    hi = sum(S.max() for S in S_list) / sum(n - 1 for n in n_list)
    assert lo <= th <= hi
    th2 = orc.theta_hat_loci(S_list * 2, n_list * 2, t0 * 2)
    assert abs(th2 - th) <= 1e-9 * th
    # a global maximum on a fine scan
    xs = np.exp(np.linspace(np.log(lo), np.log(hi), 2001))
    ll = [orc.log_rel_likelihood_loci(S_list, n_list, t0, x) for x in xs]
    assert orc.log_rel_likelihood_loci(S_list, n_list, t0, th) >= max(ll) - 1e-12
