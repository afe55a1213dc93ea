"""Distributional pins of the production GPU loop (mpcgs_sample), the GPU-side
counterparts of the oracle's P11 / P16 tests:

* P11 -- with data that carry no information (a monomorphic alignment, pi_A = 1,
  so P(D|G) = 1 for every genealogy: Eq. 20 with P_AA(t) = 1) the chain samples
  the coalescent prior at theta0 (Eq. 17-18): S_G = sum k(k-1) T_k is then
  Gamma(n - 1, theta0) (each k(k-1) T_k ~ Exp(mean theta0)).
* P16 -- n = 3 with data: E[S] and E[S^2] of the samples match the exact posterior
  (2-D quadrature over (T3, T2) for the three topologies; tests/quadrature.py).

Moment tolerances: 4 standard errors from 50 batch means (the chain's samples are
autocorrelated), or 1-2 % of the exact value, whichever is larger."""
import math

import numpy as np
import pytest
import scipy.stats

from tests import quadrature as Q

pytestmark = pytest.mark.gpu


@pytest.fixture(scope="module")
def P():
    import torch

    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    import paper_conf_ipps_davistzw17_b200 as pkg

    pkg.lib()
    return pkg


def _batch_means_se(x, nb=50):
    b = np.array_split(np.asarray(x), nb)
    m = np.array([v.mean() for v in b])
    return m.std(ddof=1) / math.sqrt(nb)


@pytest.mark.parametrize("n,theta0,precision", [(4, 0.6, 64), (7, 0.2, 64), (5, 1.3, 32)])
def test_uninformative_data_chain_samples_the_prior(P, n, theta0, precision):
    rows = ["A" * 50] * n
    # a caterpillar start: node n joins tips 0, 1; node n+i joins node n+i-1 and tip i+1
    parent = np.full(2 * n - 1, -1, np.int32)
    age = np.zeros(2 * n - 1)
    parent[0] = parent[1] = n
    for i in range(1, n - 1):
        parent[n + i - 1] = n + i
        parent[i + 1] = n + i
    age[n:] = 0.1 * np.arange(1, n)
    N, M, B = 16, 320_000, 200
    ctx = P.Context(rows, theta0, init_tree=(parent, age), burnin_steps=B, max_proposals=N, max_samples=M,
                    precision=precision)
    pi, u = ctx.mpcgs_get_model()
    assert pi[0] == 1.0 and u == 1.0  # S3: sum pi^2 = 1 -> u = 1
    ctx.mpcgs_sample(N, M, 11)
    smp = ctx.mpcgs_get_samples()
    assert np.all(np.abs(smp["logL"]) <= 1e-12)  # every genealogy has likelihood 1 (up to e + em rounding)
    S = smp["S"]
    mean, var = S.mean(), S.var()
    se = _batch_means_se(S)
    assert abs(mean - (n - 1) * theta0) <= max(4 * se, 0.01 * (n - 1) * theta0), (mean, (n - 1) * theta0, se)
    dev2 = (S - mean) ** 2
    assert abs(var - (n - 1) * theta0 ** 2) <= max(4 * _batch_means_se(dev2), 0.02 * (n - 1) * theta0 ** 2), (
        var, (n - 1) * theta0 ** 2, _batch_means_se(dev2))
    # shape: one sample per step (the last draw) against Gamma(n-1, theta0)
    last = S[N - 1::N]
    ks = scipy.stats.kstest(last, scipy.stats.gamma(n - 1, scale=theta0).cdf)
    assert ks.pvalue > 1e-4, ks


def test_n3_chain_matches_exact_posterior_moments(P):
    theta0, pi, u = 0.5, np.full(4, 0.25), 4 / 3
    codes = np.array([[0, 0, 1, 2, 2, 3], [0, 1, 0, 2, 2, 3], [1, 0, 0, 2, 2, 1]], np.uint8)

    def post(f):
        tot = 0.0
        for pair in range(3):
            def inner(x):
                g = lambda y: f(x, y) * Q.three_tip_likelihood(codes, x, y, pair, pi, u) * \
                    math.exp(-(4 * x + 2 * y) / theta0)
                return Q.piecewise_quad(g, x, math.inf, [], 1e-7)
            tot += Q.piecewise_quad(inner, 0.0, math.inf, [], 1e-6)
        return tot

    Z = post(lambda x, y: 1.0)
    # S = 3*2*T3 + 2*1*T2 with T3 = x, T2 = y - x
    e_s = post(lambda x, y: 6 * x + 2 * (y - x)) / Z
    e_s2 = post(lambda x, y: (6 * x + 2 * (y - x)) ** 2) / Z
    rows = ["".join("ACGT"[c] for c in r) for r in codes]
    parent = np.array([3, 3, 4, 4, -1], np.int32)
    age = np.array([0, 0, 0, 0.1, 0.4])
    N, M = 8, 400_000
    ctx = P.Context(rows, theta0, init_tree=(parent, age), burnin_steps=100, max_proposals=N, max_samples=M,
                    base_freq=pi, mu=u)
    ctx.mpcgs_sample(N, M, 23)
    S = ctx.mpcgs_get_samples()["S"]
    se = _batch_means_se(S)
    assert abs(S.mean() - e_s) <= max(4 * se, 0.01 * e_s), (S.mean(), e_s, se)
    assert abs((S ** 2).mean() - e_s2) <= max(4 * _batch_means_se(S ** 2), 0.01 * e_s2), ((S ** 2).mean(), e_s2)
