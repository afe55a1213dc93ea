"""P10: the coalescent prior of the oracle, ``orc_log_prior``
(Eq. 17-18, reading S8: a specific pair coalesces at rate 2/theta,
so a labelled history with times has density (2/theta)^{n-1} e^{-S_G/theta}),
pinned by what the mathematics fixes rather than by restating the formula:

* it is a probability density: summed over all labelled histories and
  integrated over the coalescence times by adaptive quadrature it gives 1
  (n = 3: 3 histories; n = 4: 18 ranked labelled histories);
* its interval moments are Kingman's, E[T_k] = theta / (k(k-1));
* it depends on the genealogy only through the times (every labelled history
  of the same ages has the same density), and E[S_G] = (n-1) theta.

The integrand is exp(orc_log_prior(tree)) evaluated on explicitly built trees;
nothing below uses the closed form."""
import itertools

import numpy as np
import pytest
import scipy.integrate


def _history_tree(n, merges, ages):
    """Tree arrays of a labelled history: merges[i] = (a, b) lineage ids joined by the
    i-th coalescence at ages[i]; the new node gets id n + i."""
    parent = np.full(2 * n - 1, -1, np.int32)
    age = np.zeros(2 * n - 1)
    for i, ((a, b), t) in enumerate(zip(merges, ages)):
        parent[a] = parent[b] = n + i
        age[n + i] = t
    return parent, age


def _histories(n):
    """All ranked labelled histories of n tips (n!(n-1)!/2^{n-1} of them)."""
    out = []

    def rec(active, merges, nxt):
        if len(active) == 1:
            out.append(list(merges))
            return
        for a, b in itertools.combinations(active, 2):
            rest = [x for x in active if x not in (a, b)] + [nxt]
            rec(rest, merges + [(a, b)], nxt + 1)

    rec(list(range(n)), [], n)
    return out


def _density(orc, n, merges, ages, theta):
    _, age = _history_tree(n, merges, ages)
    return np.exp(orc.log_prior(age, n, theta))


@pytest.mark.parametrize("theta", [0.3, 1.7])
def test_prior_n3_integrates_to_one_and_interval_means(orc, theta):
    hs = _histories(3)
    assert len(hs) == 3
    opts = dict(epsabs=1e-12, epsrel=1e-10)
    total = m3 = m2 = 0.0
    for merges in hs:
        # T3 = h1 (3 lineages), T2 = h2 - h1 (2 lineages), both on (0, inf)
        f = lambda t2, t3: _density(orc, 3, merges, [t3, t3 + t2], theta)
        total += scipy.integrate.dblquad(f, 0, np.inf, 0, np.inf, **opts)[0]
        m3 += scipy.integrate.dblquad(lambda t2, t3: t3 * f(t2, t3), 0, np.inf, 0, np.inf, **opts)[0]
        m2 += scipy.integrate.dblquad(lambda t2, t3: t2 * f(t2, t3), 0, np.inf, 0, np.inf, **opts)[0]
    assert abs(total - 1.0) <= 1e-8
    assert abs(m3 - theta / 6.0) <= 1e-8 * theta      # E[T_3] = theta / (3*2)
    assert abs(m2 - theta / 2.0) <= 1e-8 * theta      # E[T_2] = theta / (2*1)


def test_prior_n4_integrates_to_one(orc):
    theta = 0.8
    hs = _histories(4)
    assert len(hs) == 18
    # label independence: every history has the same density at the same times
    rng = np.random.default_rng(1)
    for _ in range(5):
        ages = np.cumsum(rng.exponential(0.5, 3))
        d = [_density(orc, 4, m, ages, theta) for m in hs]
        assert np.allclose(d, d[0], rtol=1e-14)
    f = lambda t2, t3, t4: _density(orc, 4, hs[0], [t4, t4 + t3, t4 + t3 + t2], theta)
    one = scipy.integrate.nquad(f, [[0, np.inf]] * 3, opts=dict(epsabs=1e-11, epsrel=1e-8))[0]
    assert abs(18 * one - 1.0) <= 1e-6
    # E[T_4] = theta / 12 from the same density
    g = lambda t2, t3, t4: t4 * f(t2, t3, t4)
    m4 = scipy.integrate.nquad(g, [[0, np.inf]] * 3, opts=dict(epsabs=1e-11, epsrel=1e-8))[0]
    assert abs(18 * m4 - theta / 12.0) <= 1e-6 * theta


def test_prior_mean_S_by_importance_sampling(orc):
    """E[S_G] = (n-1) theta under the prior (P10), estimated by self-normalised
    importance sampling with the oracle's density as the target (proposal:
    independent exponential intervals of mean 1, n = 5)."""
    n, theta = 5, 0.6
    rng = np.random.default_rng(3)
    merges = _histories(n)[7]
    K = 60000
    T = rng.exponential(1.0, size=(K, n - 1))         # T_n, T_{n-1}, ..., T_2
    logq = -T.sum(axis=1)
    logp = np.empty(K)
    S = np.empty(K)
    for i in range(K):
        ages = np.cumsum(T[i])
        _, age = _history_tree(n, merges, ages)
        logp[i] = orc.log_prior(age, n, theta)
        S[i] = orc.coalescent_S(age, n)
    w = np.exp(logp - logq - np.max(logp - logq))
    est = np.sum(w * S) / np.sum(w)
    assert abs(est / ((n - 1) * theta) - 1.0) <= 0.03
