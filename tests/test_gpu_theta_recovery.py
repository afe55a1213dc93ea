"""theta recovery (the shape of Table 1, without
LAMARC): data simulated under the coalescent + F81 (synth/), the EM loop of
Fig. 11 (L1208-1225) driven from theta0 = 0.01 (Fig. 5's driving value,
L786-788).  With 10 kbp alignments the posterior concentrates on the true
genealogy, so theta-hat must approach the single-tree MLE S(G_true)/(n-1).

Reading P19: no estimator from ONE locus can beat the
single-true-tree MLE, S(G_true)/(n-1) ~ theta * Gamma(n-1, 1)/(n-1), whose
coefficient of variation is 1/sqrt(n-1) = 0.30 at n = 12.  For theta_true in
{0.5, 1, 2} that caps the expected Pearson r(theta_true, theta-hat) at ~0.84
(the paper's own Table 1 gives r(true, mpcgs) = 0.86 over its five points), so
the single-locus test asks theta-hat to track that MLE and to correlate as well
as it does; SURVEY's r >= 0.9 is asserted where it is reachable: four loci
sharing theta, CV 1/sqrt(4(n-1)) = 0.15, expected r ~ 0.95.
These bars were fixed before the runs that check them, from the CV alone."""
import numpy as np
import pytest

import synth

pytestmark = pytest.mark.gpu

THETAS = (0.5, 1.0, 2.0)
N_SEQ, L_SITES = 12, 10000


@pytest.fixture(scope="module")
def P():
    import torch

    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    import paper_conf_ipps_davistzw17_b200 as pkg

    pkg.lib()
    return pkg


def _dataset(theta, rep, locus=0):
    n, L = N_SEQ, L_SITES
    rng = np.random.default_rng(9000 + 100 * rep + int(10 * theta) + 7919 * locus)
    p, a = synth.coalescent_tree(n, theta, rng)
    codes = synth.f81_alignment(p, a, L, np.full(4, 0.25), 4 / 3, rng)
    h = np.sort(a[n:])
    s_true = 2.0 * sum((n - i) * h[i - 1] for i in range(1, n))  # S(G_true) (Eq. 18's statistic)
    return codes, s_true


def _ctx(P, codes):
    return P.Context(synth.to_strings(codes), 0.01, burnin_steps=300, max_proposals=64, max_samples=20000)


def test_em_recovers_theta_single_locus(P):
    R = 8
    truth, est, single = [], [], []
    for theta in THETAS:
        for rep in range(R):
            codes, s_true = _dataset(theta, rep)
            ctx = _ctx(P, codes)
            trace = ctx.mpcgs_em(8, 64, 20000, 31 + rep)
            truth.append(theta)
            est.append(trace[-1])
            single.append(s_true / (N_SEQ - 1))
            assert abs(trace[-1] - trace[-3]) <= 0.10 * trace[-1]  # the EM re-drive has settled
    est, single, truth = map(np.array, (est, single, truth))
    rel = np.abs(est / single - 1.0)
    assert np.all(rel <= 0.20) and np.median(rel) <= 0.05, np.c_[truth, single, est]
    r_est, r_single = np.corrcoef(truth, est)[0, 1], np.corrcoef(truth, single)[0, 1]
    assert r_est >= max(0.7, r_single - 0.05), (r_est, r_single)
    ratio = est / truth
    assert 0.8 <= ratio.mean() <= 1.25, ratio.mean()


def test_em_recovers_theta_four_loci(P):
    """Four independent loci share theta (joint EM, mpcgs_em_loci): r >= 0.9 (P19)."""
    R, K = 7, 4
    truth, est, single = [], [], []
    for theta in THETAS:
        for rep in range(R):
            data = [_dataset(theta, rep, locus=1 + k) for k in range(K)]
            ctxs = [_ctx(P, codes) for codes, _ in data]
            trace = P.mpcgs_em_loci(ctxs, 8, 64, 20000, [31 + rep + 101 * k for k in range(K)])
            truth.append(theta)
            est.append(trace[-1])
            single.append(sum(s for _, s in data) / (K * (N_SEQ - 1)))  # joint single-true-tree MLE
            for c in ctxs:
                c.free()
    est, single, truth = map(np.array, (est, single, truth))
    rel = np.abs(est / single - 1.0)
    assert np.all(rel <= 0.15) and np.median(rel) <= 0.05, np.c_[truth, single, est]
    r_est = np.corrcoef(truth, est)[0, 1]
    assert r_est >= 0.9, (r_est, np.corrcoef(truth, single)[0, 1])
    ratio = est / truth
    assert 0.8 <= ratio.mean() <= 1.25, ratio.mean()
