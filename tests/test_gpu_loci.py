"""GPU parity of multiple loci sharing theta through the C ABI:
concurrent sampling of several loci (one context each) and the joint theta-hat
(product of Eq. 25 over loci) against the oracle's orc_theta_hat_loci."""
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


def _loci(P, shapes, theta0=0.01, **kw):
    ctxs = []
    for k, (n, L) in enumerate(shapes):
        rng = np.random.default_rng(500 + k)
        p, a = synth.coalescent_tree(n, 1.0, rng)
        codes = synth.f81_alignment(p, a, L, np.full(4, 0.25), 4.0 / 3.0, rng)
        ctxs.append(P.Context(synth.to_strings(codes), theta0, burnin_steps=20, max_proposals=32,
                              max_samples=4096, **kw))
    return ctxs


SHAPES = [(4, 100), (6, 200), (8, 150)]


def test_sample_loci_equals_sequential_sampling(P):
    a, b = _loci(P, SHAPES), _loci(P, SHAPES)
    seeds = [11, 22, 33]
    P.mpcgs_sample_loci(a, 16, 1000, seeds)
    for c, sd in zip(b, seeds):
        c.mpcgs_sample(16, 1000, sd)
    for x, y in zip(a, b):
        sx, sy = x.mpcgs_get_samples(), y.mpcgs_get_samples()
        for k in sx:
            assert np.array_equal(sx[k], sy[k]), k


def test_joint_theta_hat_matches_oracle(P, orc):
    ctxs = _loci(P, SHAPES)
    P.mpcgs_sample_loci(ctxs, 16, 2000, [5, 6, 7])
    S_list = [c.mpcgs_get_samples()["S"] for c in ctxs]
    n_list = [n for n, _ in SHAPES]
    got, gt, gl = P.mpcgs_estimate_theta_loci(ctxs, 256, curve=True)
    want = orc.theta_hat_loci(S_list, n_list, [0.01] * 3)
    assert abs(got - want) <= 1e-6 * want
    # the summed curve is the product of the per-locus relative likelihoods
    for g in (0, 100, 255):
        ref = orc.log_rel_likelihood_loci(S_list, n_list, [0.01] * 3, gt[g])
        assert abs(gl[g] - ref) <= 1e-9 * max(1.0, abs(ref))
    # one locus through the multi-locus entry point is the single-locus estimate
    assert P.mpcgs_estimate_theta_loci(ctxs[:1]) == ctxs[0].mpcgs_estimate_theta()


def test_em_loci_matches_manual_loop(P):
    a, b = _loci(P, SHAPES), _loci(P, SHAPES)
    seeds = np.array([3, 4, 5], np.uint64)
    trace = P.mpcgs_em_loci(a, 3, 16, 1000, seeds)
    manual = []
    for it in range(3):
        P.mpcgs_sample_loci(b, 16, 1000, seeds + it)
        th = P.mpcgs_estimate_theta_loci(b)
        manual.append(th)
        for c in b:
            c.mpcgs_set_theta0(th)
    assert np.array_equal(trace, np.array(manual))
    assert np.all(trace > 0)


def test_loci_errors(P):
    ctxs = _loci(P, SHAPES[:2])
    with pytest.raises(P.MpcgsError):
        P.mpcgs_estimate_theta_loci(ctxs)  # no samples yet
    with pytest.raises(P.MpcgsError):
        P.mpcgs_estimate_theta_loci([])
    with pytest.raises(P.MpcgsError):
        P.mpcgs_sample_loci(ctxs, 64, 100, [1, 2])  # N above max_proposals
