"""Pins of the oracle's GMH step and chain (
PAPER.md Alg. 1, Eq. 29-31, Fig. 12).
"""
import math

import numpy as np
import scipy.stats

import synth
from tests import quadrature as Q


def test_inverse_cdf_draw_matches_softmax(orc):
    """P14: stratified uniforms reproduce softmax(logL) to 1/M."""
    logL = np.array([-1203.5, -1201.0, -1204.2, -1200.7, -1210.0])
    w, cum = orc.weights(logL)
    p = np.exp(logL - logL.max())
    p /= p.sum()
    M = 20000
    counts = np.zeros(len(logL))
    for i in range(M):
        counts[orc.draw(cum, (i + 0.5) / M)[0]] += 1
    assert np.allclose(counts / M, p, atol=2.0 / M)
    # N = 1: the move probability is Barker's L1/(L0+L1) (SURVEY P14 note on L925-927)
    w2, cum2 = orc.weights(np.array([-10.0, -10.0 + math.log(3.0)]))
    assert np.isclose(1 - cum2[0] / cum2[1], 0.75)


def test_lowest_index_tie_break(orc):
    w, cum = orc.weights(np.array([0.0, -np.inf, 0.0]))
    assert orc.draw(cum, 0.5)[0] == 0     # x = C_0 exactly -> lowest index
    assert orc.draw(cum, 0.5000001)[0] == 2   # zero-weight slot 1 never chosen


def test_prior_not_in_weights_zero_data_draws_uniform(orc):
    """P15 / S18: with no data every logL is 0, so draws are uniform over the
    N+1 states whatever their coalescent priors (S) are."""
    n, N = 6, 7
    rng = np.random.default_rng(1)
    parent, age = synth.coalescent_tree(n, 1.0, rng)
    codes = np.zeros((n, 0), np.uint8)
    counts = np.zeros(N + 1)
    spread = []
    for step in range(400):
        tr = orc.gmh_step(codes, np.full(4, 0.25), 4 / 3, 0.5, N, N, 5, step, parent, age, 0.0)
        for d in tr["draws"]:
            counts[d] += 1
        spread.append(np.ptp(tr["S"]))
        parent, age = tr["parent"], tr["age"]
    assert np.mean(spread) > 0.1
    assert scipy.stats.chisquare(counts).pvalue > 1e-3


def _topology_n4(parent):
    kids = Q.children(parent)
    root = int(np.where(parent < 0)[0][0])
    a, b = kids[root]
    if a >= 4 and b >= 4:
        cher = sorted(tuple(sorted(kids[a])) + tuple(sorted(kids[b])))
        pair = tuple(sorted(kids[a]))
        return ("bal", min(pair, tuple(sorted(kids[b]))))
    inner = a if a >= 4 else b
    k2 = kids[inner]
    inner2 = [c for c in k2 if c >= 4][0]
    return ("cat", tuple(sorted(kids[inner2])), [c for c in k2 if c < 4][0])


def test_zero_data_chain_samples_the_prior(orc):
    """P11: the no-data chain samples the coalescent prior at theta0: E[T_k] =
    theta0/(k(k-1)); ranked labelled histories of n = 4 are uniform, so each
    balanced labelled topology has mass 1/9 and each caterpillar 1/18."""
    n, N, theta0 = 4, 8, 0.6
    parent = np.array([4, 4, 5, 5, 6, 6, -1], np.int32)
    age = np.array([0, 0, 0, 0, 0.1, 0.2, 0.5])
    codes = np.zeros((n, 0), np.uint8)
    topo, Tk = {}, []
    steps = 24000
    for step in range(steps):
        tr = orc.gmh_step(codes, np.full(4, 0.25), 4 / 3, theta0, N, 1, 31, step, parent, age, 0.0)
        parent, age = tr["parent"], tr["age"]
        if step < 200:
            continue
        key = _topology_n4(parent)
        topo[key] = topo.get(key, 0) + 1
        h = np.sort(age[n:])
        Tk.append([h[0], h[1] - h[0], h[2] - h[1]])   # T4, T3, T2
    tot = sum(topo.values())
    bal = [v / tot for k, v in topo.items() if k[0] == "bal"]
    cat = [v / tot for k, v in topo.items() if k[0] == "cat"]
    assert len(bal) == 3 and len(cat) == 12
    assert np.allclose(bal, 1 / 9, atol=0.02)
    assert np.allclose(cat, 1 / 18, atol=0.015)
    Tk = np.array(Tk)
    want = [theta0 / 12, theta0 / 6, theta0 / 2]
    assert np.allclose(Tk.mean(axis=0), want, rtol=0.06)


def test_n3_chain_matches_exact_posterior(orc):
    """P16: n = 3 with data; topology frequencies and E[T3], E[T2] against the
    exact posterior computed by 2-D quadrature over (T3, T2) per topology."""
    theta0 = 0.5
    pi = np.full(4, 0.25)
    u = 4 / 3
    # columns: support for (0,1), (0,2), (1,2), plus constant sites
    codes = np.array([[0, 0, 1, 2, 2, 3], [0, 1, 0, 2, 2, 3], [1, 0, 0, 2, 2, 1]], np.uint8)

    def post(f):
        tot = 0.0
        for pair in range(3):
            def inner(x):
                g = lambda y: f(x, y, pair) * Q.three_tip_likelihood(codes, x, y, pair, pi, u) * \
                    math.exp(-(4 * x + 2 * y) / theta0)
                return Q.piecewise_quad(g, x, math.inf, [], 1e-7)
            tot += Q.piecewise_quad(inner, 0.0, math.inf, [], 1e-6)
        return tot

    Z = post(lambda x, y, p: 1.0)
    p_top = np.array([post(lambda x, y, p, c=c: float(p == c)) / Z for c in range(3)])
    e_t3 = post(lambda x, y, p: x) / Z
    e_t2 = post(lambda x, y, p: y - x) / Z
    assert p_top.min() > 0.05

    parent = np.array([3, 3, 4, 4, -1], np.int32)
    age = np.array([0, 0, 0, 0.1, 0.4])
    gl = orc.log_likelihood(codes, parent, age, pi, u)
    N = 8
    tops, t3, t2 = [], [], []
    for step in range(4000):
        tr = orc.gmh_step(codes, pi, u, theta0, N, N, 17, step, parent, age, gl)
        if step >= 50:
            gen_pair = {(0, 1): 0, (0, 2): 1, (1, 2): 2}[tuple(sorted(np.nonzero(parent == 3)[0]))]
            for d in tr["draws"]:
                pr = gen_pair if d == 0 else tr["pair"][d]
                tops.append(pr)
                t3.append(tr["t12"][d][0] if d else age[3])
                t2.append((tr["t12"][d][1] - tr["t12"][d][0]) if d else age[4] - age[3])
        parent, age, gl = tr["parent"], tr["age"], tr["gen_logL"]
    freq = np.bincount(tops, minlength=3) / len(tops)
    assert np.allclose(freq, p_top, atol=0.02), (freq, p_top)
    assert abs(np.mean(t3) - e_t3) < 0.04 * e_t3
    assert abs(np.mean(t2) - e_t2) < 0.04 * e_t2


def test_chain_bookkeeping(orc):
    """Burn-in draws are not stored (L497-498); sampling stores min(N, remaining) per set."""
    wl = synth.workload("c1")
    pi = orc.base_freqs(wl["codes"])
    u = orc.default_rate(pi)
    parent, age = orc.upgma(wl["codes"], wl["theta0"])
    res = orc.run_chain(wl["codes"], pi, u, wl["theta0"], 16, 5, 40, 9, parent, age)
    assert list(res["step"][:16]) == [5] * 16
    assert list(res["step"][16:32]) == [6] * 16
    assert list(res["step"][32:]) == [7] * 8
    assert np.all((res["slot"] >= 0) & (res["slot"] <= 16))


def test_gmh_step_model_reduces_to_f81(orc):
    """f4: F84 with kappa = 0 and HKY85 with kappa = 1 are F81, so the
    model step must reproduce the F81 step: same target, trees, weights and draws."""
    wl = synth.workload("c1")
    codes = wl["codes"]
    pi = orc.base_freqs(codes)
    u = orc.default_rate(pi)
    parent, age = orc.upgma(codes, wl["theta0"])
    gl = orc.log_likelihood(codes, parent, age, pi, u)
    ref = orc.gmh_step(codes, pi, u, wl["theta0"], 8, 8, 11, 3, parent, age, gl)
    for model, kappa in (("F84", 0.0), ("HKY85", 1.0)):
        got = orc.gmh_step(codes, pi, 0.0, wl["theta0"], 8, 8, 11, 3, parent, age, gl, model=model, kappa=kappa)
        assert got["target"] == ref["target"]
        assert np.array_equal(got["t12"], ref["t12"]) and np.array_equal(got["pair"], ref["pair"])
        assert np.allclose(got["logL"], ref["logL"], rtol=1e-12, atol=0)
        assert np.array_equal(got["draws"], ref["draws"])
    # a real transition bias changes the likelihoods but not the proposals (Alg. 1)
    got = orc.gmh_step(codes, pi, 0.0, wl["theta0"], 8, 8, 11, 3, parent, age, gl, model="HKY85", kappa=8.0)
    assert np.array_equal(got["t12"], ref["t12"])
    assert np.all(np.abs(got["logL"][1:] - ref["logL"][1:]) > 1e-6)
