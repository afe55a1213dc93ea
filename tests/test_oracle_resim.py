"""Pins of the oracle's target draw, neighbourhood context and resimulation
(PAPER.md 4.2 L967-1043, 4.3 L1064-1102).

The reference values come from 2-D quadrature of the coalescent prior
restricted to the neighbourhood (tests/quadrature.py), which uses neither the
backward messages nor the closed-form transition weights of the oracle.
"""
import math

import numpy as np
import pytest
import scipy.stats

import synth
from tests import quadrature as Q

# SURVEY Appendix B worked example 1 (theta = 0.7): n5=(0,1)@0.1 target,
# n6=(n5,2)@0.3, n7=(3,4)@0.2, n8=(n6,n7)@0.5 root.
EX1_PARENT = np.array([5, 5, 6, 7, 7, 6, 8, 8, -1], np.int32)
EX1_AGE = np.array([0, 0, 0, 0, 0, 0.1, 0.3, 0.2, 0.5])


def _interval0_event_probs(ctx):
    k0 = ctx["k0"]
    om = ctx["omega"][0][k0 - 1]           # omega[k'-1] for k' = 1..3
    w = np.array([om[k0 - 1 - j] if k0 - 1 - j >= 0 else 0.0 for j in range(3)])
    return w / w.sum()                       # P(0, 1, 2 events in interval 0)


def _quad_interval0_event_probs(parent, age, theta, target):
    ctx_tau1 = None
    cs, fixed, t_anc = Q.neighbourhood(parent, age, target)
    a = sorted(float(age[c]) for c in cs)
    cuts = sorted(set(([a[2]] if a[2] > a[1] else []) + [f for f in fixed if a[1] < f < t_anc]))
    ctx_tau1 = cuts[0] if cuts else t_anc
    tot = Q.restricted_prior_integral(parent, age, theta, target)
    probs = []
    for j in range(3):
        f = lambda x, y, pc, j=j: 1.0 if ((x <= ctx_tau1) + (y <= ctx_tau1)) == j else 0.0
        probs.append(Q.restricted_prior_integral(parent, age, theta, target, f) / tot)
    return np.array(probs)


def test_worked_example_1_interval_probabilities(orc):
    ctx = orc.context_info(EX1_PARENT, EX1_AGE, 0.7, 5)
    assert ctx["k0"] == 3 and ctx["m"] == 2 and ctx["rootcase"] is False
    assert list(ctx["l"]) == [2, 1]
    p = _interval0_event_probs(ctx)
    # SURVEY Appendix B (verified there by 2-D quadrature): 0.025391, 0.324185, 0.650424
    assert np.allclose(p, [0.025391, 0.324185, 0.650424], atol=2e-6)
    q = _quad_interval0_event_probs(EX1_PARENT, EX1_AGE, 0.7, 5)
    assert np.allclose(p, q, rtol=1e-7, atol=1e-9)


def _random_trees(n, count, seed):
    rng = np.random.default_rng(seed)
    for _ in range(count):
        parent, age = synth.coalescent_tree(n, 1.0, rng)
        yield parent, age


@pytest.mark.parametrize("n", [4, 5, 6])
def test_context_matches_restricted_prior_quadrature(orc, n):
    """P13: the choice law of the first interval equals the restricted prior."""
    checked = 0
    for parent, age in _random_trees(n, 3, 40 + n):
        for target in range(n, 2 * n - 1):
            if parent[target] < 0:
                continue
            theta = 0.45
            ctx = orc.context_info(parent, age, theta, target)
            p = _interval0_event_probs(ctx)
            q = _quad_interval0_event_probs(parent, age, theta, target)
            assert np.allclose(p, q, rtol=1e-6, atol=1e-8), (target, p, q)
            checked += 1
            if checked >= 6:
                return


def test_context_bookkeeping_counts(orc):
    """l_p = lineages of the pruned tree at tau_p minus active ones (S10, S11)."""
    rng = np.random.default_rng(9)
    n = 9
    parent, age = synth.coalescent_tree(n, 1.0, rng)
    for target in range(n, 2 * n - 1):
        if parent[target] < 0:
            continue
        ctx = orc.context_info(parent, age, 1.0, target)
        par = ctx["Par"]
        tau = ctx["tau"]
        assert np.all(np.diff(tau) > 0)
        for p in range(ctx["m"]):
            t = tau[p]
            total = n - sum(1 for v in range(n, 2 * n - 1) if v not in (target, par) and age[v] <= t)
            act = sum(1 for c in ctx["children"] if age[c] <= t)
            assert ctx["l"][p] == total - act
        if ctx["rootcase"]:
            assert ctx["l"][-1] == 0 and math.isinf(tau[-1])


def test_n3_proposals_follow_the_prior(orc):
    """P12: for n = 3 the proposal is an independent draw from the coalescent
    prior: T3 ~ Exp(6/theta), T2 ~ Exp(2/theta), topology uniform over 3."""
    parent = np.array([3, 3, 4, 4, -1], np.int32)
    age = np.array([0, 0, 0, 0.2, 0.9])
    theta = 0.8
    t1, t2, pairs = [], [], []
    for slot in range(1, 4001):
        _, _, t12, pair, _ = orc.propose(parent, age, theta, 3, 77, 5, slot)
        t1.append(t12[0])
        t2.append(t12[1] - t12[0])
        pairs.append(pair)
    assert scipy.stats.kstest(t1, scipy.stats.expon(scale=theta / 6).cdf).pvalue > 1e-3
    assert scipy.stats.kstest(t2, scipy.stats.expon(scale=theta / 2).cdf).pvalue > 1e-3
    counts = np.bincount(pairs, minlength=3)
    assert scipy.stats.chisquare(counts).pvalue > 1e-3


def test_proposal_marginals_match_quadrature(orc):
    """P13 beyond the first interval: E[x], E[y] and pair probabilities."""
    parent, age = EX1_PARENT, EX1_AGE
    theta, target = 0.7, 5
    tot = Q.restricted_prior_integral(parent, age, theta, target)
    ex = Q.restricted_prior_integral(parent, age, theta, target, lambda x, y, p: x) / tot
    ey = Q.restricted_prior_integral(parent, age, theta, target, lambda x, y, p: y) / tot
    pp = [Q.restricted_prior_integral(parent, age, theta, target,
                                      lambda x, y, p, c=c: float(p == c)) / tot for c in range(3)]
    xs, ys, pairs = [], [], []
    for slot in range(1, 6001):
        _, _, t12, pair, _ = orc.propose(parent, age, theta, target, 123, 0, slot)
        xs.append(t12[0])
        ys.append(t12[1])
        pairs.append(pair)
    xs, ys = np.array(xs), np.array(ys)
    assert abs(xs.mean() - ex) < 4.5 * xs.std() / math.sqrt(len(xs))
    assert abs(ys.mean() - ey) < 4.5 * ys.std() / math.sqrt(len(ys))
    freq = np.bincount(pairs, minlength=3) / len(pairs)
    for c in range(3):
        assert abs(freq[c] - pp[c]) < 4.5 * math.sqrt(pp[c] * (1 - pp[c]) / len(pairs))
    assert np.all(ys <= 0.5) and np.all(xs <= ys)


def test_proposal_tree_is_valid_and_local(orc):
    rng = np.random.default_rng(21)
    n = 12
    parent, age = synth.coalescent_tree(n, 1.0, rng)
    for step in range(40):
        target = orc.pick_target(parent, 99, step)
        new_parent, new_age, t12, pair, _ = orc.propose(parent, age, 0.3, target, 99, step, 1)
        assert orc.check_tree(new_parent, new_age) == 0
        changed = set(np.nonzero(new_parent != parent)[0]) | set(np.nonzero(new_age != age)[0])
        ctx = orc.context_info(parent, age, 0.3, target)
        assert changed <= {target, ctx["Par"], *ctx["children"]}
        assert new_age[target] == t12[0] and new_age[ctx["Par"]] == t12[1]
        parent, age = new_parent, new_age


def test_target_uniform_over_nonroot_interior(orc):
    rng = np.random.default_rng(4)
    n = 8
    parent, age = synth.coalescent_tree(n, 1.0, rng)
    root = int(np.where(parent < 0)[0][0])
    tg = [orc.pick_target(parent, 2024, s) for s in range(12000)]
    assert root not in tg and min(tg) >= n
    counts = np.bincount(tg, minlength=2 * n - 1)[n:]
    counts = np.delete(counts, root - n)
    assert len(counts) == n - 2
    assert scipy.stats.chisquare(counts).pvalue > 1e-3


def test_S_identity_and_prior_closed_form(orc):
    """P10: S = sum_k k(k-1) T_k = 2 sum_i (n-i) h_i; Eq. 18 closed form."""
    rng = np.random.default_rng(8)
    for n in [3, 5, 17]:
        parent, age = synth.coalescent_tree(n, 0.6, rng)
        h = np.sort(age[n:])
        S2 = 2.0 * sum((n - i) * h[i - 1] for i in range(1, n))
        S = orc.coalescent_S(age, n)
        assert np.isclose(S, S2, rtol=1e-13)
        assert np.isclose(orc.log_prior(age, n, 0.6), (n - 1) * np.log(2 / 0.6) - S / 0.6)
    # n = 3 by hand: T3 = 0.2, T2 = 0.5 -> S = 6*0.2 + 2*0.5
    assert np.isclose(orc.coalescent_S(np.array([0, 0, 0, 0.2, 0.7]), 3), 2.2)
