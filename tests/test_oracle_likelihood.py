"""Pins of the oracle's model and data likelihood.

Each pin fixes the oracle against something other than itself: known-answer
vectors, the matrix exponential of the F81 rate matrix, brute-force summation
over all ancestral states, closed forms and invariances.
"""
import itertools

import numpy as np
import pytest
import scipy.linalg

import synth


# ------------------------------------------------------------------ P17 RNG
def test_philox_known_answers(orc):
    # Random123 kat_vectors for philox4x32_10 (Salmon et al., SC'11)
    kat = [
        ([0, 0, 0, 0], [0, 0], [0x6627E8D5, 0xE169C58D, 0xBC57AC4C, 0x9B00DBD8]),
        ([0xFFFFFFFF] * 4, [0xFFFFFFFF] * 2, [0x408F276D, 0x41C83B0E, 0xA20BC7C6, 0x6D5451FD]),
        ([0x243F6A88, 0x85A308D3, 0x13198A2E, 0x03707344], [0xA4093822, 0x299F31D0],
         [0xD16CFE09, 0x94FDCCEB, 0x5001E420, 0x24126EA1]),
    ]
    for ctr, key, want in kat:
        assert list(orc.philox(ctr, key)) == want


def test_u01_range_and_resolution(orc):
    lib = orc.lib()
    assert lib.orc_u01(0, 0) == 2.0 ** -53
    assert lib.orc_u01(0xFFFFFFFF, 0xFFFFFFFF) == 1.0
    us = np.array([orc.uniform(7, 3, s, 1, i) for s in range(50) for i in range(40)])
    assert us.min() > 0.0 and us.max() <= 1.0
    assert abs(us.mean() - 0.5) < 0.02


# ------------------------------------------------------------------ P1 F81
def _f81_Q(pi, u):
    Q = u * np.tile(pi, (4, 1))
    np.fill_diagonal(Q, 0.0)
    np.fill_diagonal(Q, -Q.sum(axis=1))
    return Q


@pytest.mark.parametrize("pi", [[0.25] * 4, [0.1, 0.2, 0.3, 0.4], [0.7, 0.1, 0.1, 0.1]])
def test_transition_is_expm_of_f81_generator(orc, pi):
    pi = np.array(pi)
    u = orc.default_rate(pi)
    assert np.isclose(u, 1.0 / (1.0 - np.sum(pi ** 2)))
    Q = _f81_Q(pi, u)
    for t in [0.0, 1e-9, 0.01, 0.3, 2.0, 40.0]:
        P = orc.transition(t, u, pi)
        assert np.allclose(P, scipy.linalg.expm(Q * t), rtol=1e-12, atol=1e-14)
        assert np.allclose(P.sum(axis=1), 1.0, atol=1e-15)
    assert np.array_equal(orc.transition(0.0, u, pi), np.eye(4))
    assert np.allclose(orc.transition(1e6, u, pi), np.tile(pi, (4, 1)), atol=1e-15)
    # Chapman-Kolmogorov
    P1, P2, P12 = (orc.transition(t, u, pi) for t in (0.2, 0.45, 0.65))
    assert np.allclose(P1 @ P2, P12, atol=1e-15)
    # expected substitutions per unit time equal 1 under u = 1/(1 - sum pi^2) (reading S3)
    assert np.isclose(-np.dot(pi, np.diag(Q)), 1.0)


# ------------------------------------------------------------------ P3 brute force
def _brute_force_loglik(codes, parent, age, pi, u):
    """Sum over all 4^(n-1) interior assignments of pi_root * prod_branches P."""
    n = codes.shape[0]
    nn = 2 * n - 1
    root = int(np.where(parent < 0)[0][0])
    Q = _f81_Q(pi, u)
    Pb = {v: scipy.linalg.expm(Q * (age[parent[v]] - age[v])) for v in range(nn) if parent[v] >= 0}
    interior = list(range(n, nn))
    total = np.zeros(codes.shape[1])
    for assign in itertools.product(range(4), repeat=len(interior)):
        state = {v: a for v, a in zip(interior, assign)}
        prob = np.full(codes.shape[1], pi[state[root]])
        for v in range(nn):
            if parent[v] < 0:
                continue
            ps = state[parent[v]]
            if v < n:
                prob = prob * Pb[v][ps, codes[v]]
            else:
                prob = prob * Pb[v][ps, state[v]]
        total += prob
    return np.log(total)


@pytest.mark.parametrize("n", [2, 3, 4, 5])
@pytest.mark.parametrize("shape", ["caterpillar", "balanced", "random"])
def test_pruning_equals_brute_force(orc, n, shape):
    rng = np.random.default_rng(100 + n)
    parent, age = synth.shaped_tree(n, shape, rng, scale=0.3)
    pi = np.array([0.1, 0.2, 0.3, 0.4])
    u = orc.default_rate(pi)
    codes = synth.random_alignment(n, 30, rng, pi)
    ll, site = orc.log_likelihood(codes, parent, age, pi, u, site_ll=True)
    want = _brute_force_loglik(codes, parent, age, pi, u)
    assert np.allclose(site, want, rtol=1e-12, atol=1e-12)
    assert np.isclose(ll, want.sum(), rtol=1e-13)


# ------------------------------------------------------------------ P2 / P4 / P5 / P6 / P7
def test_monomorphic_and_infinite_branches(orc):
    rng = np.random.default_rng(3)
    parent, age = synth.shaped_tree(6, "random", rng)
    codes = np.zeros((6, 25), np.uint8)
    assert orc.log_likelihood(codes, parent, age, np.array([1.0, 0, 0, 0]), 1.0) == 0.0
    # infinite branches: every tip independent draw from pi
    pi = np.array([0.4, 0.3, 0.2, 0.1])
    codes = synth.random_alignment(6, 25, rng, pi)
    far = age * 1e4
    want = np.log(pi[codes]).sum()
    assert np.isclose(orc.log_likelihood(codes, parent, far, pi, orc.default_rate(pi)), want,
                      rtol=1e-12)


def test_two_tip_pulley_closed_form(orc):
    pi = np.array([0.3, 0.2, 0.1, 0.4])
    u = orc.default_rate(pi)
    parent = np.array([2, 2, -1])
    age = np.array([0.0, 0.0, 0.37])
    codes = np.array([[0, 1, 2, 3, 0, 3], [0, 2, 2, 1, 3, 3]], np.uint8)
    P = scipy.linalg.expm(_f81_Q(pi, u) * 0.74)
    want = np.sum(np.log(pi[codes[0]] * P[codes[0], codes[1]]))
    assert np.isclose(orc.log_likelihood(codes, parent, age, pi, u), want, rtol=1e-13)


def test_root_position_invariance(orc):
    # (tip0, (tip1, tip2)v) with the root slid along the root-to-tip0 / root-to-v path
    pi = np.array([0.25, 0.25, 0.3, 0.2])
    u = orc.default_rate(pi)
    rng = np.random.default_rng(5)
    codes = synth.random_alignment(3, 40, rng, pi)
    parent = np.array([4, 3, 3, 4, -1])
    base = orc.log_likelihood(codes, parent, np.array([0.0, 0.0, 0.0, 0.2, 0.5]), pi, u)
    for d in [-0.15, 0.07, 0.3]:
        age = np.array([2 * d, 0.0, 0.0, 0.2, 0.5 + d])
        assert np.isclose(orc.log_likelihood(codes, parent, age, pi, u), base, rtol=1e-12)


def test_site_and_label_permutation_and_duplication(orc):
    rng = np.random.default_rng(11)
    n = 7
    parent, age = synth.coalescent_tree(n, 1.0, rng)
    pi = np.array([0.2, 0.3, 0.3, 0.2])
    u = orc.default_rate(pi)
    codes = synth.f81_alignment(parent, age, 64, pi, u, rng)
    base = orc.log_likelihood(codes, parent, age, pi, u)
    perm = rng.permutation(64)
    assert np.isclose(orc.log_likelihood(codes[:, perm], parent, age, pi, u), base, rtol=1e-13)
    dup = np.concatenate([codes, codes], axis=1)
    assert np.isclose(orc.log_likelihood(dup, parent, age, pi, u), 2 * base, rtol=1e-13)
    # relabel tips: tip i -> sigma(i), rows permuted accordingly
    sigma = rng.permutation(n)
    parent2 = parent.copy()
    for i in range(n):
        parent2[sigma[i]] = parent[i]
    codes2 = np.zeros_like(codes)
    codes2[sigma] = codes
    assert np.isclose(orc.log_likelihood(codes2, parent2, age, pi, u), base, rtol=1e-13)


def test_all_zero_branches(orc):
    n = 5
    parent = np.array([5, 5, 6, 7, 7, 6, 8, 8, -1], np.int32)
    age = np.zeros(9)
    pi = np.array([0.1, 0.2, 0.3, 0.4])
    const = np.tile(np.array([[0, 3, 2, 2, 1]], np.uint8), (n, 1))
    assert np.isclose(orc.log_likelihood(const, parent, age, pi, 1.0), np.log(pi[[0, 3, 2, 2, 1]]).sum())
    mixed = const.copy()
    mixed[2, 1] = 0
    assert orc.log_likelihood(mixed, parent, age, pi, 1.0) == -np.inf


def test_theta_independence_of_data_likelihood(orc):
    """Eq. 23 (L720-723): the likelihood has no theta argument; only u and t enter."""
    rng = np.random.default_rng(2)
    parent, age = synth.coalescent_tree(5, 0.5, rng)
    pi = np.full(4, 0.25)
    codes = synth.f81_alignment(parent, age, 50, pi, 4 / 3, rng)
    a = orc.log_likelihood(codes, parent, age, pi, 4 / 3)
    b = orc.log_likelihood(codes, parent, age * 2, pi, 4 / 6)   # (u, t) -> (u/2, 2t)
    assert np.isclose(a, b, rtol=1e-13)


def test_base_freqs_pooled(orc):
    codes = np.array([[0, 0, 1, 2], [3, 3, 3, 0]], np.uint8)
    assert np.allclose(orc.base_freqs(codes), [3 / 8, 1 / 8, 1 / 8, 3 / 8])


# ------------------------------------------------------------------ f4: F84 / HKY85
def _model_Q(model, kappa, pi):
    """Rate matrix from the model's definition, normalised to mean rate 1."""
    grp = [0, 1, 0, 1]                       # A, C, G, T: purines 0, pyrimidines 1
    Pi = [pi[0] + pi[2], pi[1] + pi[3]]
    Q = np.zeros((4, 4))
    for i in range(4):
        for j in range(4):
            if i == j:
                continue
            same = grp[i] == grp[j]
            if model == "F84":
                Q[i, j] = pi[j] * (1 + (kappa / Pi[grp[j]] if same else 0.0))
            else:  # HKY85
                Q[i, j] = (kappa if same else 1.0) * pi[j]
    np.fill_diagonal(Q, -Q.sum(axis=1))
    return Q / -np.dot(pi, np.diag(Q))


@pytest.mark.parametrize("model", ["F84", "HKY85"])
@pytest.mark.parametrize("kappa", [0.5, 2.0, 7.3])
def test_model_transition_is_expm(orc, model, kappa):
    pi = np.array([0.35, 0.15, 0.2, 0.3])
    Q = _model_Q(model, kappa, pi)
    for t in [0.0, 1e-6, 0.05, 0.7, 3.0]:
        P = orc.transition_model(model, kappa, t, pi)
        assert np.allclose(P, scipy.linalg.expm(Q * t), rtol=1e-11, atol=1e-13)
    # reductions to F81: F84 with kappa = 0, HKY85 with kappa = 1
    u = orc.default_rate(pi)
    assert np.allclose(orc.transition_model("F84", 0.0, 0.4, pi), orc.transition(0.4, u, pi), atol=1e-15)
    assert np.allclose(orc.transition_model("HKY85", 1.0, 0.4, pi), orc.transition(0.4, u, pi), atol=1e-15)


@pytest.mark.parametrize("model", ["F84", "HKY85"])
def test_model_pruning_equals_brute_force(orc, model):
    rng = np.random.default_rng(77)
    n, kappa = 4, 3.0
    parent, age = synth.shaped_tree(n, "random", rng, scale=0.3)
    pi = np.array([0.3, 0.2, 0.15, 0.35])
    codes = synth.random_alignment(n, 25, rng, pi)
    Q = _model_Q(model, kappa, pi)
    nn = 2 * n - 1
    root = int(np.where(parent < 0)[0][0])
    Pb = {v: scipy.linalg.expm(Q * (age[parent[v]] - age[v])) for v in range(nn) if parent[v] >= 0}
    interior = list(range(n, nn))
    total = np.zeros(codes.shape[1])
    for assign in itertools.product(range(4), repeat=len(interior)):
        st = dict(zip(interior, assign))
        prob = np.full(codes.shape[1], pi[st[root]])
        for v in range(nn):
            if parent[v] >= 0:
                prob = prob * (Pb[v][st[parent[v]], codes[v]] if v < n else Pb[v][st[parent[v]], st[v]])
        total += prob
    assert np.isclose(orc.log_likelihood_model(model, kappa, codes, parent, age, pi), np.log(total).sum(),
                      rtol=1e-12)


# ------------------------------------------------------------------ ambiguity codes (f4, reading S24)
def _set_of(code):
    return [code] if code < 4 else [x for x in range(4) if ((code - 16) >> x) & 1]


@pytest.mark.parametrize("model", ["F81", "HKY85"])
def test_ambiguity_pruning_equals_brute_force(orc, model):
    """An ambiguous tip's likelihood is the sum over the bases it stands for:
    brute force over interior assignments AND tip resolutions."""
    rng = np.random.default_rng(91)
    n, kappa = 4, 2.5
    parent, age = synth.shaped_tree(n, "random", rng, scale=0.3)
    pi = np.array([0.3, 0.2, 0.15, 0.35])
    u = orc.default_rate(pi)
    codes = synth.ambiguate(synth.random_alignment(n, 20, rng, pi), 0.3, rng, gap_frac=0.1)
    assert (codes >= 16).any() and (codes == 31).any()
    Q = _f81_Q(pi, u) if model == "F81" else _model_Q(model, kappa, pi)
    nn = 2 * n - 1
    root = int(np.where(parent < 0)[0][0])
    Pb = {v: scipy.linalg.expm(Q * (age[parent[v]] - age[v])) for v in range(nn) if parent[v] >= 0}
    interior = list(range(n, nn))
    want = np.zeros(codes.shape[1])
    for s in range(codes.shape[1]):
        tot = 0.0
        for assign in itertools.product(range(4), repeat=len(interior)):
            st = dict(zip(interior, assign))
            prob = pi[st[root]]
            for v in range(nn):
                if parent[v] < 0:
                    continue
                if v < n:
                    prob *= sum(Pb[v][st[parent[v]], x] for x in _set_of(int(codes[v, s])))
                else:
                    prob *= Pb[v][st[parent[v]], st[v]]
            tot += prob
        want[s] = np.log(tot)
    if model == "F81":
        got = orc.log_likelihood(codes, parent, age, pi, u)
    else:
        got = orc.log_likelihood_model(model, kappa, codes, parent, age, pi)
    assert np.isclose(got, want.sum(), rtol=1e-12)


def test_ambiguity_special_cases(orc):
    rng = np.random.default_rng(5)
    n = 6
    parent, age = synth.coalescent_tree(n, 0.5, rng)
    pi = np.array([0.1, 0.2, 0.3, 0.4])
    u = orc.default_rate(pi)
    codes = synth.random_alignment(n, 12, rng, pi)
    # an all-N column has site likelihood exactly 1
    c2 = codes.copy()
    c2[:, 3] = 31
    _, site = orc.log_likelihood(c2, parent, age, pi, u, site_ll=True)
    assert site[3] == 0.0 or abs(site[3]) < 1e-15
    # a one-base "set" is that base
    c3 = codes.copy()
    c3[2, :] = 16 + (1 << codes[2, :])
    assert orc.log_likelihood(c3, parent, age, pi, u) == orc.log_likelihood(codes, parent, age, pi, u)
    # R at a tip = A there + G there (linearity of Eq. 19 in a tip vector)
    cA, cG, cR = codes.copy(), codes.copy(), codes.copy()
    cA[1, 5], cG[1, 5], cR[1, 5] = 0, 2, 16 + 5
    sA = orc.log_likelihood(cA, parent, age, pi, u, site_ll=True)[1][5]
    sG = orc.log_likelihood(cG, parent, age, pi, u, site_ll=True)[1][5]
    sR = orc.log_likelihood(cR, parent, age, pi, u, site_ll=True)[1][5]
    assert np.isclose(np.exp(sR), np.exp(sA) + np.exp(sG), rtol=1e-13)
    # base frequencies ignore ambiguous characters; UPGMA: N differs from nothing
    amb = synth.ambiguate(codes, 0.5, rng)
    known = amb[amb < 4]
    assert np.allclose(orc.base_freqs(amb), np.bincount(known, minlength=4) / known.size)
    two = np.array([[0, 1, 2, 3], [31, 31, 31, 31], [0, 1, 2, 0]], np.uint8)
    p, a = orc.upgma(two, 1.0)
    assert a[p[1]] <= 1e-6 + 1e-12  # row 1 joins first (distance 0 to everything)
