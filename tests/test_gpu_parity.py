"""GPU parity of the CUDA path against the oracle, through the C ABI
(BASELINE.json north_star tolerances):

* per-genealogy ln P(D|G): 1e-9 relative (FP64 partials), 1e-4 (FP32);
* target, interval choices/pair codes and draw indices bit-exact (draws flagged
  near a threshold by the oracle are skipped), event times 1e-12 relative to
  the tree height, S_G 1e-12;
* theta-hat 1e-6 relative.
"""
import numpy as np
import pytest

import synth

pytestmark = pytest.mark.gpu

LL_TOL = {64: 1e-9, 32: 1e-4}


@pytest.fixture(scope="module")
def P():
    import torch

    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    import paper_conf_ipps_davistzw17_b200 as pkg

    pkg.lib()
    return pkg


def _ctx(P, codes, theta0, tree=None, **kw):
    return P.Context(synth.to_strings(codes), theta0, init_tree=tree, **kw)


# ------------------------------------------------------------------ pruning
@pytest.mark.parametrize("precision", [64, 32])
@pytest.mark.parametrize("n,L", [(3, 1), (4, 100), (12, 1000), (24, 129), (64, 1000), (128, 257), (256, 2000)])
def test_score_trees_matches_oracle(P, orc, precision, n, L):
    rng = np.random.default_rng(7 * n + L)
    pi = np.array([0.22, 0.28, 0.31, 0.19])
    u = orc.default_rate(pi)
    true_p, true_a = synth.coalescent_tree(n, 0.05, rng)
    codes = synth.f81_alignment(true_p, true_a, L, pi, u, rng)
    trees = [synth.coalescent_tree(n, th, rng) for th in (0.01, 0.05, 0.3)]
    trees += [synth.shaped_tree(n, s, rng, scale=0.02) for s in ("caterpillar", "balanced")]
    ctx = _ctx(P, codes, 0.05, tree=trees[0], precision=precision, base_freq=pi, mu=u, max_proposals=8,
               max_samples=16)
    got = ctx.mpcgs_score_trees(np.stack([t[0] for t in trees]), np.stack([t[1] for t in trees]))
    for (p, a), g in zip(trees, got):
        want = orc.log_likelihood(codes, p, a, pi, u)
        assert abs(g - want) <= LL_TOL[precision] * abs(want), (g, want)


@pytest.mark.parametrize("model,kappa", [("F84", 2.0), ("HKY85", 6.0), ("F84", 0.0)])
@pytest.mark.parametrize("precision", [64, 32])
@pytest.mark.parametrize("n,L", [(3, 1), (12, 1000), (24, 129), (64, 1000), (256, 2000)])
def test_score_trees_general_model(P, orc, model, kappa, precision, n, L):
    """pruning under F84 / HKY85 (per-op P matrices from the
    eigen-system, flat kernel) against the oracle's closed-form likelihood."""
    rng = np.random.default_rng(11 * n + L)
    pi = np.array([0.22, 0.28, 0.31, 0.19])
    true_p, true_a = synth.coalescent_tree(n, 0.05, rng)
    codes = synth.f81_alignment(true_p, true_a, L, pi, orc.default_rate(pi), rng)
    trees = [synth.coalescent_tree(n, th, rng) for th in (0.01, 0.05, 0.3, 3.0)]
    trees += [synth.shaped_tree(n, s, rng, scale=0.02) for s in ("caterpillar", "balanced")]
    ctx = _ctx(P, codes, 0.05, tree=trees[0], precision=precision, base_freq=pi, max_proposals=8,
               max_samples=16, model=model, kappa=kappa)
    got = ctx.mpcgs_score_trees(np.stack([t[0] for t in trees]), np.stack([t[1] for t in trees]))
    for (p, a), g in zip(trees, got):
        want = orc.log_likelihood_model(model, kappa, codes, p, a, pi)
        assert abs(g - want) <= LL_TOL[precision] * abs(want), (g, want)


@pytest.mark.parametrize("model,kappa,name,N,steps", [("F84", 2.0, "c1", 16, 25), ("HKY85", 4.0, "c2", 32, 8),
                                                      ("F84", 5.0, "c3", 64, 3)])
def test_lockstep_general_model(P, orc, model, kappa, name, N, steps):
    wl = synth.workload(name, L=400) if name != "c1" else synth.workload(name)
    assert _lockstep(P, orc, wl, N, steps, wl["chain_seed"], model=model, kappa=kappa) <= max(2, steps // 4)


def test_lockstep_general_model_compressed_fp32(P, orc):
    wl = synth.workload("c1")
    _lockstep(P, orc, wl, 16, 10, wl["chain_seed"], precision=32, compress=True, model="HKY85", kappa=3.0)


@pytest.mark.parametrize("model,kappa", [("F81", 0.0), ("HKY85", 4.0)])
@pytest.mark.parametrize("precision", [64, 32])
@pytest.mark.parametrize("n,L", [(3, 7), (12, 1000), (64, 300), (256, 500)])
def test_score_trees_ambiguity_codes(P, orc, model, kappa, precision, n, L):
    """SURVEY 8(f) f4 / reading S24: IUPAC ambiguity codes and gaps as base-set
    indicator tips (flat kernel with mask codes) against the oracle."""
    rng = np.random.default_rng(13 * n + L)
    pi = np.array([0.22, 0.28, 0.31, 0.19])
    true_p, true_a = synth.coalescent_tree(n, 0.05, rng)
    codes = synth.ambiguate(synth.f81_alignment(true_p, true_a, L, pi, orc.default_rate(pi), rng), 0.15, rng,
                            gap_frac=0.1)
    trees = [synth.coalescent_tree(n, th, rng) for th in (0.01, 0.3)]
    trees += [synth.shaped_tree(n, s, rng, scale=0.02) for s in ("caterpillar", "balanced")]
    u = orc.default_rate(pi)
    ctx = _ctx(P, codes, 0.05, tree=trees[0], precision=precision, base_freq=pi, mu=u, max_proposals=8,
               max_samples=16, model=model, kappa=kappa, ambiguity=True)
    got = ctx.mpcgs_score_trees(np.stack([t[0] for t in trees]), np.stack([t[1] for t in trees]))
    for (p, a), g in zip(trees, got):
        if model == "F81":
            want = orc.log_likelihood(codes, p, a, pi, u)
        else:
            want = orc.log_likelihood_model(model, kappa, codes, p, a, pi)
        assert abs(g - want) <= LL_TOL[precision] * abs(want), (g, want)


@pytest.mark.parametrize("incremental,compress,model", [(False, False, "F81"), (True, False, "F81"),
                                                        (False, True, "F81"), (False, False, "F84")])
def test_lockstep_ambiguity_codes(P, orc, incremental, compress, model):
    wl = dict(synth.workload("c2", L=300))
    wl["codes"] = synth.ambiguate(wl["codes"], 0.1, np.random.default_rng(4), gap_frac=0.05)
    assert _lockstep(P, orc, wl, 32, 8, wl["chain_seed"], incremental=incremental, compress=compress,
                     model=model, kappa=2.0 if model != "F81" else 0.0, ambiguity=True) <= 2


def test_ambiguity_off_rejects_iupac(P):
    with pytest.raises(P.MpcgsError):
        P.Context(["ACGT", "ACGN", "ACGA"], 0.1, max_proposals=4, max_samples=4)
    ctx = P.Context(["ACGT", "ACGN", "AC-A"], 0.1, max_proposals=4, max_samples=4, ambiguity=True)
    ctx.free()


def test_general_model_argument_errors(P):
    rows = ["ACGT", "ACGA", "ACGG"]
    with pytest.raises(P.MpcgsError):
        P.Context(rows, 0.1, model="F84", kappa=2.0, incremental=True, max_proposals=4, max_samples=4)
    with pytest.raises(P.MpcgsError):
        P.Context(["AAGG", "AAGG", "GGAA"], 0.1, model="HKY85", kappa=2.0, max_proposals=4, max_samples=4)
    with pytest.raises(P.MpcgsError):
        P.Context(rows, 0.1, model=5, max_proposals=4, max_samples=4)


def test_score_adversarial_branch_lengths(P, orc):
    rng = np.random.default_rng(3)
    n, L = 16, 300
    pi = np.array([0.1, 0.4, 0.4, 0.1])
    u = orc.default_rate(pi)
    codes = synth.random_alignment(n, L, rng, pi)
    trees = []
    for scale in (1e-9, 1e3, 0.0):
        p, a = synth.shaped_tree(n, "random", rng, scale=1.0)
        a = a * scale if scale > 0 else np.zeros_like(a)
        trees.append((p, a))
    p, a = synth.shaped_tree(n, "caterpillar", rng)
    a[n:] = np.arange(1, n) * 1e-9          # tiny steps
    trees.append((p, a))
    ctx = _ctx(P, codes, 0.05, tree=trees[1], base_freq=pi, mu=u, max_proposals=8, max_samples=16)
    got = ctx.mpcgs_score_trees(np.stack([t[0] for t in trees]), np.stack([t[1] for t in trees]))
    for (p, a), g in zip(trees, got):
        want = orc.log_likelihood(codes, p, a, pi, u)
        if np.isinf(want):
            assert g == want
        else:
            assert abs(g - want) <= 1e-9 * abs(want)


@pytest.mark.parametrize("n,precision", [(16, 64), (64, 64), (16, 32), (64, 32)])
def test_unit_branch_form_budget(P, orc, n, precision):
    """Table kernel, unit-diagonal branches (DESIGN 5, k_prune_tab item 7): every
    branch is applied divided by its e = exp(-u t), so vectors grow by up to
    exp(u * tree length); the form is used while that stays below 2^(900 - n) and
    the tree falls back to the standard branch above (FP32 keeps the standard form;
    its cases score long trees at the FP32 form's 2^(120 - n) scale).  Trees whose u * length sits
    just below and just above the budget (and far above it) must all match the
    oracle, as must short-branch trees (unit form, tiny C)."""
    rng = np.random.default_rng(17 + n)
    L = 16400  # the unit form is used on alignments of >= 16384 sites (MPCGS_UNIT_MIN_L)
    pi = np.array([0.2, 0.3, 0.3, 0.2])
    u = orc.default_rate(pi)
    codes = synth.random_alignment(n, L, rng, pi)
    budget_nats = ((900 if precision == 64 else 120) - n) * np.log(2.0)
    trees = []
    for frac in (0.97, 1.03, 3.0, 1e-3):
        p, a = synth.shaped_tree(n, "random", rng, scale=1.0)
        length = sum(a[p[v]] - a[v] for v in range(2 * n - 2))
        trees.append((p, a * (frac * budget_nats / (u * length))))
    ctx = _ctx(P, codes, 0.05, tree=trees[3], base_freq=pi, mu=u, max_proposals=len(trees), max_samples=16,
               precision=precision)
    got = ctx.mpcgs_score_trees(np.stack([t[0] for t in trees]), np.stack([t[1] for t in trees]))
    for k, ((p, a), g) in enumerate(zip(trees, got)):
        want = orc.log_likelihood(codes, p, a, pi, u)
        assert np.isfinite(g) and abs(g - want) <= LL_TOL[precision] * abs(want), (k, g, want)


def test_underflow_rescaling_long_alignment_many_tips(P, orc):
    """P8: n = 256 tips with long branches forces per-node rescaling in both
    precisions; sampled sites are checked one by one via L = 64 prefixes."""
    rng = np.random.default_rng(5)
    n, L = 256, 64
    pi = np.array([0.05, 0.45, 0.45, 0.05])
    u = orc.default_rate(pi)
    p, a = synth.coalescent_tree(n, 5.0, rng)
    codes = synth.random_alignment(n, L, rng, pi)
    want = orc.log_likelihood(codes, p, a, pi, u)
    assert want < -700 * 1.0  # per-site likelihoods far below FP32 range
    for prec in (64, 32):
        ctx = _ctx(P, codes, 0.05, tree=(p, a), base_freq=pi, mu=u, precision=prec, max_proposals=2,
                   max_samples=4)
        g = ctx.mpcgs_score_trees(p[None], a[None])[0]
        assert abs(g - want) <= LL_TOL[prec] * abs(want)


@pytest.mark.parametrize("precision", [64, 32])
@pytest.mark.parametrize("n", [24, 64, 128])
def test_table_kernel_triplets_and_sparse_checks(P, orc, precision, n):
    """Table kernel (n <= 128): fused cherry+tip triplet tables and the FP64
    sparse underflow checks placed by integer bounds (S5).  Trees mix long
    branches (values fall far below 2^-256 within a subtree, so checks must fire),
    tiny branches with mismatching tips (the bound's em factor), zero-length
    branches (no bound: every node checked) and caterpillars (a triplet at the
    bottom, then a chain of TS ops); L spans several site batches and a ragged tail."""
    rng = np.random.default_rng(100 + n)
    L = 1100
    pi = np.array([0.07, 0.43, 0.38, 0.12])
    u = orc.default_rate(pi)
    codes = synth.random_alignment(n, L, rng, pi)
    trees = [synth.coalescent_tree(n, th, rng) for th in (8.0, 0.3, 1e-4)]
    for shape in ("caterpillar", "random", "balanced"):
        p, a = synth.shaped_tree(n, shape, rng, scale=1.0)
        trees.append((p, a * 3.0))
    p, a = synth.shaped_tree(n, "random", rng, scale=1.0)
    a[n:] = np.cumsum(np.where(np.arange(n - 1) % 3 == 0, 1e-7, rng.exponential(2.0, n - 1)))  # tiny and long steps
    trees.append((p, a))
    p, a = synth.shaped_tree(n, "caterpillar", rng, scale=1.0)
    a[n:n + 3] = 0.0  # zero-length branches near the tips
    trees.append((p, a))
    ctx = _ctx(P, codes, 0.05, tree=trees[1], precision=precision, base_freq=pi, mu=u, max_proposals=len(trees),
               max_samples=16)
    got = ctx.mpcgs_score_trees(np.stack([t[0] for t in trees]), np.stack([t[1] for t in trees]))
    for k, ((p, a), g) in enumerate(zip(trees, got)):
        want = orc.log_likelihood(codes, p, a, pi, u)
        if np.isinf(want):
            assert g == want, k
        else:
            assert abs(g - want) <= LL_TOL[precision] * abs(want), (k, g, want)


# ------------------------------------------------------------------ GMH step (lock-step, P20)
def _lockstep(P, orc, wl, N, steps, seed, K=None, precision=64, incremental=False, compress=False,
              model="F81", kappa=0.0, ambiguity=False):
    codes = wl["codes"]
    pi = orc.base_freqs(codes)
    u = orc.default_rate(pi)
    theta0 = wl["theta0"]
    parent, age = orc.upgma(codes, theta0)
    if model == "F81":
        gl = orc.log_likelihood(codes, parent, age, pi, u)
    else:
        gl = orc.log_likelihood_model(model, kappa, codes, parent, age, pi)
    ctx = _ctx(P, codes, theta0, tree=(parent, age), precision=precision, max_proposals=N, max_samples=16,
               incremental=incremental, compress_patterns=compress, model=model, kappa=kappa,
               ambiguity=ambiguity)
    K = N if K is None else K
    height = age.max()
    skipped = 0
    for s in range(steps):
        ctx.mpcgs_set_state(parent, age)
        gp, ga, g_ll, g_S = ctx.mpcgs_get_state()
        assert abs(g_ll - gl) <= LL_TOL[precision] * abs(gl)
        tr = ctx.mpcgs_step_trace(s, N, K, seed)
        ref = orc.gmh_step(codes, pi, u, theta0, N, K, seed, s, parent, age, gl, model=model, kappa=kappa)
        assert tr["target"] == ref["target"]
        ok = ~ref["slot_flag"]
        ok[0] = True
        assert np.array_equal(tr["pair"][1:][ok[1:]], ref["pair"][1:][ok[1:]])
        scale = max(height, ref["t12"].max())
        assert np.allclose(tr["t12"][ok], ref["t12"][ok], rtol=0, atol=1e-12 * scale)
        assert np.allclose(tr["S"][ok], ref["S"][ok], rtol=1e-12, atol=0)
        assert np.all(np.abs(tr["logL"][ok] - ref["logL"][ok]) <= LL_TOL[precision] * np.abs(ref["logL"][ok]))
        if precision == 64 and not ref["draw_flag"].any() and ok.all():
            assert np.array_equal(tr["draws"], ref["draws"])
            # the generator the GPU committed (k_draw: last draw's slot, Fig. 12) is the oracle's
            gp, ga, g_ll2, g_S2 = ctx.mpcgs_get_state()
            assert np.array_equal(gp, ref["parent"])
            assert np.allclose(ga, ref["age"], rtol=0, atol=1e-12 * max(height, ref["age"].max()))
            assert abs(g_ll2 - ref["gen_logL"]) <= LL_TOL[precision] * abs(ref["gen_logL"])
            assert abs(g_S2 - ref["S"][ref["draws"][-1]]) <= 1e-12 * abs(g_S2)
        else:
            skipped += 1
        parent, age, gl = ref["parent"], ref["age"], ref["gen_logL"]
        height = age.max()
    return skipped


def test_lockstep_c1(P, orc):
    wl = synth.workload("c1")
    assert _lockstep(P, orc, wl, 16, 40, wl["chain_seed"]) <= 2


def test_lockstep_c2_shape(P, orc):
    wl = synth.workload("c2", L=300)
    assert _lockstep(P, orc, wl, 64, 12, wl["chain_seed"]) <= 1


def test_lockstep_n24_ragged(P, orc):
    wl = synth.workload("c3", L=257, N=48)
    assert _lockstep(P, orc, wl, 48, 6, 77) <= 1


@pytest.mark.parametrize("name,over,N,steps", [("c1", {}, 16, 30), ("c2", {"L": 300}, 64, 10),
                                               ("c3", {"L": 257, "N": 48}, 48, 6), ("c4", {"n": 128, "L": 300}, 32, 4)])
def test_lockstep_incremental_rescoring(P, orc, name, over, N, steps):
    """incremental rescoring gives the oracle's (full-pruning)
    likelihoods to 1e-9 and the same draws."""
    wl = synth.workload(name, **over)
    assert _lockstep(P, orc, wl, N, steps, wl["chain_seed"], incremental=True) <= 1


@pytest.mark.parametrize("incremental", [False, True])
@pytest.mark.parametrize("theta_true", [1.0, 0.01])
def test_lockstep_pattern_compression(P, orc, incremental, theta_true):
    """scoring distinct columns weighted by their counts gives
    the uncompressed oracle likelihoods (site independence, L714-716)."""
    wl = synth.workload("c2", L=600, theta_true=theta_true)
    ctx = _ctx(P, wl["codes"], wl["theta0"], compress_patterns=True, max_proposals=64, max_samples=16)
    n_pat = ctx.mpcgs_num_patterns()
    assert n_pat == np.unique(wl["codes"].T, axis=0).shape[0] < 600
    assert _lockstep(P, orc, wl, 64, 6, wl["chain_seed"], incremental=incremental, compress=True) <= 1


def test_incremental_chain_matches_full_pruning(P):
    """Free-running: the incremental context keeps its stored partials in step
    with the generator over many commits (same chain as full pruning)."""
    wl = synth.workload("c2", L=400)
    rows = synth.to_strings(wl["codes"])
    tree = (wl["true_parent"], wl["true_age"])
    out = []
    for inc in (False, True):
        c = P.Context(rows, wl["theta0"], init_tree=tree, max_proposals=64, max_samples=6400, burnin_steps=20,
                      incremental=inc)
        c.mpcgs_sample(64, 6400, 3)
        out.append(c.mpcgs_get_samples())
        _, _, gl, _ = c.mpcgs_get_state()
        # the stored partials still describe the generator: rescoring it from scratch agrees
        p, a, _, _ = c.mpcgs_get_state()
        assert abs(c.mpcgs_score_trees(p[None], a[None])[0] - gl) <= 1e-9 * abs(gl)
    full, inc = out
    same = np.cumprod(full["slot"] == inc["slot"]).sum()
    assert same >= 2000, same   # identical until a near-threshold draw (if any)
    assert np.allclose(full["logL"][:same], inc["logL"][:same], rtol=1e-10, atol=0)


def test_lockstep_fp32_loglik_only(P, orc):
    wl = synth.workload("c1")
    _lockstep(P, orc, wl, 16, 10, 5, precision=32)


def test_root_case_and_n3(P, orc):
    rng = np.random.default_rng(0)
    wl = dict(codes=synth.random_alignment(3, 40, rng), theta0=0.2)
    assert _lockstep(P, orc, wl, 8, 20, 9) <= 1


# The free-running loop (mpcgs_sample, mpcgs_em) on moving chains: tests/test_gpu_chain.py

# ------------------------------------------------------------------ theta MLE
def test_theta_hat_matches_oracle(P, orc):
    wl = synth.workload("c2", L=400)
    codes = wl["codes"]
    N, M = 64, 3000
    ctx = _ctx(P, codes, wl["theta0"], burnin_steps=20, max_proposals=N, max_samples=M)
    ctx.mpcgs_sample(N, M, 123)
    S = ctx.mpcgs_get_samples()["S"]
    th = ctx.mpcgs_estimate_theta(256)
    want = orc.theta_hat(S, 12, wl["theta0"])
    assert abs(th - want) <= 1e-6 * want
    for t in (0.5 * th, th, 2 * th):
        assert np.isclose(ctx.mpcgs_log_rel_likelihood(t), orc.log_rel_likelihood(S, 12, wl["theta0"], t),
                          rtol=1e-10, atol=1e-10)


def test_theta_hat_degenerate_single_value(P, orc):
    wl = synth.workload("c1")
    ctx = _ctx(P, wl["codes"], wl["theta0"], max_proposals=16, max_samples=16)
    ctx.mpcgs_sample(16, 1, 3)
    S = ctx.mpcgs_get_samples()["S"]
    assert np.isclose(ctx.mpcgs_estimate_theta(64), S[0] / 3, rtol=1e-15)


# ------------------------------------------------------------------ errors
def test_argument_errors(P):
    wl = synth.workload("c1")
    rows = synth.to_strings(wl["codes"])
    with pytest.raises(P.MpcgsError):
        P.Context(rows[:2], 0.01)
    with pytest.raises(P.MpcgsError):
        P.Context(rows, -1.0)
    bad = list(rows)
    bad[1] = bad[1][:5] + "N" + bad[1][6:]
    with pytest.raises(P.MpcgsError) as ei:
        P.Context(bad, 0.01)
    assert ei.value.status == -2
    ctx = P.Context(rows, 0.01, max_proposals=16, max_samples=100)
    with pytest.raises(P.MpcgsError):
        ctx.mpcgs_estimate_theta()        # before sample -> E_STATE
    with pytest.raises(P.MpcgsError):
        ctx.mpcgs_sample(32, 10, 1)       # N above capacity
    with pytest.raises(P.MpcgsError):
        ctx.mpcgs_sample(16, 1000, 1)     # M above capacity


def test_init_newick_equals_arrays(P, orc):
    """SURVEY 8(b) init_newick: a context started from a Newick G0 holds the same
    generator (and its likelihood) as one started from the parsed arrays."""
    wl = synth.workload("c2", L=300)
    codes, p, a = wl["codes"], wl["true_parent"], wl["true_age"]
    n = len(codes)
    kids = {v: [] for v in range(2 * n - 1)}
    for v in range(2 * n - 1):
        if p[v] >= 0:
            kids[int(p[v])].append(v)

    def rec(v):
        return str(v) if v < n else "(" + ",".join(f"{rec(c)}:{float(a[v] - a[c])!r}" for c in kids[v]) + ")"

    nw = rec(int(np.where(p < 0)[0][0])) + ";"
    c1 = _ctx(P, codes, wl["theta0"], init_newick=nw, max_proposals=8, max_samples=8)
    g1 = c1.mpcgs_get_state()
    assert np.array_equal(g1[0], p) and np.allclose(g1[1], a, rtol=1e-13)
    pi = orc.base_freqs(codes)
    want = orc.log_likelihood(codes, p, a, pi, orc.default_rate(pi))
    assert abs(g1[2] - want) <= 1e-9 * abs(want)
    with pytest.raises(P.MpcgsError) as ei:
        _ctx(P, codes, wl["theta0"], init_newick="((0:1,1:1):1,2:2);", max_proposals=8, max_samples=8)
    assert ei.value.status == -1 and "init_newick" in str(ei.value)


def test_all_weights_non_finite_is_numeric_error(P):
    """S6 / MPCGS_E_NUMERIC: a user pi with pi_T = 0 on data containing T makes every
    genealogy's likelihood 0 (the root sum weights state T by pi_T), so all N + 1 weights
    are non-finite: mpcgs_sample reports MPCGS_E_NUMERIC instead of drawing."""
    rows = ["ACGTACGTAC", "ACGAACGTAC", "ACGTACGAAC", "TCGAACGTAC"]
    ctx = P.Context(rows, 0.1, base_freq=[0.4, 0.3, 0.3, 0.0], mu=1.0, max_proposals=8, max_samples=16)
    _, _, gl, _ = ctx.mpcgs_get_state()
    assert gl == -np.inf
    with pytest.raises(P.MpcgsError) as ei:
        ctx.mpcgs_sample(8, 16, 1)
    assert ei.value.status == -7
