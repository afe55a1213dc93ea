"""CPU tests of the C-ABI library's host logic (no GPU needed): exports, the
Philox block, UPGMA, shard ranges, PHYLIP reading and the post-order register
schedule consumed by the pruning kernel (interpreted here with numpy and
compared with the oracle's likelihood)."""
import ctypes
import os
import re

import numpy as np
import pytest

import synth
import paper_conf_ipps_davistzw17_b200 as P
from paper_conf_ipps_davistzw17_b200 import mpcgs as B

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def test_library_exports_every_declared_symbol():
    lib = P.lib()
    header = open(os.path.join(ROOT, "include", "mpcgs.h")).read()
    declared = set(re.findall(r"\b(mpcgs_[a-z0-9_]+)\s*\(", header))
    declared -= {"mpcgs_status"}
    assert declared, "no declarations parsed"
    for name in declared:
        assert hasattr(lib, name), name
    assert declared == set(B.EXPORTS)


def test_philox_kat_product_side():
    assert list(P.mpcgs_philox([0, 0, 0, 0], [0, 0])) == [0x6627E8D5, 0xE169C58D, 0xBC57AC4C, 0x9B00DBD8]
    assert list(P.mpcgs_philox([0xFFFFFFFF] * 4, [0xFFFFFFFF] * 2)) == [0x408F276D, 0x41C83B0E, 0xA20BC7C6,
                                                                        0x6D5451FD]


def test_upgma_matches_oracle(orc):
    for name in ["c1", "c2", "c3"]:
        wl = synth.workload(name)
        p1, a1 = P.mpcgs_upgma(wl["codes"], wl["theta0"])
        p2, a2 = orc.upgma(wl["codes"], wl["theta0"])
        assert np.array_equal(p1, p2)
        assert np.allclose(a1, a2, rtol=1e-15)


def test_shard_ranges_partition_slots():
    for N, world in [(16, 1), (64, 2), (1024, 8), (512, 4)]:
        seen = []
        for r in range(world):
            f, c = P.mpcgs_shard_range(N, r, world)
            seen += list(range(f, f + c))
        assert seen == list(range(1, N + 1))
    with pytest.raises(P.MpcgsError):
        P.mpcgs_shard_range(10, 0, 3)


def test_workspace_bytes_monotone():
    a = P.mpcgs_workspace_bytes(12, 1000, 64, 20000, 64)
    b = P.mpcgs_workspace_bytes(12, 1000, 64, 40000, 64)
    c = P.mpcgs_workspace_bytes(12, 1000, 64, 20000, 32)
    assert 0 < c < a < b
    assert P.mpcgs_workspace_bytes(1, 10, 4, 4, 64) == 0


def test_phylip_reader(tmp_path):
    f = tmp_path / "x.phy"
    f.write_text("3 8\nalpha     ACGTACGT\nb ACGT ACGT\nc_long_nam\nacgtacgt\n")
    rows = P.mpcgs_phylip_read(str(f))
    assert rows == ["ACGTACGT", "ACGTACGT", "acgtacgt"]
    amb = tmp_path / "amb.phy"  # IUPAC characters are read; mpcgs_init decides (S2 / S24)
    amb.write_text("2 4\na ACGN\nb AC-R\n")
    assert P.mpcgs_phylip_read(str(amb)) == ["ACGN", "AC-R"]
    bad = tmp_path / "bad.phy"
    bad.write_text("2 4\na ACGX\nb ACGT\n")
    with pytest.raises(P.MpcgsError):
        P.mpcgs_phylip_read(str(bad))


def test_upgma_ambiguity_sets_match_oracle(orc):
    rng = np.random.default_rng(3)
    wl = synth.workload("c2")
    codes = synth.ambiguate(wl["codes"], 0.2, rng, gap_frac=0.05)
    p1, a1 = P.mpcgs_upgma(codes, wl["theta0"])
    p2, a2 = orc.upgma(codes, wl["theta0"])
    assert np.array_equal(p1, p2)
    assert np.allclose(a1, a2, rtol=1e-15)


def _interpret(op, e, codes, pi):
    """Run the register schedule of common.cuh in numpy (FP64), all sites at once."""
    L = codes.shape[1]
    R = {}

    def tip(x, ee, em):
        v = np.tile((em * pi[x])[None, :], (4, 1)).T.copy()  # [L,4] filled with em*pi_x
        v = np.repeat((em * pi[x])[:, None], 4, axis=1)
        v[np.arange(L), x] += ee
        return v

    def branch(v, ee, em):
        s = v @ pi
        return ee * v + em * s[:, None]

    for code, (ea, ema, eb, emb) in zip(op, e):
        typ, sp = code & 3, (code >> 2) & 15
        ta, tb = (code >> 6) & 2047, (code >> 17) & 2047
        if typ == 0:
            R[sp] = tip(codes[ta], ea, ema) * tip(codes[tb], eb, emb)
        elif typ == 1:
            R[sp - 1] = tip(codes[ta], ea, ema) * branch(R[sp - 1], eb, emb)
        else:
            R[sp - 2] = branch(R[sp - 2], ea, ema) * branch(R[sp - 1], eb, emb)
    return float(np.sum(np.log(R[0] @ pi)))


@pytest.mark.parametrize("n,shape", [(2, "random"), (3, "random"), (7, "caterpillar"), (16, "balanced"),
                                     (33, "random"), (64, "balanced")])
def test_schedule_semantics_match_oracle(orc, n, shape):
    rng = np.random.default_rng(n)
    parent, age = synth.shaped_tree(n, shape, rng, scale=0.05)
    pi = np.array([0.3, 0.2, 0.25, 0.25])
    u = orc.default_rate(pi)
    codes = synth.f81_alignment(parent, age, 50, pi, u, rng)
    op, e, depth = P.mpcgs_tree_schedule(parent, age, u)
    assert len(op) == n - 1
    assert depth <= max(1, int(np.floor(np.log2(n))))
    got = _interpret(op, e, codes, pi)
    want = orc.log_likelihood(codes, parent, age, pi, u)
    assert np.isclose(got, want, rtol=1e-12)


def test_schedule_register_need_bound():
    # a balanced tree of 2^k tips needs exactly k registers (Sethi-Ullman)
    for k in range(1, 9):
        n = 2 ** k
        parent, age = synth.shaped_tree(n, "balanced", np.random.default_rng(k))
        _, _, depth = P.mpcgs_tree_schedule(parent, age, 1.0)
        assert depth == k
    parent, age = synth.shaped_tree(200, "caterpillar", np.random.default_rng(0))
    assert P.mpcgs_tree_schedule(parent, age, 1.0)[2] == 1


@pytest.mark.parametrize("model", ["F84", "HKY85"])
def test_library_transition_matches_oracle_closed_forms(orc, model):
    """the library forms P(t) from the eigen-system of the normalised
    rate matrix (host.cu rate_matrix / eigen_system, device pmat); the oracle from
    the published closed forms (oracle.c orc_transition_model).  Independent routes."""
    rng = np.random.default_rng(7)
    pis = [np.full(4, 0.25), np.array([0.1, 0.2, 0.3, 0.4])] + [rng.dirichlet(np.ones(4) * 2) for _ in range(4)]
    for pi in pis:
        for kappa in [0.0, 0.5, 2.0, 10.0, 40.0]:
            for t in [0.0, 1e-9, 1e-4, 0.05, 0.7, 3.0, 50.0]:
                got = P.mpcgs_transition(model, kappa, pi, 0.0, t)
                ref = orc.transition_model(model, kappa, t, pi)
                assert np.allclose(got, ref, rtol=0, atol=2e-14), (model, pi, kappa, t)
                assert np.all(got >= 0.0)


def test_library_transition_f81_and_errors(orc):
    pi = np.array([0.1, 0.2, 0.3, 0.4])
    u = orc.default_rate(pi)
    for t in [0.0, 0.3, 4.0]:
        assert np.allclose(P.mpcgs_transition("F81", 0.0, pi, u, t), orc.transition(t, u, pi), rtol=0, atol=1e-15)
    with pytest.raises(P.MpcgsError):
        P.mpcgs_transition("F84", -1.0, pi, 0.0, 1.0)
    with pytest.raises(P.MpcgsError):
        P.mpcgs_transition("HKY85", 2.0, [0.5, 0.5, 0.0, 0.0], 0.0, 1.0)
    with pytest.raises(P.MpcgsError):
        P.mpcgs_transition(7, 2.0, pi, 0.0, 1.0)


def test_workspace_bytes_cfg_counts_model_buffers():
    cfg = B.mpcgs_config()
    P.lib().mpcgs_config_default(ctypes.byref(cfg))
    cfg.max_proposals, cfg.max_samples = 64, 20000
    f81 = P.lib().mpcgs_workspace_bytes_cfg(12, 1000, ctypes.byref(cfg))
    assert f81 == P.mpcgs_workspace_bytes(12, 1000, 64, 20000, 64)
    cfg.model = P.MODELS["F84"]
    assert P.lib().mpcgs_workspace_bytes_cfg(12, 1000, ctypes.byref(cfg)) >= f81 + 64 * 11 * 32 * 8


# ------------------------------------------------------------------ Newick G0 (SURVEY 8(b) init_newick)
def _newick(parent, age):
    """Plain recursive Newick writer (tips labelled by row index)."""
    parent = np.asarray(parent)
    nn = len(parent)
    n = (nn + 1) // 2
    kids = {v: [] for v in range(nn)}
    for v in range(nn):
        if parent[v] >= 0:
            kids[int(parent[v])].append(v)
    root = int(np.where(parent < 0)[0][0])

    def rec(v):
        if v < n:
            return str(v)
        return "(" + ",".join(f"{rec(c)}:{float(age[v] - age[c])!r}" for c in kids[v]) + ")"

    return rec(root) + ";"


def test_parse_newick_hand_example():
    import paper_conf_ipps_davistzw17_b200 as P

    # ((0,1) at 0.1, 2) at 0.4, with 3 joined at the root 1.0
    p, a = P.mpcgs_parse_newick(4, " (((0:0.1, 1:0.1)x:0.3,2:0.4):0.6, 3:1.0);\n")
    assert list(p) == [4, 4, 5, 6, 5, 6, -1]
    assert np.allclose(a, [0, 0, 0, 0, 0.1, 0.4, 1.0], rtol=0, atol=1e-15)


def test_parse_newick_roundtrip_random_trees():
    import paper_conf_ipps_davistzw17_b200 as P

    rng = np.random.default_rng(12)
    for n in (2, 3, 5, 12, 64, 257):
        p, a = synth.coalescent_tree(n, 0.7, rng)   # interior ids already in ascending age
        gp, ga = P.mpcgs_parse_newick(n, _newick(p, a))
        assert np.array_equal(gp, p)
        assert np.allclose(ga, a, rtol=1e-13, atol=1e-15)


@pytest.mark.parametrize("bad", [
    "((0:0.1,1:0.1):0.3,2:0.4)",            # no ';'
    "((0:0.1,1:0.1):0.3,2);",               # missing length
    "((0:0.1,1:0.1):0.3,2:0.9);",           # not contemporaneous
    "((0:0.1,1:0.1,2:0.1):0.3,3:0.4);",     # multifurcation
    "((0:0.1,0:0.1):0.3,2:0.4);",           # duplicate tip
    "((0:0.1,5:0.1):0.3,2:0.4);",           # label out of range
    "((a:0.1,1:0.1):0.3,2:0.4);",           # non-numeric label
    "((0:0.1,1:-0.1):0.3,2:0.2);",          # negative length
    "(0:0.4,1:0.4);",                       # too few tips for n = 3
])
def test_parse_newick_errors(bad):
    import paper_conf_ipps_davistzw17_b200 as P

    with pytest.raises(P.MpcgsError):
        P.mpcgs_parse_newick(3, bad)
