"""Seeded synthetic inputs shared by the oracle-side tests and the CUDA path.

This module holds NONE of the method's arithmetic (no pruning, no resimulation,
no weights, no MLE).  It only generates inputs shaped like the paper's
workloads (PAPER.md 6.1 L1494-1518: ``ms 12 1 -T`` coalescent trees and
``seq-gen`` sequences; here F81 instead of seq-gen's F84, reading in DESIGN.md):

* ``coalescent_tree``   -- Kingman coalescent with parameter theta: while k
  lineages remain, wait Exp(rate k(k-1)/theta), merge a uniform pair; node ids
  in creation order (tips 0..n-1, interior n..2n-2).
* ``f81_alignment``     -- root base ~ pi; along a branch of length t the base is
  kept with probability e^{-ut}, else redrawn from pi.
* ``shaped_tree``       -- caterpillar / balanced / random topologies with
  adversarial branch lengths for likelihood parity tests.
* ``workload``          -- the BASELINE.json configs c1..c5 (data seed
  1000 + 100*config + sweep index, chain seed 2000 + 100*config + sweep index).

Everything is numpy ``default_rng(seed)``; nothing here touches a GPU.
"""
from __future__ import annotations

import numpy as np

BASES = "ACGT"


def coalescent_tree(n: int, theta: float, rng: np.random.Generator):
    parent = np.full(2 * n - 1, -1, np.int32)
    age = np.zeros(2 * n - 1)
    active = list(range(n))
    t = 0.0
    nxt = n
    while len(active) > 1:
        k = len(active)
        t += rng.exponential(theta / (k * (k - 1)))
        i, j = rng.choice(k, size=2, replace=False)
        a, b = active[i], active[j]
        parent[a] = nxt
        parent[b] = nxt
        age[nxt] = t
        active = [x for x in active if x not in (a, b)] + [nxt]
        nxt += 1
    return parent, age


def f81_alignment(parent, age, L: int, pi, u: float, rng: np.random.Generator):
    parent = np.asarray(parent)
    nn = len(parent)
    n = (nn + 1) // 2
    pi = np.asarray(pi, np.float64)
    states = np.zeros((nn, L), np.uint8)
    root = int(np.where(parent < 0)[0][0])
    states[root] = rng.choice(4, size=L, p=pi)
    # visit nodes from old to young so that a parent is drawn before its children
    order = sorted(range(nn), key=lambda v: -age[v])
    for v in order:
        if v == root:
            continue
        p = parent[v]
        t = age[p] - age[v]
        keep = rng.random(L) < np.exp(-u * t)
        fresh = rng.choice(4, size=L, p=pi).astype(np.uint8)
        states[v] = np.where(keep, states[p], fresh)
    return np.ascontiguousarray(states[:n])


def shaped_tree(n: int, shape: str, rng: np.random.Generator, scale: float = 1.0):
    """Random-label tree of the given shape with increasing node ages.

    shape: 'caterpillar' | 'balanced' | 'random'.  Ages are cumulative sums of
    Exp(scale) increments; callers overwrite them for adversarial lengths.
    """
    parent = np.full(2 * n - 1, -1, np.int32)
    age = np.zeros(2 * n - 1)
    pool = list(rng.permutation(n))
    nxt = n
    t = 0.0
    if shape == "caterpillar":
        cur = pool.pop()
        while pool:
            other = pool.pop()
            t += rng.exponential(scale)
            parent[cur] = parent[other] = nxt
            age[nxt] = t
            cur = nxt
            nxt += 1
    elif shape == "balanced":
        level = pool
        while len(level) > 1:
            new = []
            for i in range(0, len(level) - 1, 2):
                t += rng.exponential(scale) / len(level)
                parent[level[i]] = parent[level[i + 1]] = nxt
                age[nxt] = max(age[level[i]], age[level[i + 1]]) + rng.exponential(scale)
                new.append(nxt)
                nxt += 1
            if len(level) % 2:
                new.append(level[-1])
            level = new
    else:
        active = pool
        while len(active) > 1:
            i, j = rng.choice(len(active), size=2, replace=False)
            a, b = active[i], active[j]
            t += rng.exponential(scale)
            parent[a] = parent[b] = nxt
            age[nxt] = max(t, age[a], age[b])
            active = [x for x in active if x not in (a, b)] + [nxt]
            nxt += 1
    return parent, age


def random_alignment(n: int, L: int, rng: np.random.Generator, pi=None):
    pi = np.full(4, 0.25) if pi is None else np.asarray(pi)
    return rng.choice(4, size=(n, L), p=pi).astype(np.uint8)


# IUPAC ambiguity letters by base-set mask (bit X = base X of A, C, G, T); code 16 + mask
IUPAC = {1: "A", 2: "C", 4: "G", 8: "T", 5: "R", 10: "Y", 6: "S", 9: "W", 12: "K", 3: "M",
         14: "B", 13: "D", 11: "H", 7: "V", 15: "N"}


def _letter(c: int) -> str:
    return BASES[c] if c < 4 else IUPAC[c - 16]


def to_strings(codes):
    return ["".join(_letter(int(c)) for c in row) for row in np.asarray(codes)]


def ambiguate(codes, frac: float, rng: np.random.Generator, gap_frac: float = 0.0):
    """Replace a fraction of characters by ambiguity codes (16 + mask, the mask
    drawn uniformly among the multi-base IUPAC sets containing the replaced base,
    N included) and a further fraction by N (gaps / missing data)."""
    out = np.array(codes, dtype=np.uint8, copy=True)
    multi = [m for m in IUPAC if bin(m).count("1") > 1]
    having = [np.array([m for m in multi if (m >> x) & 1], dtype=np.uint8) for x in range(4)]
    hit = np.argwhere(rng.random(out.shape) < frac)
    for i, j in hit:  # a set that contains the base it replaces
        out[i, j] = 16 + rng.choice(having[int(codes[i][j]) if codes[i][j] < 4 else 0])
    gap = rng.random(out.shape) < gap_frac
    out[gap] = 16 + 15
    return out


# BASELINE.json configs: (n, L, N, M, theta0)
CONFIGS = {
    "c1": dict(n=4, L=100, N=16, M=1000, theta0=0.01),
    "c2": dict(n=12, L=1000, N=64, M=20000, theta0=0.01),
    "c3": dict(n=24, L=1000, N=256, M=10000, theta0=0.01),
    "c4": dict(n=64, L=2000, N=512, M=0, theta0=0.01),
    "c5": dict(n=64, L=100000, N=1024, M=0, theta0=0.01),
}


def workload(name: str, sweep: int = 0, theta_true: float = 1.0, **override):
    """Synthetic workload for config `name`: coalescent tree at theta_true, F81
    alignment with uniform pi (seq-gen's default), u = 1/(1 - sum pi^2)."""
    cfg = dict(CONFIGS[name])
    cfg.update(override)
    idx = int(name[1:])
    data_seed = 1000 + 100 * idx + sweep
    chain_seed = 2000 + 100 * idx + sweep
    rng = np.random.default_rng(data_seed)
    parent, age = coalescent_tree(cfg["n"], theta_true, rng)
    pi = np.full(4, 0.25)
    u = 1.0 / (1.0 - float(np.sum(pi * pi)))
    codes = f81_alignment(parent, age, cfg["L"], pi, u, rng)
    cfg.update(true_parent=parent, true_age=age, codes=codes, data_seed=data_seed,
               chain_seed=chain_seed, theta_true=theta_true)
    return cfg
