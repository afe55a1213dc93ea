"""Independent numerical integrals used to pin the oracle's resimulation and
GMH step.

Nothing here calls the oracle.  The only model facts used are

* the coalescent prior density of a labelled history with times,
  (2/theta)^{n-1} exp(-S/theta), S = 2 sum_i (n-i) h_i over sorted coalescence
  ages h_i (Eq. 18; the identity is proven in tests), and
* the F81 transition matrix as the matrix exponential of its generator.

The conditional law of a LAMARC neighbourhood given the rest of the tree is the
prior restricted to the valid (x, y, pair) configurations (L1039-1043): the
younger new node at age x joins the chosen pair, the older at age y joins the
third child, and y stays below the ancestor.
"""
import itertools
import math

import numpy as np
import scipy.integrate
import scipy.linalg


def children(parent):
    nn = len(parent)
    kids = {v: [] for v in range(nn)}
    for v in range(nn):
        if parent[v] >= 0:
            kids[int(parent[v])].append(v)
    return kids


def neighbourhood(parent, age, target):
    kids = children(parent)
    par = int(parent[target])
    anc = int(parent[par])
    sib = [c for c in kids[par] if c != target][0]
    cs = sorted(kids[target] + [sib], key=lambda v: (age[v], v))
    n = (len(parent) + 1) // 2
    fixed = [float(age[v]) for v in range(n, len(parent)) if v not in (target, par)]
    t_anc = float(age[anc]) if anc >= 0 else math.inf
    return cs, fixed, t_anc


def S_of(fixed, x, y, n):
    h = sorted(fixed + [x, y])
    return 2.0 * sum((n - i) * h[i - 1] for i in range(1, n))


PAIRS = [(0, 1, 2), (0, 2, 1), (1, 2, 0)]   # (pair child, pair child, third child)


def piecewise_quad(g, lo, hi, pts, epsrel):
    """Integral of g over [lo, hi] split at the kinks pts (hi may be +inf)."""
    edges = [lo] + [p for p in sorted(pts) if lo < p < hi] + [hi]
    return sum(scipy.integrate.quad(g, a, b, limit=200, epsabs=0, epsrel=epsrel)[0]
               for a, b in zip(edges[:-1], edges[1:]) if b > a)


def restricted_prior_integral(parent, age, theta, target, f=lambda x, y, pair: 1.0):
    """sum_pair int int f(x, y, pair) exp(-S/theta) over the valid region."""
    n = (len(parent) + 1) // 2
    cs, fixed, t_anc = neighbourhood(parent, age, target)
    a = [float(age[c]) for c in cs]
    s0 = S_of(fixed, a[2], a[2], n)   # constant offset to keep exp() in range
    pts = sorted(set(fixed + a))
    total = 0.0
    for pc, (i, j, k) in enumerate(PAIRS):
        xlo = max(a[i], a[j])

        def inner(x):
            ylo = max(x, a[k])
            g = lambda y: f(x, y, pc) * math.exp(-(S_of(fixed, x, y, n) - s0) / theta)
            return piecewise_quad(g, ylo, t_anc, pts + [x], 1e-11)

        total += piecewise_quad(inner, xlo, t_anc, pts, 1e-10)
    return total


_EIG = {}


def f81_P(t, pi, u):
    """exp(Q t) for the F81 generator, via an eigendecomposition of Q cached per (pi, u)."""
    key = (tuple(np.round(pi, 15)), u)
    if key not in _EIG:
        Q = u * np.tile(pi, (4, 1))
        np.fill_diagonal(Q, 0.0)
        np.fill_diagonal(Q, -Q.sum(axis=1))
        lam, V = np.linalg.eig(Q)
        _EIG[key] = (lam.real, V.real, np.linalg.inv(V).real)
    lam, V, Vi = _EIG[key]
    return (V * np.exp(lam * t)) @ Vi


def three_tip_likelihood(codes, x, y, pair, pi, u):
    """P(D|G) for n=3 by summing over the two interior states (brute force)."""
    i, j, k = PAIRS[pair]
    Px = f81_P(x, pi, u)          # tips i, j to the younger node
    Pk = f81_P(y, pi, u)          # tip k to the root
    Pxy = f81_P(y - x, pi, u)     # younger node to the root
    L = np.zeros(codes.shape[1])
    for r, v in itertools.product(range(4), range(4)):
        L += pi[r] * Pk[r, codes[k]] * Pxy[r, v] * Px[v, codes[i]] * Px[v, codes[j]]
    return float(np.prod(L))
