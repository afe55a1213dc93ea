"""CPU oracle of the mpcgs hot path -- TEST INFRASTRUCTURE ONLY.

Plain FP64 C (``oracle/oracle.c``) behind a thin ctypes wrapper.  Only
``tests/``, ``__graft_entry__.smoke()`` and ``bench.py``'s ``cpu_baseline`` /
``--impl reference`` legs may import this package.  It shares no code with
``paper_conf_ipps_davistzw17_b200`` and never imports it.

Citations are PAPER.md lines (Davis 2016); readings S1..S23 are in DESIGN.md.
"""
from __future__ import annotations

import ctypes
import os
import subprocess

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_SRC = os.path.join(_HERE, "oracle.c")
_LIB_PATH = os.path.join(_HERE, "liboracle.so")
_lib = None

TAG_TARGET, TAG_PROPOSE, TAG_DRAW = 0, 1, 2

_i32p = np.ctypeslib.ndpointer(dtype=np.int32, flags="C_CONTIGUOUS")
_i64p = np.ctypeslib.ndpointer(dtype=np.int64, flags="C_CONTIGUOUS")
_f64p = np.ctypeslib.ndpointer(dtype=np.float64, flags="C_CONTIGUOUS")
_u8p = np.ctypeslib.ndpointer(dtype=np.uint8, flags="C_CONTIGUOUS")
_u32p = np.ctypeslib.ndpointer(dtype=np.uint32, flags="C_CONTIGUOUS")


def build(force: bool = False) -> str:
    """Compile oracle.c with gcc (plain -O2, no fast-math, no SIMD intrinsics)."""
    if force or not os.path.exists(_LIB_PATH) or os.path.getmtime(_LIB_PATH) < max(
        os.path.getmtime(_SRC), os.path.getmtime(os.path.join(_HERE, "oracle.h"))
    ):
        tmp = _LIB_PATH + f".tmp{os.getpid()}"
        subprocess.check_call(
            ["gcc", "-O2", "-std=c99", "-fno-fast-math", "-ffp-contract=off", "-fPIC", "-shared",
             "-o", tmp, _SRC, "-lm"]
        )
        os.replace(tmp, _LIB_PATH)
    return _LIB_PATH


def lib():
    global _lib
    if _lib is None:
        build()
        L = ctypes.CDLL(_LIB_PATH)
        c = ctypes
        L.orc_philox4x32_10.argtypes = [_u32p, _u32p, _u32p]
        L.orc_u01.argtypes = [c.c_uint32, c.c_uint32]
        L.orc_u01.restype = c.c_double
        L.orc_uniform.argtypes = [c.c_uint64, c.c_uint32, c.c_uint32, c.c_uint32, c.c_uint32]
        L.orc_uniform.restype = c.c_double
        L.orc_base_freqs.argtypes = [c.c_int, c.c_int, _u8p, _f64p]
        L.orc_default_rate.argtypes = [_f64p]
        L.orc_default_rate.restype = c.c_double
        L.orc_transition.argtypes = [c.c_double, c.c_double, _f64p, _f64p]
        L.orc_check_tree.argtypes = [c.c_int, _i32p, _f64p]
        L.orc_model_rate.argtypes = [c.c_int, c.c_double, _f64p]
        L.orc_model_rate.restype = c.c_double
        L.orc_transition_model.argtypes = [c.c_int, c.c_double, c.c_double, _f64p, _f64p]
        L.orc_log_likelihood_model.argtypes = [c.c_int, c.c_double, c.c_int, c.c_int, _u8p, _i32p, _f64p,
                                               _f64p, c.c_void_p]
        L.orc_log_likelihood_model.restype = c.c_double
        L.orc_log_likelihood.argtypes = [c.c_int, c.c_int, _u8p, _i32p, _f64p, _f64p, c.c_double,
                                         c.c_void_p]
        L.orc_log_likelihood.restype = c.c_double
        L.orc_coalescent_S.argtypes = [c.c_int, _f64p]
        L.orc_coalescent_S.restype = c.c_double
        L.orc_log_prior.argtypes = [c.c_int, _f64p, c.c_double]
        L.orc_log_prior.restype = c.c_double
        L.orc_pick_target.argtypes = [c.c_int, _i32p, c.c_uint64, c.c_uint32]
        L.orc_context_info.argtypes = [c.c_int, _i32p, _f64p, c.c_double, c.c_int, _i32p, _f64p,
                                       _f64p, _i32p, _i32p, _f64p, _f64p]
        L.orc_propose.argtypes = [c.c_int, _i32p, _f64p, c.c_double, c.c_int, c.c_uint64,
                                  c.c_uint32, c.c_uint32, _i32p, _f64p, _f64p, _i32p, _i32p]
        L.orc_weights.argtypes = [c.c_int, _f64p, _f64p, _f64p]
        L.orc_draw.argtypes = [c.c_int, _f64p, c.c_double, _i32p]
        L.orc_gmh_step.argtypes = [c.c_int, c.c_int, _u8p, _f64p, c.c_double, c.c_double, c.c_int,
                                   c.c_int, c.c_uint64, c.c_uint32, _i32p, _f64p, _f64p, _i32p,
                                   _f64p, _f64p, _f64p, _i32p, _i32p, _i32p, _i32p]
        L.orc_gmh_step_model.argtypes = [c.c_int, c.c_double, c.c_int, c.c_int, _u8p, _f64p, c.c_double,
                                         c.c_int, c.c_int, c.c_uint64, c.c_uint32, _i32p, _f64p, _f64p,
                                         _i32p, _f64p, _f64p, _f64p, _i32p, _i32p, _i32p, _i32p]
        L.orc_run_chain.argtypes = [c.c_int, c.c_int, _u8p, _f64p, c.c_double, c.c_double,
                                    c.c_int, c.c_int, c.c_int, c.c_uint64, _i32p, _f64p, _f64p,
                                    _f64p, _i64p, _i32p, _i32p, _i64p]
        L.orc_em.argtypes = [c.c_int, c.c_int, _u8p, _f64p, c.c_double, c.c_double, c.c_int, c.c_int,
                             c.c_int, c.c_uint64, c.c_int, c.c_int, _i32p, _f64p, _f64p, _i64p]
        L.orc_log_rel_likelihood.argtypes = [c.c_int, _f64p, c.c_int, c.c_double, c.c_double]
        L.orc_log_rel_likelihood.restype = c.c_double
        L.orc_weighted_mean_S.argtypes = [c.c_int, _f64p, c.c_double, c.c_double]
        L.orc_weighted_mean_S.restype = c.c_double
        L.orc_em_map.argtypes = [c.c_int, _f64p, c.c_int, c.c_double, c.c_double]
        L.orc_em_map.restype = c.c_double
        L.orc_theta_hat.argtypes = [c.c_int, _f64p, c.c_int, c.c_double, c.c_int, c.c_void_p,
                                    c.c_void_p]
        L.orc_theta_hat.restype = c.c_double
        L.orc_log_rel_likelihood_loci.argtypes = [c.c_int, _i32p, _f64p, _i32p, _f64p, c.c_double]
        L.orc_log_rel_likelihood_loci.restype = c.c_double
        L.orc_theta_hat_loci.argtypes = [c.c_int, _i32p, _f64p, _i32p, _f64p, c.c_int, c.c_void_p,
                                         c.c_void_p]
        L.orc_theta_hat_loci.restype = c.c_double
        L.orc_theta_alg2.argtypes = [c.c_int, _f64p, c.c_int, c.c_double, c.c_int]
        L.orc_theta_alg2.restype = c.c_double
        L.orc_upgma.argtypes = [c.c_int, c.c_int, _u8p, c.c_double, _i32p, _f64p]
        _lib = L
    return _lib


class OracleError(RuntimeError):
    pass


def _chk(rc):
    if rc != 0:
        raise OracleError(f"oracle returned {rc}")


def _tree(parent, age):
    return np.ascontiguousarray(parent, dtype=np.int32), np.ascontiguousarray(age, dtype=np.float64)


def _codes(codes):
    return np.ascontiguousarray(codes, dtype=np.uint8)


# ---------------------------------------------------------------- RNG
def philox(ctr, key):
    out = np.zeros(4, np.uint32)
    lib().orc_philox4x32_10(np.asarray(ctr, np.uint32), np.asarray(key, np.uint32), out)
    return out


def uniform(seed, c1, step, tag, idx):
    return lib().orc_uniform(seed, c1, step, tag, idx)


# ---------------------------------------------------------------- model
def base_freqs(codes):
    codes = _codes(codes)
    pi = np.zeros(4)
    lib().orc_base_freqs(codes.shape[0], codes.shape[1], codes, pi)
    return pi


def default_rate(pi):
    return lib().orc_default_rate(np.ascontiguousarray(pi, np.float64))


def transition(t, u, pi):
    P = np.zeros(16)
    lib().orc_transition(float(t), float(u), np.ascontiguousarray(pi, np.float64), P)
    return P.reshape(4, 4)


MODELS = {"F81": 0, "F84": 1, "HKY85": 2}


def model_rate(model, kappa, pi):
    return lib().orc_model_rate(MODELS[model], float(kappa), np.ascontiguousarray(pi, np.float64))


def transition_model(model, kappa, t, pi):
    P = np.zeros(16)
    lib().orc_transition_model(MODELS[model], float(kappa), float(t), np.ascontiguousarray(pi, np.float64), P)
    return P.reshape(4, 4)


def log_likelihood_model(model, kappa, codes, parent, age, pi):
    """ln P(D|G) under F81 / F84 / HKY85, Eq. 19-22 in log space."""
    codes = _codes(codes)
    parent, age = _tree(parent, age)
    n = (len(parent) + 1) // 2
    return lib().orc_log_likelihood_model(MODELS[model], float(kappa), n, codes.shape[1], codes, parent, age,
                                          np.ascontiguousarray(pi, np.float64), None)


def check_tree(parent, age):
    parent, age = _tree(parent, age)
    return lib().orc_check_tree((len(parent) + 1) // 2, parent, age)


def log_likelihood(codes, parent, age, pi, u, site_ll=False):
    """ln P(D|G): Eq. 19-22 (L660-719) in log space (5.3)."""
    codes = _codes(codes)
    parent, age = _tree(parent, age)
    n = (len(parent) + 1) // 2
    L = codes.shape[1] if codes.ndim == 2 else 0
    if codes.size == 0:
        codes = np.zeros((n, 1), np.uint8)
    buf = np.zeros(max(L, 1))
    ll = lib().orc_log_likelihood(n, L, codes, parent, age, np.ascontiguousarray(pi, np.float64),
                                  float(u), buf.ctypes.data if site_ll else None)
    return (ll, buf[:L]) if site_ll else ll


def coalescent_S(age, n):
    return lib().orc_coalescent_S(n, np.ascontiguousarray(age, np.float64))


def log_prior(age, n, theta):
    return lib().orc_log_prior(n, np.ascontiguousarray(age, np.float64), theta)


# ---------------------------------------------------------------- step
def pick_target(parent, seed, step):
    parent = np.ascontiguousarray(parent, np.int32)
    return lib().orc_pick_target((len(parent) + 1) // 2, parent, seed, step)


def context_info(parent, age, theta0, target):
    parent, age = _tree(parent, age)
    n = (len(parent) + 1) // 2
    info = np.zeros(9, np.int32)
    tau = np.zeros(n + 2)
    ln = np.zeros(n + 2)
    l = np.zeros(n + 2, np.int32)
    entry = np.zeros(n + 2, np.int32)
    om = np.zeros((n + 2) * 9)
    beta = np.zeros((n + 2) * 3)
    _chk(lib().orc_context_info(n, parent, age, theta0, target, info, tau, ln, l, entry, om, beta))
    m = int(info[5])
    return dict(T=int(info[0]), Par=int(info[1]), A=int(info[2]), rootcase=bool(info[3]),
                k0=int(info[4]), m=m, children=[int(x) for x in info[6:9]], tau=tau[: m + 1],
                len=ln[:m], l=l[:m], entry=entry[: m + 1], omega=om[: m * 9].reshape(m, 3, 3),
                beta=beta[: (m + 1) * 3].reshape(m + 1, 3))


def propose(parent, age, theta0, target, seed, step, slot):
    parent, age = _tree(parent, age)
    n = (len(parent) + 1) // 2
    np_, na = np.zeros_like(parent), np.zeros_like(age)
    t12 = np.zeros(2)
    pair = np.zeros(1, np.int32)
    flag = np.zeros(1, np.int32)
    _chk(lib().orc_propose(n, parent, age, theta0, target, seed, step, slot, np_, na, t12, pair,
                           flag))
    return np_, na, t12, int(pair[0]), bool(flag[0])


def weights(logL):
    logL = np.ascontiguousarray(logL, np.float64)
    w, cum = np.zeros_like(logL), np.zeros_like(logL)
    _chk(lib().orc_weights(len(logL), logL, w, cum))
    return w, cum


def draw(cum, u):
    flag = np.zeros(1, np.int32)
    i = lib().orc_draw(len(cum), np.ascontiguousarray(cum, np.float64), float(u), flag)
    return i, bool(flag[0])


def gmh_step(codes, pi, u, theta0, N, K, seed, step, parent, age, gen_logL, model="F81", kappa=0.0):
    """One GMH step (Alg. 1, Fig. 12). Returns a dict trace and the new generator.
    model "F84" / "HKY85": P(D|G) under that model, u unused."""
    codes = _codes(codes)
    parent, age = _tree(parent, age)
    parent, age = parent.copy(), age.copy()
    n = (len(parent) + 1) // 2
    gl = np.array([gen_logL], np.float64)
    tgt = np.zeros(1, np.int32)
    logL = np.zeros(N + 1)
    S = np.zeros(N + 1)
    t12 = np.zeros(2 * (N + 1))
    pair = np.zeros(N + 1, np.int32)
    sflag = np.zeros(N + 1, np.int32)
    draws = np.zeros(max(K, 1), np.int32)
    dflag = np.zeros(max(K, 1), np.int32)
    m = MODELS[model] if isinstance(model, str) else int(model)
    if m == 0:
        _chk(lib().orc_gmh_step(n, codes.shape[1], codes, np.ascontiguousarray(pi, np.float64),
                                float(u), theta0, N, K, seed, step, parent, age, gl, tgt, logL, S, t12,
                                pair, sflag, draws, dflag))
    else:
        _chk(lib().orc_gmh_step_model(m, float(kappa), n, codes.shape[1], codes,
                                      np.ascontiguousarray(pi, np.float64), theta0, N, K, seed, step,
                                      parent, age, gl, tgt, logL, S, t12, pair, sflag, draws, dflag))
    return dict(target=int(tgt[0]), logL=logL, S=S, t12=t12.reshape(N + 1, 2), pair=pair,
                slot_flag=sflag.astype(bool), draws=draws[:K], draw_flag=dflag[:K].astype(bool),
                parent=parent, age=age, gen_logL=float(gl[0]))


def run_chain(codes, pi, u, theta0, N, burnin, M, seed, parent, age):
    codes = _codes(codes)
    parent, age = _tree(parent, age)
    parent, age = parent.copy(), age.copy()
    n = (len(parent) + 1) // 2
    L = codes.shape[1]
    if L == 0:
        codes = np.zeros((n, 1), np.uint8)
    S = np.zeros(M)
    logL = np.zeros(M)
    st = np.zeros(M, np.int64)
    sl = np.zeros(M, np.int32)
    nf = np.zeros(1, np.int32)
    ff = np.zeros(1, np.int64)
    _chk(lib().orc_run_chain(n, L, codes, np.ascontiguousarray(pi, np.float64), float(u), theta0,
                             N, burnin, M, seed, parent, age, S, logL, st, sl, nf, ff))
    return dict(S=S, logL=logL, step=st, slot=sl, n_flagged=int(nf[0]), first_flag_step=int(ff[0]),
                parent=parent, age=age)


def em(codes, pi, u, theta0, N, burnin, M, seed, n_iter, parent, age, G=4096):
    """EM re-drive (Fig. 11): per iteration run_chain(seed + it) -> theta_hat -> theta0.
    Returns the theta trace, each iteration's first flagged step (-1: none) and the final genealogy."""
    codes = _codes(codes)
    parent, age = _tree(parent, age)
    parent, age = parent.copy(), age.copy()
    n = (len(parent) + 1) // 2
    trace = np.zeros(n_iter)
    ff = np.zeros(n_iter, np.int64)
    _chk(lib().orc_em(n, codes.shape[1], codes, np.ascontiguousarray(pi, np.float64), float(u), float(theta0), N,
                      burnin, M, seed, n_iter, G, parent, age, trace, ff))
    return dict(trace=trace, first_flag_step=ff, parent=parent, age=age)


# ---------------------------------------------------------------- MLE
def log_rel_likelihood(S, n, theta0, theta):
    S = np.ascontiguousarray(S, np.float64)
    return lib().orc_log_rel_likelihood(len(S), S, n, theta0, theta)


def weighted_mean_S(S, theta0, theta):
    S = np.ascontiguousarray(S, np.float64)
    return lib().orc_weighted_mean_S(len(S), S, theta0, theta)


def em_map(S, n, theta0, theta):
    S = np.ascontiguousarray(S, np.float64)
    return lib().orc_em_map(len(S), S, n, theta0, theta)


def theta_hat(S, n, theta0, G=4096, curve=False):
    S = np.ascontiguousarray(S, np.float64)
    gt, gl = np.zeros(G), np.zeros(G)
    th = lib().orc_theta_hat(len(S), S, n, theta0, G, gt.ctypes.data, gl.ctypes.data)
    return (th, gt, gl) if curve else th


def _loci(S_list, n_list, theta0_list):
    M = np.array([len(x) for x in S_list], np.int32)
    S = np.ascontiguousarray(np.concatenate([np.asarray(x, np.float64) for x in S_list]))
    return (len(S_list), M, S, np.ascontiguousarray(n_list, np.int32),
            np.ascontiguousarray(theta0_list, np.float64))


def log_rel_likelihood_loci(S_list, n_list, theta0_list, theta):
    """Joint ln L(theta) of independent loci sharing theta."""
    return lib().orc_log_rel_likelihood_loci(*_loci(S_list, n_list, theta0_list), theta)


def theta_hat_loci(S_list, n_list, theta0_list, G=4096, curve=False):
    gt, gl = np.zeros(G), np.zeros(G)
    th = lib().orc_theta_hat_loci(*_loci(S_list, n_list, theta0_list), G, gt.ctypes.data, gl.ctypes.data)
    return (th, gt, gl) if curve else th


def theta_alg2(S, n, theta0, max_iter=10000):
    S = np.ascontiguousarray(S, np.float64)
    return lib().orc_theta_alg2(len(S), S, n, theta0, max_iter)


def upgma(codes, theta0):
    codes = _codes(codes)
    n = codes.shape[0]
    parent = np.zeros(2 * n - 1, np.int32)
    age = np.zeros(2 * n - 1)
    _chk(lib().orc_upgma(n, codes.shape[1], codes, theta0, parent, age))
    return parent, age
