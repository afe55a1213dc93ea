"""Thin ctypes binding of libmpcgs.so (include/mpcgs.h): argument marshalling only.

Every function keeps the C name.  Host arrays are numpy; device memory
(the workspace) and the stream may come from PyTorch.  There is no CPU
fallback: if the CUDA library is missing or fails to load, every call raises.
"""
from __future__ import annotations

import ctypes
import os

import numpy as np

from . import _build

MPCGS_OK = 0
STATUS_NAMES = {0: "OK", -1: "E_ARG", -2: "E_ALIGNMENT", -3: "E_STATE", -4: "E_CUDA", -5: "E_NCCL",
                -6: "E_NOMEM", -7: "E_NUMERIC"}
MAX_SEQ, MAX_PROPOSALS, MAX_GRID = 1024, 4096, 4096
REC = 5


class MpcgsError(RuntimeError):
    def __init__(self, status, msg=""):
        super().__init__(f"mpcgs {STATUS_NAMES.get(status, status)}: {msg}")
        self.status = status


class mpcgs_alignment(ctypes.Structure):
    _fields_ = [("n_seq", ctypes.c_int32), ("n_sites", ctypes.c_int32),
                ("rows", ctypes.POINTER(ctypes.c_char_p))]


class mpcgs_config(ctypes.Structure):
    _fields_ = [
        ("base_freq", ctypes.c_double * 4), ("mu", ctypes.c_double), ("precision", ctypes.c_int32),
        ("burnin_steps", ctypes.c_int32), ("max_proposals", ctypes.c_int32),
        ("max_samples", ctypes.c_int64), ("init_parent", ctypes.c_void_p),
        ("init_age", ctypes.c_void_p), ("rank", ctypes.c_int32), ("world", ctypes.c_int32),
        ("nccl_id", ctypes.c_void_p), ("stream", ctypes.c_void_p), ("workspace", ctypes.c_void_p),
        ("workspace_bytes", ctypes.c_size_t), ("incremental", ctypes.c_int32),
        ("compress_patterns", ctypes.c_int32), ("model", ctypes.c_int32), ("kappa", ctypes.c_double),
        ("ambiguity", ctypes.c_int32), ("init_newick", ctypes.c_char_p),
    ]


MODELS = {"F81": 0, "F84": 1, "HKY85": 2}  # MPCGS_MODEL_*


_lib = None
_P = ctypes.c_void_p
_i32, _i64, _u64, _f64, _sz = ctypes.c_int32, ctypes.c_int64, ctypes.c_uint64, ctypes.c_double, ctypes.c_size_t

# name: (restype, argtypes)
_SIGS = {
    "mpcgs_config_default": (None, [_P]),
    "mpcgs_workspace_bytes": (_sz, [_i32, _i32, _i32, _i64, _i32]),
    "mpcgs_workspace_bytes_ex": (_sz, [_i32, _i32, _i32, _i64, _i32, _i32]),
    "mpcgs_workspace_bytes_cfg": (_sz, [_i32, _i32, _P]),
    "mpcgs_transition": (_i32, [_i32, _f64, _P, _f64, _f64, _P]),
    "mpcgs_init": (_i32, [_P, _P, _f64, _P]),
    "mpcgs_init_phylip": (_i32, [ctypes.c_char_p, _P, _f64, _P]),
    "mpcgs_sample": (_i32, [_P, _i32, _i64, _u64]),
    "mpcgs_sample_steps": (_i32, [_P, _i32, _i64, _u64, _i64, _i64]),
    "mpcgs_put_samples": (_i32, [_P, _i64, _P, _P, _P, _P]),
    "mpcgs_state_bytes": (ctypes.c_size_t, [_P]),
    "mpcgs_save_state": (_i32, [_P, _P, ctypes.c_size_t]),
    "mpcgs_load_state": (_i32, [_P, _P, ctypes.c_size_t]),
    "mpcgs_estimate_theta": (_i32, [_P, _P, _i32, _P, _P]),
    "mpcgs_log_rel_likelihood": (_i32, [_P, _f64, _P]),
    "mpcgs_score_trees": (_i32, [_P, _i32, _P, _P, _P]),
    "mpcgs_set_state": (_i32, [_P, _P, _P]),
    "mpcgs_get_state": (_i32, [_P, _P, _P, _P, _P]),
    "mpcgs_step_trace": (_i32, [_P, _i64, _i32, _i32, _u64, _P, _P, _P, _P, _P, _P]),
    "mpcgs_step_local": (_i32, [_P, _i64, _i32, _u64]),
    "mpcgs_get_records": (_i32, [_P, _i32, _i32, _P]),
    "mpcgs_put_records": (_i32, [_P, _i32, _i32, _P]),
    "mpcgs_step_finish": (_i32, [_P, _i64, _i32, _i32, _u64, _P]),
    "mpcgs_get_samples": (_i32, [_P, _i64, _i64, _P, _P, _P, _P]),
    "mpcgs_num_samples": (_i64, [_P]),
    "mpcgs_load_samples": (_i32, [_P, _i64, _P, _P, _f64]),
    "mpcgs_num_patterns": (_i32, [_P]),
    "mpcgs_set_theta0": (_i32, [_P, _f64]),
    "mpcgs_em": (_i32, [_P, _i32, _i32, _i64, _u64, _i32, _P]),
    "mpcgs_get_model": (_i32, [_P, _P, _P]),
    "mpcgs_sample_loci": (_i32, [_P, _i32, _i32, _i64, _P]),
    "mpcgs_estimate_theta_loci": (_i32, [_P, _i32, _P, _i32, _P, _P]),
    "mpcgs_em_loci": (_i32, [_P, _i32, _i32, _i32, _i64, _P, _i32, _P]),
    "mpcgs_set_timing": (_i32, [_P, _i32]),
    "mpcgs_last_timing": (_i32, [_P, _P, _P, _P]),
    "mpcgs_last_timing_ex": (_i32, [_P, _P, _P]),
    "mpcgs_probe_peak": (_i32, [_i32, _P]),
    "mpcgs_last_error": (ctypes.c_char_p, [_P]),
    "mpcgs_free": (None, [_P]),
    "mpcgs_shard_range": (_i32, [_i32, _i32, _i32, _P, _P]),
    "mpcgs_upgma": (_i32, [_i32, _i32, _P, _f64, _P, _P]),
    "mpcgs_tree_schedule": (_i32, [_i32, _P, _P, _f64, _P, _P]),
    "mpcgs_parse_newick": (_i32, [_i32, ctypes.c_char_p, _P, _P]),
    "mpcgs_prune_tiling": (_i32, [_i32, _i32, _i32, _i32, _P, _P, _P]),
    "mpcgs_phylip_dims": (_i32, [ctypes.c_char_p, _P, _P]),
    "mpcgs_phylip_read": (_i32, [ctypes.c_char_p, _P, _i32]),
    "mpcgs_philox": (None, [_P, _P, _P]),
    "mpcgs_nccl_unique_id": (_i32, [_P]),
    "mpcgs_version": (ctypes.c_char_p, []),
}
EXPORTS = tuple(_SIGS)


def lib(build_if_missing: bool = True):
    """Load (building if stale) the in-tree libmpcgs.so.  Raises if it cannot."""
    global _lib
    if _lib is None:
        path = os.environ.get("MPCGS_LIB", _build.LIB)  # tuning variants only; default in-tree build
        if path == _build.LIB and build_if_missing and _build.stale():
            _build.build()
        if not os.path.exists(path):
            raise MpcgsError(-4, f"CUDA library missing: {path}")
        L = ctypes.CDLL(path)
        for name, (res, args) in _SIGS.items():
            if path != _build.LIB and not hasattr(L, name):
                continue  # an older tuning variant (A/B runs) may lack newer entry points
            f = getattr(L, name)
            f.restype = res
            f.argtypes = args
        _lib = L
    return _lib


def _ptr(a):
    return None if a is None else a.ctypes.data


def _f64a(x, n=None):
    a = np.ascontiguousarray(x, dtype=np.float64)
    if n is not None and a.size != n:
        raise ValueError(f"expected {n} doubles, got {a.size}")
    return a


def _i32a(x, n=None):
    a = np.ascontiguousarray(x, dtype=np.int32)
    if n is not None and a.size != n:
        raise ValueError(f"expected {n} int32, got {a.size}")
    return a


# ------------------------------------------------------------------ host-only
def mpcgs_version():
    return lib().mpcgs_version().decode()


def mpcgs_workspace_bytes(n_seq, n_sites, max_proposals, max_samples, precision=64):
    return int(lib().mpcgs_workspace_bytes(n_seq, n_sites, max_proposals, max_samples, precision))


def mpcgs_shard_range(n_proposals, rank, world):
    f, c = ctypes.c_int32(), ctypes.c_int32()
    st = lib().mpcgs_shard_range(n_proposals, rank, world, ctypes.byref(f), ctypes.byref(c))
    if st:
        raise MpcgsError(st, "shard_range")
    return f.value, c.value


def mpcgs_upgma(codes, theta0):
    codes = np.ascontiguousarray(codes, dtype=np.uint8)
    n, L = codes.shape
    parent = np.zeros(2 * n - 1, np.int32)
    age = np.zeros(2 * n - 1)
    st = lib().mpcgs_upgma(n, L, _ptr(codes), theta0, _ptr(parent), _ptr(age))
    if st:
        raise MpcgsError(st, "upgma")
    return parent, age


def mpcgs_tree_schedule(parent, age, mu):
    parent = _i32a(parent)
    age = _f64a(age)
    n = (len(parent) + 1) // 2
    op = np.zeros(n - 1, np.uint32)
    e = np.zeros(4 * (n - 1))
    d = lib().mpcgs_tree_schedule(n, _ptr(parent), _ptr(age), mu, _ptr(op), _ptr(e))
    if d < 0:
        raise MpcgsError(d, "tree_schedule")
    return op, e.reshape(n - 1, 4), d


def mpcgs_prune_tiling(n_seq, n_sites, ntrees, precision=64):
    """(tiles, sites_per_cta, unit_batches) of one pruning launch over ntrees genealogies."""
    t, s, u = ctypes.c_int32(), ctypes.c_int32(), ctypes.c_int32()
    st = lib().mpcgs_prune_tiling(n_seq, n_sites, ntrees, precision, ctypes.byref(t), ctypes.byref(s), ctypes.byref(u))
    if st:
        raise MpcgsError(st, "prune_tiling")
    return t.value, s.value, u.value


def mpcgs_parse_newick(n_seq, newick):
    parent = np.zeros(2 * n_seq - 1, np.int32)
    age = np.zeros(2 * n_seq - 1)
    st = lib().mpcgs_parse_newick(int(n_seq), newick.encode(), _ptr(parent), _ptr(age))
    if st:
        raise MpcgsError(st, "parse_newick")
    return parent, age


def mpcgs_phylip_read(path):
    n, L = ctypes.c_int32(), ctypes.c_int32()
    st = lib().mpcgs_phylip_dims(path.encode(), ctypes.byref(n), ctypes.byref(L))
    if st:
        raise MpcgsError(st, path)
    buf = ctypes.create_string_buffer(n.value * L.value)
    st = lib().mpcgs_phylip_read(path.encode(), buf, n.value * L.value)
    if st:
        raise MpcgsError(st, path)
    raw = buf.raw
    return [raw[i * L.value:(i + 1) * L.value].decode() for i in range(n.value)]


def mpcgs_philox(ctr, key):
    c = np.ascontiguousarray(ctr, np.uint32)
    k = np.ascontiguousarray(key, np.uint32)
    out = np.zeros(4, np.uint32)
    lib().mpcgs_philox(_ptr(c), _ptr(k), _ptr(out))
    return out


def mpcgs_transition(model, kappa, pi, mu, t):
    """P(t) as the kernels form it (host-only entry point); model name or MPCGS_MODEL_* code."""
    m = MODELS[model] if isinstance(model, str) else int(model)
    p = _f64a(pi)
    out = np.zeros(16, np.float64)
    st = lib().mpcgs_transition(m, float(kappa), _ptr(p), float(mu), float(t), _ptr(out))
    if st:
        raise MpcgsError(st, "transition")
    return out.reshape(4, 4)


# ------------------------------------------------------------------ multiple loci (f4)
def _loci_args(contexts, seeds=None):
    hs = (ctypes.c_void_p * len(contexts))(*[c.h for c in contexts])
    sd = None if seeds is None else np.ascontiguousarray(seeds, np.uint64)
    return hs, sd


def _loci_err(st, contexts, what):
    if st:
        msgs = [lib().mpcgs_last_error(c.h).decode() for c in contexts if c.h]
        raise MpcgsError(st, f"{what}: {'; '.join(m for m in msgs if m)}")


def mpcgs_sample_loci(contexts, n_proposals, n_samples, seeds):
    """Sample every locus (one Context each) with its own seed; loops overlap on the GPU."""
    hs, sd = _loci_args(contexts, seeds)
    _loci_err(lib().mpcgs_sample_loci(hs, len(contexts), n_proposals, n_samples, _ptr(sd)), contexts,
              "sample_loci")


def mpcgs_estimate_theta_loci(contexts, n_grid=256, curve=False):
    """Joint theta-hat of loci sharing theta (product of Eq. 25 over loci)."""
    hs, _ = _loci_args(contexts)
    th = ctypes.c_double()
    gt, gl = np.zeros(n_grid), np.zeros(n_grid)
    _loci_err(lib().mpcgs_estimate_theta_loci(hs, len(contexts), ctypes.byref(th), n_grid, _ptr(gt), _ptr(gl)),
              contexts, "estimate_theta_loci")
    return (th.value, gt, gl) if curve else th.value


def mpcgs_em_loci(contexts, n_iter, n_proposals, n_samples, seeds, n_grid=256):
    hs, sd = _loci_args(contexts, seeds)
    trace = np.zeros(n_iter)
    _loci_err(lib().mpcgs_em_loci(hs, len(contexts), n_iter, n_proposals, n_samples, _ptr(sd), n_grid,
                                  _ptr(trace)), contexts, "em_loci")
    return trace


def mpcgs_probe_peak(kind):
    """Measured FP64 FMA (0, TFLOP/s), FP32 FMA (1, TFLOP/s) or shared-memory load (2, GB/s) peak."""
    v = ctypes.c_double()
    st = lib().mpcgs_probe_peak(int(kind), ctypes.byref(v))
    if st:
        raise MpcgsError(st, "probe_peak")
    return v.value


def mpcgs_nccl_unique_id():
    buf = ctypes.create_string_buffer(128)
    st = lib().mpcgs_nccl_unique_id(buf)
    if st:
        raise MpcgsError(st, "nccl unique id")
    return buf.raw


# ------------------------------------------------------------------ context API
def _config(precision=64, burnin_steps=0, max_proposals=1024, max_samples=1 << 20, base_freq=None, mu=0.0,
            incremental=False, compress_patterns=False, model="F81", kappa=0.0, ambiguity=False):
    cfg = mpcgs_config()
    lib().mpcgs_config_default(ctypes.byref(cfg))
    if base_freq is not None:
        for i in range(4):
            cfg.base_freq[i] = float(base_freq[i])
    cfg.mu = float(mu)
    cfg.precision = int(precision)
    cfg.burnin_steps = int(burnin_steps)
    cfg.max_proposals = int(max_proposals)
    cfg.max_samples = int(max_samples)
    cfg.incremental = int(bool(incremental))
    cfg.compress_patterns = int(bool(compress_patterns))
    cfg.model = MODELS[model] if isinstance(model, str) else int(model)
    cfg.kappa = float(kappa)
    cfg.ambiguity = int(bool(ambiguity))
    return cfg


def mpcgs_workspace_bytes_cfg(n_seq, n_sites, **options):
    """Device bytes a context of these capacities / options needs (Context keyword names):
    a caller-owned workspace of this size can be passed as Context(..., workspace=(ptr, bytes))."""
    cfg = _config(**options)
    return int(lib().mpcgs_workspace_bytes_cfg(int(n_seq), int(n_sites), ctypes.byref(cfg)))


class Context:
    """Owns an mpcgs_ctx*.  Methods map 1:1 to the C entry points."""

    def __init__(self, rows, theta0, *, precision=64, burnin_steps=0, max_proposals=1024,
                 max_samples=1 << 20, base_freq=None, mu=0.0, init_tree=None, rank=0, world=1,
                 nccl_id=None, stream=None, workspace=None, phylip=None, incremental=False,
                 compress_patterns=False, model="F81", kappa=0.0, ambiguity=False, init_newick=None):
        L = lib()
        cfg = _config(precision, burnin_steps, max_proposals, max_samples, base_freq, mu, incremental,
                      compress_patterns, model, kappa, ambiguity)
        self._keep = []
        if init_newick is not None:
            nw = init_newick.encode() if isinstance(init_newick, str) else bytes(init_newick)
            self._keep.append(nw)
            cfg.init_newick = nw
        if init_tree is not None:
            p = _i32a(init_tree[0])
            a = _f64a(init_tree[1])
            self._keep += [p, a]
            cfg.init_parent = p.ctypes.data
            cfg.init_age = a.ctypes.data
        cfg.rank, cfg.world = int(rank), int(world)
        if nccl_id is not None:
            idbuf = ctypes.create_string_buffer(bytes(nccl_id), 128)
            self._keep.append(idbuf)
            cfg.nccl_id = ctypes.cast(idbuf, ctypes.c_void_p).value
        cfg.stream = stream
        if workspace is not None:
            cfg.workspace = int(workspace[0])
            cfg.workspace_bytes = int(workspace[1])
        h = ctypes.c_void_p()
        if phylip is not None:
            rows = mpcgs_phylip_read(phylip)
            st = L.mpcgs_init_phylip(phylip.encode(), ctypes.byref(cfg), float(theta0), ctypes.byref(h))
        else:
            rows = [r.encode() if isinstance(r, str) else bytes(r) for r in rows]
            arr = (ctypes.c_char_p * len(rows))(*rows)
            aln = mpcgs_alignment(len(rows), len(rows[0]) if rows else 0,
                                  ctypes.cast(arr, ctypes.POINTER(ctypes.c_char_p)))
            st = L.mpcgs_init(ctypes.byref(aln), ctypes.byref(cfg), float(theta0), ctypes.byref(h))
        self.h = h.value
        if st:
            msg = L.mpcgs_last_error(self.h).decode() if self.h else ""
            self.free()
            raise MpcgsError(st, msg)
        self.n = len(rows)
        self.nn = 2 * self.n - 1

    def _chk(self, st, what):
        if st:
            raise MpcgsError(st, f"{what}: {lib().mpcgs_last_error(self.h).decode()}")

    def free(self):
        if getattr(self, "h", None):
            lib().mpcgs_free(self.h)
            self.h = None

    def __del__(self):
        try:
            self.free()
        except Exception:
            pass

    def mpcgs_sample(self, n_proposals, n_samples, seed):
        self._chk(lib().mpcgs_sample(self.h, n_proposals, n_samples, seed), "sample")

    def mpcgs_sample_steps(self, n_proposals, n_samples, seed, first_step, last_step=-1):
        """Steps [first_step, last_step) of the mpcgs_sample run (checkpoint / resume)."""
        self._chk(lib().mpcgs_sample_steps(self.h, n_proposals, n_samples, seed, first_step, last_step),
                  "sample_steps")

    def mpcgs_save_state(self):
        """Checkpoint blob of the chain state (bytes)."""
        nb = lib().mpcgs_state_bytes(self.h)
        buf = np.zeros(nb, np.uint8)
        self._chk(lib().mpcgs_save_state(self.h, _ptr(buf), nb), "save_state")
        return buf.tobytes()

    def mpcgs_load_state(self, blob):
        buf = np.frombuffer(blob, dtype=np.uint8).copy()
        self._chk(lib().mpcgs_load_state(self.h, _ptr(buf), buf.size), "load_state")

    def mpcgs_put_samples(self, S, logL, step=None, slot=None):
        """Restore a checkpoint's sample store (step / slot optional)."""
        S = _f64a(S)
        ll = _f64a(logL, S.size)
        st = None if step is None else np.ascontiguousarray(step, dtype=np.int64)
        sl = None if slot is None else np.ascontiguousarray(slot, dtype=np.int32)
        self._chk(lib().mpcgs_put_samples(self.h, S.size, _ptr(S), _ptr(ll), _ptr(st), _ptr(sl)), "put_samples")

    def mpcgs_estimate_theta(self, n_grid=256, curve=False):
        th = ctypes.c_double()
        gt = np.zeros(n_grid)
        gl = np.zeros(n_grid)
        self._chk(lib().mpcgs_estimate_theta(self.h, ctypes.byref(th), n_grid, _ptr(gt), _ptr(gl)),
                  "estimate_theta")
        return (th.value, gt, gl) if curve else th.value

    def mpcgs_log_rel_likelihood(self, theta):
        out = ctypes.c_double()
        self._chk(lib().mpcgs_log_rel_likelihood(self.h, theta, ctypes.byref(out)), "log_rel_likelihood")
        return out.value

    def mpcgs_score_trees(self, parents, ages):
        parents = _i32a(parents).reshape(-1, self.nn)
        ages = _f64a(ages).reshape(-1, self.nn)
        out = np.zeros(parents.shape[0])
        self._chk(lib().mpcgs_score_trees(self.h, parents.shape[0], _ptr(parents), _ptr(ages), _ptr(out)),
                  "score_trees")
        return out

    def mpcgs_set_state(self, parent, age):
        self._chk(lib().mpcgs_set_state(self.h, _ptr(_i32a(parent, self.nn)), _ptr(_f64a(age, self.nn))),
                  "set_state")

    def mpcgs_get_state(self):
        p = np.zeros(self.nn, np.int32)
        a = np.zeros(self.nn)
        ll, S = ctypes.c_double(), ctypes.c_double()
        self._chk(lib().mpcgs_get_state(self.h, _ptr(p), _ptr(a), ctypes.byref(ll), ctypes.byref(S)),
                  "get_state")
        return p, a, ll.value, S.value

    def mpcgs_step_trace(self, step, n_proposals, n_draws, seed):
        N = n_proposals
        tgt = ctypes.c_int32()
        logL, S = np.zeros(N + 1), np.zeros(N + 1)
        t12 = np.zeros(2 * (N + 1))
        pair = np.zeros(N + 1, np.int32)
        draws = np.zeros(n_draws, np.int32)
        self._chk(lib().mpcgs_step_trace(self.h, step, N, n_draws, seed, ctypes.byref(tgt), _ptr(logL),
                                         _ptr(S), _ptr(t12), _ptr(pair), _ptr(draws)), "step_trace")
        return dict(target=tgt.value, logL=logL, S=S, t12=t12.reshape(N + 1, 2), pair=pair, draws=draws)

    def mpcgs_step_local(self, step, n_proposals, seed):
        self._chk(lib().mpcgs_step_local(self.h, step, n_proposals, seed), "step_local")

    def mpcgs_get_records(self, first, count):
        out = np.zeros((count, REC))
        self._chk(lib().mpcgs_get_records(self.h, first, count, _ptr(out)), "get_records")
        return out

    def mpcgs_put_records(self, first, rec):
        rec = _f64a(rec).reshape(-1, REC)
        self._chk(lib().mpcgs_put_records(self.h, first, rec.shape[0], _ptr(rec)), "put_records")

    def mpcgs_step_finish(self, step, n_proposals, n_draws, seed):
        draws = np.zeros(n_draws, np.int32)
        self._chk(lib().mpcgs_step_finish(self.h, step, n_proposals, n_draws, seed, _ptr(draws)),
                  "step_finish")
        return draws

    def mpcgs_num_patterns(self):
        return int(lib().mpcgs_num_patterns(self.h))

    def mpcgs_num_samples(self):
        return int(lib().mpcgs_num_samples(self.h))

    def mpcgs_get_samples(self, first=0, count=None):
        if count is None:
            count = self.mpcgs_num_samples() - first
        S, ll = np.zeros(count), np.zeros(count)
        st, sl = np.zeros(count, np.int64), np.zeros(count, np.int32)
        self._chk(lib().mpcgs_get_samples(self.h, first, count, _ptr(S), _ptr(ll), _ptr(st), _ptr(sl)),
                  "get_samples")
        return dict(S=S, logL=ll, step=st, slot=sl)

    def mpcgs_load_samples(self, S, theta0, logL=None):
        S = _f64a(S)
        ll = None if logL is None else _f64a(logL, S.size)
        self._chk(lib().mpcgs_load_samples(self.h, S.size, _ptr(S), _ptr(ll), float(theta0)), "load_samples")

    def mpcgs_set_theta0(self, theta0):
        self._chk(lib().mpcgs_set_theta0(self.h, theta0), "set_theta0")

    def mpcgs_em(self, n_iter, n_proposals, n_samples, seed, n_grid=256):
        trace = np.zeros(n_iter)
        self._chk(lib().mpcgs_em(self.h, n_iter, n_proposals, n_samples, seed, n_grid, _ptr(trace)), "em")
        return trace

    def mpcgs_get_model(self):
        pi = np.zeros(4)
        mu = ctypes.c_double()
        self._chk(lib().mpcgs_get_model(self.h, _ptr(pi), ctypes.byref(mu)), "get_model")
        return pi, mu.value

    def mpcgs_set_timing(self, mode):
        """mode bit 0: CUDA events per step / kernel; bit 1: 256 MiB L2 flush between steps."""
        self._chk(lib().mpcgs_set_timing(self.h, int(mode) & 3), "set_timing")

    def mpcgs_last_timing_ex(self):
        """{loop, propose, prune, draw} ms of the last device-timed loop, and its launches."""
        ms = np.zeros(4)
        n = ctypes.c_int64()
        self._chk(lib().mpcgs_last_timing_ex(self.h, _ptr(ms), ctypes.byref(n)), "last_timing_ex")
        return dict(loop=ms[0], propose=ms[1], prune=ms[2], draw=ms[3], launches=n.value)

    def mpcgs_last_timing(self):
        a, b, c = ctypes.c_double(), ctypes.c_double(), ctypes.c_int64()
        self._chk(lib().mpcgs_last_timing(self.h, ctypes.byref(a), ctypes.byref(b), ctypes.byref(c)),
                  "last_timing")
        return a.value, b.value, c.value
