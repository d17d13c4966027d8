"""TEST INFRASTRUCTURE ONLY -- ctypes wrapper around ``oracle/liboracle.so``.

The C file ``oracle/jpo.c`` is the oracle; this module only marshals numpy
arrays in and out of it (no arithmetic of the method lives here).
"""
from __future__ import annotations

import ctypes as C
import os
import subprocess
import threading

import numpy as np

OP_ADD_C, OP_SAXPY, OP_PRIV_TMP, OP_STENCIL2 = 0, 1, 2, 3
I32, F32 = 0, 1
OK, ERR_ARG, ERR_INDEX = 0, -1, -5

_HERE = os.path.dirname(os.path.abspath(__file__))
_SO = os.path.join(_HERE, "liboracle.so")
_lock = threading.Lock()
_lib = None


def build(force: bool = False) -> str:
    """Compile the C oracle (gcc, -ffp-contract=off).  Returns the .so path."""
    src = [os.path.join(_HERE, f) for f in ("jpo.c", "jpo.h")]
    stale = (not os.path.exists(_SO)) or any(os.path.getmtime(s) > os.path.getmtime(_SO) for s in src)
    if force or stale:
        subprocess.check_call(["make", "-s", "-C", _HERE, "liboracle.so"] + (["-B"] if force else []))
    return _SO


class _Loop(C.Structure):
    _fields_ = [
        ("n", C.c_int64), ("op", C.c_int32), ("dtype", C.c_int32),
        ("r", C.c_void_p), ("r2", C.c_void_p), ("w", C.c_void_p), ("s", C.c_void_p),
        ("A", C.c_void_p), ("len_A", C.c_int64),
        ("X", C.c_void_p), ("len_X", C.c_int64),
        ("T", C.c_void_p), ("len_T", C.c_int64),
        ("c0", C.c_uint32), ("c1", C.c_uint32),
    ]


class _Profile(C.Structure):
    _fields_ = [(k, C.c_int64) for k in ("n", "raw_iters", "war_iters", "waw_iters", "first_raw_iter",
                                          "raw_pairs", "war_pairs", "waw_pairs")]


class _TlsStats(C.Structure):
    _fields_ = [(k, C.c_int64) for k in ("committed", "executed", "windows", "violations")]


def _load():
    global _lib
    with _lock:
        if _lib is None:
            lib = C.CDLL(build())
            P = C.POINTER
            lib.jpo_run_seq.argtypes = [P(_Loop)]
            lib.jpo_run_order.argtypes = [P(_Loop), C.c_void_p]
            lib.jpo_profile_run.argtypes = [P(_Loop), P(_Profile), C.c_void_p]
            lib.jpo_pairs.argtypes = [P(_Loop), P(_Profile), C.c_void_p]
            lib.jpo_raw_sources.argtypes = [P(_Loop), C.c_void_p]
            lib.jpo_sim_tls.argtypes = [P(_Loop), C.c_int64, C.c_int64, C.c_int64, P(_TlsStats)]
            lib.jpo_sim_tls_fwd.argtypes = [P(_Loop), C.c_int64, P(_TlsStats)]
            lib.jpo_tls_next_window.argtypes = [C.c_int64] * 4
            lib.jpo_tls_next_window.restype = C.c_int64
            lib.jpo_sim_priv.argtypes = [P(_Loop)]
            _lib = lib
    return _lib


def _bits(v, dtype) -> int:
    if dtype == F32:
        if isinstance(v, (np.floating, float)):
            return int(np.float32(v).view(np.uint32))
        return int(v) & 0xFFFFFFFF
    return int(v) & 0xFFFFFFFF


class Loop:
    """A loop descriptor over private numpy copies (inputs are never mutated)."""

    def __init__(self, op, dtype, n, A, r=None, r2=None, w=None, s=None, X=None, T=None, c0=0, c1=0):
        el = np.int32 if dtype == I32 else np.float32
        self.op, self.dtype, self.n = int(op), int(dtype), int(n)
        self.A = np.ascontiguousarray(A, dtype=el).copy()
        self.X = None if X is None else np.ascontiguousarray(X, dtype=el).copy()
        self.T = None if T is None else np.ascontiguousarray(T, dtype=el).copy()
        self.r, self.r2, self.w, self.s = (None if v is None else np.ascontiguousarray(v, dtype=np.int32)
                                           for v in (r, r2, w, s))
        self.c0, self.c1 = _bits(c0, dtype), _bits(c1, dtype)

    def copy(self) -> "Loop":
        L = Loop.__new__(Loop)
        L.__dict__.update({k: (v.copy() if isinstance(v, np.ndarray) else v) for k, v in self.__dict__.items()})
        return L

    def _c(self) -> _Loop:
        p = lambda a: None if a is None else a.ctypes.data  # noqa: E731
        ln = lambda a: 0 if a is None else a.size  # noqa: E731
        return _Loop(self.n, self.op, self.dtype, p(self.r), p(self.r2), p(self.w), p(self.s),
                     p(self.A), ln(self.A), p(self.X), ln(self.X), p(self.T), ln(self.T), self.c0, self.c1)


def run_seq(loop: Loop):
    """Sequential definition.  Returns (status, A', T') on copies."""
    L = loop.copy()
    st = _load().jpo_run_seq(C.byref(L._c()))
    return st, L.A, L.T


def run_seq_inplace(loop: Loop) -> int:
    """Sequential definition on the loop's own arrays (no copy; used for timing)."""
    return _load().jpo_run_seq(C.byref(loop._c()))


def run_order(loop: Loop, perm):
    L = loop.copy()
    perm = np.ascontiguousarray(perm, dtype=np.int64)
    st = _load().jpo_run_order(C.byref(L._c()), perm.ctypes.data)
    return st, L.A, L.T


def _prof(fn, loop: Loop):
    out = _Profile()
    flags = np.zeros(max(loop.n, 1), dtype=np.uint8)
    st = fn(C.byref(loop._c()), C.byref(out), flags.ctypes.data)
    d = {k: getattr(out, k) for k, _ in _Profile._fields_}
    d["status"] = st
    d["flags"] = flags[: loop.n]
    return d


def profile(loop: Loop) -> dict:
    """Single-pass density profile (reading A1).  flags bit0 raw, bit1 war, bit2 waw."""
    return _prof(_load().jpo_profile_run, loop)


def pairs(loop: Loop) -> dict:
    """O(n^2) pair enumeration (brute force)."""
    return _prof(_load().jpo_pairs, loop)


def raw_sources(loop: Loop) -> np.ndarray:
    """src[j] = 1 iff a write of j is an exposed read of a later iteration."""
    src = np.zeros(max(loop.n, 1), dtype=np.uint8)
    st = _load().jpo_raw_sources(C.byref(loop._c()), src.ctypes.data)
    if st != OK:
        raise ValueError(f"jpo_raw_sources: status {st}")
    return src[: loop.n]


def sim_tls(loop: Loop, window: int, w_max: int = 65536, prof_raw_iters: int = -1):
    """Windowed TLS definition. Returns (status, A', T', stats dict)."""
    L = loop.copy()
    st = _TlsStats()
    s = _load().jpo_sim_tls(C.byref(L._c()), int(window), int(w_max), int(prof_raw_iters), C.byref(st))
    return s, L.A, L.T, {k: getattr(st, k) for k, _ in _TlsStats._fields_}


def sim_tls_fwd(loop: Loop, window: int):
    """Windowed TLS with on-chip recovery (reading B7). Returns (status, A', T', stats dict)."""
    L = loop.copy()
    st = _TlsStats()
    s = _load().jpo_sim_tls_fwd(C.byref(L._c()), int(window), C.byref(st))
    return s, L.A, L.T, {k: getattr(st, k) for k, _ in _TlsStats._fields_}


def tls_next_window(n: int, prof_raw_iters: int, prev_commit: int, w_max: int = 65536) -> int:
    return int(_load().jpo_tls_next_window(int(n), int(prof_raw_iters), int(prev_commit), int(w_max)))


def sim_priv(loop: Loop):
    L = loop.copy()
    st = _load().jpo_sim_priv(C.byref(L._c()))
    return st, L.A, L.T
