"""jp-b200: the Japonica (ICPP'13) loop-mode hot path on B200 (sm_100a).

A thin binding over ``libjp.so`` (C ABI declared in ``include/jp.h``).  Functions
keep the C names; this module only turns torch tensors into device pointers,
the current torch stream into a ``cudaStream_t`` and status codes into
exceptions.  PyTorch is used for device memory, streams and (in ``dist``)
process groups -- every step of the loop runs in the CUDA kernels.
"""
from __future__ import annotations

import ctypes as C
import struct

import torch

from . import _abi
from ._abi import (  # noqa: F401
    JP_I32, JP_F32, JP_OP_ADD_C, JP_OP_SAXPY, JP_OP_PRIV_TMP, JP_OP_STENCIL2,
    JP_MODE_DOALL, JP_MODE_PRIVATIZED, JP_MODE_TLS, JP_MODE_SEQ_RECOMMENDED, MODE_NAMES,
    JP_SCHED_SHARING, JP_SCHED_STEALING, JP_SCHED_AUTO, JP_TLS_RESTART, JP_TLS_ONCHIP, JP_WS_PROFILE, JP_WS_PRIV, JP_WS_TLS, JP_WS_SCHED, JP_WS_GUIDE, JP_WS_ALL,
    REGIONS, JPError, check, lib,
)

__all__ = [
    "Loop", "workspace", "jp_workspace_bytes", "jp_ws_region", "jp_validate", "jp_profile_stamp",
    "jp_profile_classify", "jp_profile_density", "jp_select_mode", "jp_run_doall", "jp_run_privatized",
    "jp_priv_stream", "jp_priv_finalize", "jp_doall_kernel", "jp_tls_guide", "jp_tls_next_window", "jp_run_tls", "jp_schedule", "jp_stage_bytes", "jp_schedule_host",
    "jp_plan_sharing", "jp_plan_stealing", "jp_merge_apply",
    "jp_plan", "jp_plan_tasks", "jp_profile_plan_tasks", "jp_export_keys", "jp_keys_merge_p2p", "jp_priv_inbox_bytes", "jp_priv_stream_merge", "jp_run_priv_claim", "jp_run_doall_spill", "jp_ipc_export", "jp_ipc_import", "jp_ipc_close",
    "jp_sparse_scratch_bytes", "jp_sparse_pack", "jp_sparse_reduce_max", "jp_sparse_gather", "jp_sparse_scatter",
    "jp_last_error", "jp_version", "jp_launch_count", "jp_tls_grid_window",
]

_EL = {JP_I32: torch.int32, JP_F32: torch.float32}


def _ptr(t):
    return None if t is None else t.data_ptr()


_HAS_CUDA = None


def _stream(stream=None):
    """cudaStream_t of `stream`, else torch's current stream (raw accessor: the
    tiny-loop path is launch-latency bound, config 1)."""
    global _HAS_CUDA
    if stream is not None:
        return stream.cuda_stream if hasattr(stream, "cuda_stream") else int(stream)
    if _HAS_CUDA is None:
        _HAS_CUDA = torch.cuda.is_available()
    if _HAS_CUDA:
        return torch._C._cuda_getCurrentRawStream(torch._C._cuda_getDevice())
    return None


class Loop:
    """A loop descriptor over torch tensors (device, or pinned host for jp_schedule_host).

    op/dtype as in jp.h; index tensors are int32 [n] or None (identity);
    A (or Y), X, T are int32/float32 1-D tensors.  The tensors are referenced,
    not copied: the kernels update A (and T) in place."""

    def __init__(self, op, dtype, n, A, r=None, r2=None, w=None, s=None, X=None, T=None, c0=0, c1=0,
                 iter_base=0, ident_off=0):
        el = _EL[dtype]
        for name, t in (("A", A), ("X", X), ("T", T)):
            if t is not None and (t.dtype != el or not t.is_contiguous()):
                raise ValueError(f"{name} must be a contiguous {el} tensor")
        for name, t in (("r", r), ("r2", r2), ("w", w), ("s", s)):
            if t is not None and (t.dtype != torch.int32 or not t.is_contiguous() or t.numel() < n):
                raise ValueError(f"{name} must be a contiguous int32 tensor of >= n entries")
        self.tensors = dict(A=A, r=r, r2=r2, w=w, s=s, X=X, T=T)
        self.op, self.dtype, self.n = int(op), int(dtype), int(n)
        c = _abi.jp_loop()
        c.n, c.iter_base, c.ident_off, c.op, c.dtype = self.n, int(iter_base), int(ident_off), self.op, self.dtype
        self.iter_base, self.ident_off = int(iter_base), int(ident_off)
        c.r, c.r2, c.w, c.s = _ptr(r), _ptr(r2), _ptr(w), _ptr(s)
        c.A, c.len_A = _ptr(A), (0 if A is None else A.numel())
        c.X, c.len_X = _ptr(X), (0 if X is None else X.numel())
        c.T, c.len_T = _ptr(T), (0 if T is None else T.numel())
        self._c0, self._c1 = c0, c1
        for slot, v in (("c0", c0), ("c1", c1)):
            sc = _abi.jp_scalar()
            if dtype == JP_F32:
                sc.f = float(v)
            else:
                sc.i = int(v) - (1 << 32) if int(v) >= (1 << 31) else int(v)
            setattr(c, slot, sc)
        self.c = c

    @classmethod
    def from_workload(cls, wl, iter_base: int = 0, ident_off: int = 0):
        return cls(wl.op, wl.dtype, wl.n, wl.A, r=wl.r, r2=wl.r2, w=wl.w, s=wl.s, X=wl.X, T=wl.T, c0=wl.c0,
                   c1=wl.c1, iter_base=iter_base, ident_off=ident_off)

    def range(self, b: int, e: int) -> "Loop":
        """This loop's iterations [b, e) as a rank-local loop over the same
        (full-size) arrays: iter_base = ident_off = b, index arrays offset."""
        t = self.tensors
        sl = lambda x: None if x is None else x[b:e]  # noqa: E731
        return Loop(self.op, self.dtype, e - b, t["A"], r=sl(t["r"]), r2=sl(t["r2"]), w=sl(t["w"]), s=sl(t["s"]),
                    X=t["X"], T=t["T"], c0=self._c0, c1=self._c1, iter_base=self.iter_base + b,
                    ident_off=self.ident_off + b)

    @property
    def ref(self):
        return C.byref(self.c)


def _prof_dict(p: _abi.jp_profile) -> dict:
    return {k: getattr(p, k) for k, _ in _abi.jp_profile._fields_}


def _prof_struct(p) -> _abi.jp_profile | None:
    if p is None:
        return None
    if isinstance(p, _abi.jp_profile):
        return p
    s = _abi.jp_profile()
    for k, _ in _abi.jp_profile._fields_:
        setattr(s, k, p[k])
    return s


def _pref(p):
    s = _prof_struct(p)
    return None if s is None else C.byref(s)


def jp_workspace_bytes(loop: Loop, uses: int = JP_WS_ALL) -> int:
    return int(lib().jp_workspace_bytes(loop.ref, uses))


def workspace(loop: Loop, uses: int = JP_WS_ALL, device="cuda") -> torch.Tensor:
    """A caller-owned device workspace (torch allocations are >= 256-byte aligned)."""
    return torch.empty(max(jp_workspace_bytes(loop, uses), 256), dtype=torch.uint8, device=device)


def _ws(ws):
    return (None, 0) if ws is None else (ws.data_ptr(), ws.numel())


def jp_ws_region(loop: Loop, region) -> tuple[int, int]:
    rid = REGIONS[region] if isinstance(region, str) else int(region)
    off, nb = C.c_size_t(), C.c_size_t()
    check(lib().jp_ws_region(loop.ref, rid, C.byref(off), C.byref(nb)))
    return off.value, nb.value


def jp_validate(loop: Loop, ws, stream=None) -> int:
    bad = C.c_int64()
    p, nb = _ws(ws)
    st = lib().jp_validate(loop.ref, p, nb, C.byref(bad), _stream(stream))
    if st not in (_abi.JP_OK, _abi.JP_ERR_INDEX):
        check(st)
    return bad.value


def jp_profile_stamp(loop: Loop, ws, stream=None):
    p, nb = _ws(ws)
    check(lib().jp_profile_stamp(loop.ref, p, nb, _stream(stream)))


def jp_profile_classify(loop: Loop, ws, raw_bits=None, chunk_iters=0, chunk_counts=None, stream=None) -> dict:
    out = _abi.jp_profile()
    p, nb = _ws(ws)
    check(lib().jp_profile_classify(loop.ref, p, nb, _ptr(raw_bits), int(chunk_iters), _ptr(chunk_counts),
                                    C.byref(out), _stream(stream)))
    return _prof_dict(out)


def jp_profile_density(loop: Loop, ws, raw_bits=None, chunk_iters=0, chunk_counts=None, stream=None) -> dict:
    out = _abi.jp_profile()
    p, nb = _ws(ws)
    check(lib().jp_profile_density(loop.ref, p, nb, _ptr(raw_bits), int(chunk_iters), _ptr(chunk_counts),
                                   C.byref(out), _stream(stream)))
    return _prof_dict(out)


def jp_select_mode(loop: Loop, prof=None, tau_high: float = _abi.TAU_HIGH) -> int:
    m = lib().jp_select_mode(loop.ref, _pref(prof), float(tau_high))
    if m < 0:
        raise JPError(_abi.JP_ERR_ARG, lib().jp_last_error().decode())
    return m


def jp_static_check(loop: Loop, ws, stream=None) -> dict:
    """Static analysis lite (jp.h): affine index arrays and an exact dependence test."""
    out = _abi.jp_static()
    p, nb = _ws(ws)
    check(lib().jp_static_check(loop.ref, p, nb, C.byref(out), _stream(stream)))
    return {"affine": out.affine, "independent": out.independent, "in_range": out.in_range,
            "alpha": list(out.alpha), "beta": list(out.beta)}


def jp_affine_dependence(af: int, bf: int, ag: int, bg: int, n: int) -> bool:
    """Host-only exact test: some i != j in [0, n) with af*i + bf == ag*j + bg."""
    return bool(lib().jp_affine_dependence(int(af), int(bf), int(ag), int(bg), int(n)))


def jp_run_doall(loop: Loop, prof=None, ws=None, stream=None):
    p, nb = _ws(ws)
    check(lib().jp_run_doall(loop.ref, _pref(prof), p, nb, _stream(stream)))


def jp_run_privatized(loop: Loop, prof=None, ws=None, stream=None):
    p, nb = _ws(ws)
    check(lib().jp_run_privatized(loop.ref, _pref(prof), p, nb, _stream(stream)))


def jp_priv_stream(loop: Loop, prof=None, ws=None, clear_keys=True, stream=None):
    p, nb = _ws(ws)
    check(lib().jp_priv_stream(loop.ref, _pref(prof), p, nb, int(bool(clear_keys)), _stream(stream)))


def jp_priv_finalize(loop: Loop, ws, stream=None):
    p, nb = _ws(ws)
    check(lib().jp_priv_finalize(loop.ref, p, nb, _stream(stream)))


def jp_doall_kernel(which: int = -1) -> int:
    """Affine DOALL kernel choice: 0 LDG/STG.128 stream, 1 bulk-copy (TMA) staged; -1 queries."""
    return int(lib().jp_doall_kernel(int(which)))


def jp_tls_next_window(n: int, prof_raw_iters: int, prev_commit: int = -1, w_max: int = 4096) -> int:
    """Reading A8's window policy, computed by the library (jp.h)."""
    return int(lib().jp_tls_next_window(int(n), int(prof_raw_iters), int(prev_commit), int(w_max)))


def jp_tls_guide(loop: Loop, ws: torch.Tensor, stream=None) -> None:
    """Guide bitmaps (region 13) from a profile already run on `ws` (jp.h)."""
    p, nb = _ws(ws)
    check(lib().jp_tls_guide(loop.ref, p, nb, _stream(stream)))


def jp_run_tls(loop: Loop, window=0, w_max=65536, path=0, prof=None, ws=None, stats=True, stream=None, cluster=0,
               guided=False, recovery=0):
    """recovery: JP_TLS_RESTART (0, reading A6) or JP_TLS_ONCHIP (1, reading B7)."""
    cfg = _abi.jp_tls_cfg(int(window), int(w_max), int(path), int(cluster), int(bool(guided)), int(recovery))
    st = _abi.jp_tls_stats()
    p, nb = _ws(ws)
    check(lib().jp_run_tls(loop.ref, C.byref(cfg), _pref(prof), p, nb, C.byref(st) if stats else None,
                           _stream(stream)))
    return {k: getattr(st, k) for k, _ in _abi.jp_tls_stats._fields_} if stats else None


def sched_cfg(scheme=JP_SCHED_SHARING, tau_high=_abi.TAU_HIGH, chunk_iters=65536, tls_window=0, tls_w_max=0,
              tls_path=0, tls_recovery=0, static_check=0) -> _abi.jp_sched_cfg:
    """tls_recovery: 0 auto (on chip when the profile shows waw_iters == 0), 1 restart, 2 on chip.
    static_check: 0 run jp_static_check before profiling, 1 skip it."""
    return _abi.jp_sched_cfg(int(scheme), int(tls_path), float(tau_high), int(chunk_iters), int(tls_window),
                             int(tls_w_max), int(tls_recovery), int(static_check))


# jp_sched_result unpacked in one call (field order and natural alignment of jp.h)
_RES_FMT = struct.Struct("=ii5q3d4qqq4qq4i")
assert _RES_FMT.size == C.sizeof(_abi.jp_sched_result)


def _res_dict(r: _abi.jp_sched_result) -> dict:
    (mode, profiled, n, raw, war, waw, first, d_raw, d_war, d_waw, com, exe, win, vio, n_tasks, n_batches,
     m0, m1, m2, m3, wmax, path, guided, rec, cl) = _RES_FMT.unpack(bytes(r))
    return {"mode": mode, "mode_name": MODE_NAMES.get(mode, "?"), "profiled": profiled,
            "prof": {"n": n, "raw_iters": raw, "war_iters": war, "waw_iters": waw, "first_raw_iter": first,
                     "d_raw": d_raw, "d_war": d_war, "d_waw": d_waw},
            "tls": {"committed": com, "executed": exe, "windows": win, "violations": vio},
            "n_tasks": n_tasks, "n_batches": n_batches, "task_mode_iters": [m0, m1, m2, m3],
            "tls_w_max": wmax, "tls_path": path, "tls_guided": guided, "tls_recovery": rec, "tls_cluster": cl}


_DEFAULT_CFG = None


def jp_schedule(loop: Loop, ws=None, cfg=None, stream=None, **kw) -> dict:
    global _DEFAULT_CFG
    if cfg is None:
        if kw:
            cfg = sched_cfg(**kw)
        else:   # the C call only reads it (const jp_sched_cfg *): one shared default
            if _DEFAULT_CFG is None:
                _DEFAULT_CFG = sched_cfg()
            cfg = _DEFAULT_CFG
    res = _abi.jp_sched_result()
    p, nb = _ws(ws)
    check(lib().jp_schedule(loop.ref, C.byref(cfg), p, nb, C.byref(res), _stream(stream)))
    return _res_dict(res)


def _plan_dict(p: _abi.jp_workflow_plan, n: int) -> dict:
    return {"scheme": p.scheme, "n_batches": p.n_batches, "batch": list(p.batch[:n]), "deps": list(p.deps[:n])}


def jp_plan_workflow(loops, scheme=JP_SCHED_AUTO) -> dict:
    """PDG batches of a workflow of loops (host only; readings B9, B10)."""
    arr = (_abi.jp_loop * max(len(loops), 1))(*[lp.c for lp in loops])
    out = _abi.jp_workflow_plan()
    check(lib().jp_plan_workflow(arr, len(loops), int(scheme), C.byref(out)))
    return _plan_dict(out, len(loops))


def jp_schedule_workflow(loops, wss=None, cfg=None, stream=None, **kw):
    """Run a workflow (list of Loop) with one workspace per loop; returns (results, plan)."""
    cfg = cfg if cfg is not None else sched_cfg(**kw)
    n = len(loops)
    arr = (_abi.jp_loop * max(n, 1))(*[lp.c for lp in loops])
    wss = wss if wss is not None else [None] * n
    wp = (C.c_void_p * max(n, 1))(*[None if w is None else w.data_ptr() for w in wss])
    wb = (C.c_size_t * max(n, 1))(*[0 if w is None else w.numel() for w in wss])
    res = (_abi.jp_sched_result * max(n, 1))()
    plan = _abi.jp_workflow_plan()
    check(lib().jp_schedule_workflow(arr, n, C.byref(cfg), wp, wb, res, C.byref(plan), _stream(stream)))
    return [_res_dict(res[u]) for u in range(n)], _plan_dict(plan, n)


def jp_stage_bytes(loop: Loop) -> int:
    return int(lib().jp_stage_bytes(loop.ref))


def jp_schedule_host(loop: Loop, stage, ws=None, cfg=None, stream=None, **kw) -> dict:
    """loop's tensors live on the HOST (pinned); stage/ws are device buffers."""
    cfg = cfg if cfg is not None else sched_cfg(**kw)
    res = _abi.jp_sched_result()
    p, nb = _ws(ws)
    check(lib().jp_schedule_host(loop.ref, C.byref(cfg), stage.data_ptr(), stage.numel(), p, nb, C.byref(res),
                                 _stream(stream)))
    return _res_dict(res)


def jp_plan_sharing(n: int, world: int, weights=None) -> list[tuple[int, int]]:
    rg = (C.c_int64 * (2 * world))()
    wt = None if weights is None else (C.c_double * world)(*[float(x) for x in weights])
    check(lib().jp_plan_sharing(int(n), int(world), wt, rg))
    return [(rg[2 * k], rg[2 * k + 1]) for k in range(world)]


def jp_plan_stealing(tasks, world: int, chunk_iters: int, speed=None, speed_tls: float = 1.0):
    """tasks: [(start, end, mode)].  Returns (chunks [(start, end, mode, owner)], n_stolen)."""
    flat = [int(v) for t in tasks for v in t]
    tk = (C.c_int64 * max(len(flat), 1))(*flat)
    cap = sum(max(1, -(-(e - s) // chunk_iters)) for s, e, _ in tasks) + len(tasks) + 1
    out = (C.c_int64 * (4 * cap))()
    n_out, stolen = C.c_int64(), C.c_int64()
    sp = None if speed is None else (C.c_double * world)(*[float(x) for x in speed])
    check(lib().jp_plan_stealing(tk, len(tasks), int(world), int(chunk_iters), sp, float(speed_tls), out, cap,
                                 C.byref(n_out), C.byref(stolen)))
    return [tuple(out[4 * c:4 * c + 4]) for c in range(n_out.value)], stolen.value


def jp_merge_apply(arr: torch.Tensor, keys: torch.Tensor, stream=None):
    check(lib().jp_merge_apply(arr.data_ptr(), arr.numel(), keys.data_ptr(), _stream(stream)))


# ---- task stealing across ranks (jp.h) -------------------------------------
def jp_plan(loop: Loop, chunk_profiles, world: int, speed=None, cfg=None, **kw):
    """Host-only split plan (jp.h jp_plan): chunk_profiles = list of dicts (or
    jp_profile) of the whole loop's chunks -> [(start, end, mode, owner)]."""
    cfg = cfg if cfg is not None else sched_cfg(**kw)
    arr = (_abi.jp_profile * max(len(chunk_profiles), 1))(*[_prof_struct(p) for p in chunk_profiles])
    cap = 4 * (len(chunk_profiles) + world) + 8
    out = (C.c_int64 * (4 * cap))()
    n = C.c_int64()
    sp = None if speed is None else (C.c_double * world)(*[float(x) for x in speed])
    check(lib().jp_plan(loop.ref, C.byref(cfg), arr, len(chunk_profiles), int(world), sp, out, cap, C.byref(n)))
    return [tuple(out[4 * k:4 * k + 4]) for k in range(n.value)]


def jp_plan_tasks(loop: Loop, chunk_counts, chunk_iters: int, ws, tau_high: float = _abi.TAU_HIGH, stream=None):
    """chunk_counts: the whole loop's (raw, war, waw) per chunk (flat list / int64
    tensor).  Returns ([(start, end, mode)], conf list of 64 ints)."""
    cc = [int(x) for x in (chunk_counts.tolist() if hasattr(chunk_counts, "tolist") else chunk_counts)]
    hc = (C.c_int64 * max(len(cc), 1))(*cc)
    tk = (C.c_int64 * 192)()
    nt = C.c_int32()
    cf = (C.c_uint64 * 64)()
    p, nb = _ws(ws)
    check(lib().jp_plan_tasks(loop.ref, hc, int(chunk_iters), float(tau_high), p, nb, tk, C.byref(nt), cf,
                              _stream(stream)))
    return [(tk[3 * t], tk[3 * t + 1], tk[3 * t + 2]) for t in range(nt.value)], list(cf)


def jp_profile_plan_tasks(loop: Loop, chunk_iters: int, ws, tau_high: float = _abi.TAU_HIGH, stream=None):
    """The whole loop's profile (this rank's own, no exchange) with per-chunk
    counts, then the task plan.  Returns (profile dict, chunk counts list,
    [(start, end, mode)], conf list of 64 ints)."""
    nck = -(-loop.n // int(chunk_iters))
    pr = _abi.jp_profile()
    hc = (C.c_int64 * max(3 * nck, 1))()
    tk = (C.c_int64 * 192)()
    nt = C.c_int32()
    cf = (C.c_uint64 * 64)()
    p, nb = _ws(ws)
    check(lib().jp_profile_plan_tasks(loop.ref, int(chunk_iters), float(tau_high), p, nb, C.byref(pr), hc, tk,
                                      C.byref(nt), cf, _stream(stream)))
    return (_prof_dict(pr), list(hc[:3 * nck]), [(tk[3 * t], tk[3 * t + 1], tk[3 * t + 2]) for t in range(nt.value)],
            list(cf))


def jp_export_keys(loop: Loop, ws, stream=None):
    p, nb = _ws(ws)
    check(lib().jp_export_keys(loop.ref, p, nb, _stream(stream)))


# ---- task sharing with cross-boundary spill (jp.h, M1 / C8) --------------
def jp_run_doall_spill(views, me: int, chunk: int, ctr: torch.Tensor, stats=None, max_ctas: int = 0, stream=None):
    """views: every rank's affine shard (Loop or jp_loop with pointers valid here);
    ctr: int64 [world] device counters, zero before any rank starts; stats:
    int64 [3] device accumulator (own iters, stolen iters, stolen chunks)."""
    cs = [v.c if isinstance(v, Loop) else v for v in views]
    arr = (_abi.jp_loop * len(cs))(*cs)
    check(lib().jp_run_doall_spill(arr, len(cs), int(me), int(chunk), ctr.data_ptr(), _ptr(stats), int(max_ctas),
                                   _stream(stream)))


def jp_run_priv_claim(loop: Loop, chunks: torch.Tensor, first, me: int, ctr, ws, stats=None, max_ctas: int = 0,
                      stream=None):
    """chunks: int64 device tensor [m, 2] of (start, end); first: world+1 ints."""
    fl = (C.c_int64 * len(first))(*[int(x) for x in first])
    p, nb = _ws(ws)
    check(lib().jp_run_priv_claim(loop.ref, chunks.data_ptr() if chunks.numel() else None, fl, len(first) - 1, int(me),
                                  ctr.data_ptr(), _ptr(stats), p, nb, int(max_ctas), _stream(stream)))


def jp_keys_merge_p2p(peer_ptrs, keys: torch.Tensor, bar, epoch: int, err: torch.Tensor, arr=None, stream=None):
    """peer_ptrs: every rank's key-table device pointer (ints, this rank's
    included); bar: the shared counter (tensor or object with data_ptr())."""
    pp = (C.c_void_p * len(peer_ptrs))(*[int(p) for p in peer_ptrs])
    check(lib().jp_keys_merge_p2p(pp, len(peer_ptrs), keys.data_ptr(), keys.numel(), bar.data_ptr(), int(epoch),
                                  _ptr(arr), err.data_ptr(), _stream(stream)))


def jp_priv_inbox_bytes(loop: Loop, world: int) -> int:
    return int(lib().jp_priv_inbox_bytes(loop.ref, int(world)))


def jp_priv_stream_merge(loop: Loop, ws, inbox_ptrs, me: int, err: torch.Tensor, prof=None, stream=None):
    """inbox_ptrs: every rank's inbox pointer as mapped here (ints, own included)."""
    pp = (C.c_void_p * len(inbox_ptrs))(*[int(p) for p in inbox_ptrs])
    p, nb = _ws(ws)
    check(lib().jp_priv_stream_merge(loop.ref, _pref(prof), p, nb, pp, len(inbox_ptrs), int(me), err.data_ptr(),
                                     _stream(stream)))


def jp_ipc_export(t: torch.Tensor) -> tuple[bytes, int]:
    h = C.create_string_buffer(64)
    off = C.c_int64()
    check(lib().jp_ipc_export(t.data_ptr(), h, C.byref(off)))
    return h.raw, off.value


def jp_ipc_import(handle: bytes, offset: int) -> int:
    p = C.c_void_p()
    check(lib().jp_ipc_import(C.create_string_buffer(handle, 64), int(offset), C.byref(p)))
    return int(p.value)


def jp_ipc_close(ptr: int, offset: int):
    check(lib().jp_ipc_close(C.c_void_p(ptr), int(offset)))


# ---- owner-partitioned sparse exchange (jp.h, NEXT-2) ----------------------
def _tables(t0, t1):
    if t0.dtype not in (torch.int32, torch.int64) or (t1 is not None and (t1.dtype != t0.dtype
                                                                         or t1.numel() != t0.numel())):
        raise ValueError("sparse tables: one or two int32 / int64 tensors of the same length")
    return t0.element_size(), t0.numel(), 2 + (t1 is not None)   # row width: address + values


def jp_sparse_scratch_bytes(length: int, world: int) -> int:
    return int(lib().jp_sparse_scratch_bytes(int(length), int(world)))


def jp_sparse_pack(t0: torch.Tensor, t1=None, empty: int = -1, world: int = 1, lo: int = 0, hi=None, stream=None):
    """Rows [m, 1 + ntab] (t0's dtype; column 0 the address) of the entries of
    [lo, hi) where a table is not ``empty``, sorted by address, and the per-owner
    row counts (list of ``world`` ints)."""
    eb, n, w = _tables(t0, t1)
    hi = n if hi is None else int(hi)
    cap = max(hi - int(lo), 0)
    rows = torch.empty((max(cap, 1), w), dtype=t0.dtype, device=t0.device)
    scratch = torch.empty(max(jp_sparse_scratch_bytes(n, world) // 8, 1), dtype=torch.int64, device=t0.device)
    counts = (C.c_int64 * int(world))()
    check(lib().jp_sparse_pack(t0.data_ptr(), _ptr(t1), eb, n, int(lo), hi, int(empty), int(world), rows.data_ptr(),
                               cap, counts, scratch.data_ptr(), scratch.numel() * 8, _stream(stream)))
    cl = list(counts)
    return rows[:sum(cl)], cl


def jp_sparse_reduce_max(t0: torch.Tensor, t1, rows: torch.Tensor, stream=None):
    eb, n, _ = _tables(t0, t1)
    check(lib().jp_sparse_reduce_max(t0.data_ptr(), _ptr(t1), eb, n, rows.data_ptr(), rows.shape[0], _stream(stream)))


def jp_sparse_gather(t0: torch.Tensor, t1, rows: torch.Tensor, stream=None):
    eb, n, _ = _tables(t0, t1)
    check(lib().jp_sparse_gather(t0.data_ptr(), _ptr(t1), eb, n, rows.data_ptr(), rows.shape[0], _stream(stream)))


def jp_sparse_scatter(t0: torch.Tensor, t1, rows: torch.Tensor, stream=None):
    eb, n, _ = _tables(t0, t1)
    check(lib().jp_sparse_scatter(t0.data_ptr(), _ptr(t1), eb, n, rows.data_ptr(), rows.shape[0], _stream(stream)))


def jp_last_error() -> str:
    return lib().jp_last_error().decode()


def jp_version() -> str:
    return lib().jp_version().decode()


def jp_launch_count() -> int:
    return int(lib().jp_launch_count())


def jp_tls_grid_window() -> int:
    return int(lib().jp_tls_grid_window())
