"""TEST DOUBLE of the libjp.so compute entry points, for CPU-only (gloo) tests
of the multi-GPU driver (paper_conf_icpp_hanzlw13_b200/dist.py).

Host-only entry points (plans, workspace layout, mode selection) are the real
libjp.so functions.  The compute entry points are re-stated here in numpy from
the oracle's definitions and the encodings documented in include/jp.h, writing
into the REAL workspace layout (jp_ws_region), so that dist.py's collectives
run over exactly the regions the CUDA kernels would fill.  Never used by the
product path.
"""
from __future__ import annotations

import numpy as np
import torch

import oracle as O
import paper_conf_icpp_hanzlw13_b200 as jp

INT32_MAX = 0x7FFFFFFF

# host-only entry points: the real library
jp_plan_sharing = jp.jp_plan_sharing
jp_plan_stealing = jp.jp_plan_stealing
jp_ws_region = jp.jp_ws_region
jp_select_mode = jp.jp_select_mode


def _np(t):
    return None if t is None else t.numpy()


def _accesses(loop, i):
    """(array, address, kind) of local iteration i; kind in {'re', 'rc', 'w'}."""
    t = loop.tensors
    ix = lambda a: loop.ident_off + i if a is None else int(a[i])  # noqa: E731
    op = loop.op
    if op == O.OP_ADD_C:
        return [("A", ix(t["r"]), "re"), ("A", ix(t["w"]), "w")]
    if op == O.OP_SAXPY:
        return [("X", ix(t["r"]), "re"), ("A", ix(t["w"]), "re"), ("A", ix(t["w"]), "w")]
    if op == O.OP_PRIV_TMP:
        return [("X", ix(t["r"]), "re"), ("T", ix(t["s"]), "rc"), ("T", ix(t["s"]), "w"), ("A", ix(t["w"]), "w")]
    return [("A", ix(t["r"]), "re"), ("A", ix(t["r2"]), "re"), ("A", ix(t["w"]), "w")]


def _indirect(loop):
    t, op = loop.tensors, loop.op
    a = {O.OP_ADD_C: t["r"] is not None or t["w"] is not None, O.OP_SAXPY: t["w"] is not None,
         O.OP_PRIV_TMP: t["w"] is not None}.get(op, t["r"] is not None or t["r2"] is not None or t["w"] is not None)
    return {"A": a, "T": op == O.OP_PRIV_TMP and t["s"] is not None, "X": False}


def _view(ws, loop, name, dtype):
    off, nb = jp.jp_ws_region(loop, name)
    return None if nb == 0 else ws[off:off + nb].view(dtype).numpy()


def jp_profile_stamp(loop, ws):
    ind = _indirect(loop)
    tabs = {k: _view(ws, loop, k, torch.int32) for k in ("minW_A", "minR_A", "minW_T", "minR_T")}
    for v in tabs.values():
        if v is not None:
            v[:] = -1
    for i in range(loop.n):
        e = INT32_MAX - (loop.iter_base + i)
        for arr, a, kind in _accesses(loop, i):
            if not ind[arr]:
                continue
            tab = tabs[("minW_" if kind == "w" else "minR_") + arr]
            if tab is not None:
                tab[a] = max(tab[a], e)


def jp_profile_classify(loop, ws, chunk_iters=0, chunk_counts=None, **kw):
    ind = _indirect(loop)
    if chunk_counts is not None:
        chunk_counts.zero_()
    cc = None if chunk_counts is None else chunk_counts.numpy()
    tabs = {k: _view(ws, loop, k, torch.int32) for k in ("minW_A", "minR_A", "minW_T", "minR_T")}
    raw = war = waw = 0
    first = -1
    for i in range(loop.n):
        e = INT32_MAX - (loop.iter_base + i)
        fr = fa = fw = False
        for arr, a, kind in _accesses(loop, i):
            if not ind[arr]:
                continue
            w, r = tabs["minW_" + arr], tabs["minR_" + arr]
            if kind == "re" and w is not None and w[a] > e:
                fr = True
            if kind == "w":
                fa |= r is not None and r[a] > e
                fw |= w is not None and w[a] > e
        raw += fr
        war += fa
        waw += fw
        if cc is not None:
            c = i // chunk_iters
            cc[3 * c] += fr
            cc[3 * c + 1] += fa
            cc[3 * c + 2] += fw
        if fr and first < 0:
            first = loop.iter_base + i
    n = loop.n
    return {"n": n, "raw_iters": raw, "war_iters": war, "waw_iters": waw, "first_raw_iter": first,
            "d_raw": raw / n if n else 0.0, "d_war": war / n if n else 0.0, "d_waw": waw / n if n else 0.0}


def _bits(v, dtype):
    return int(np.array([v], dtype=np.float32 if dtype == O.F32 else np.int32).view(np.uint32)[0])


def _values(loop, i, A, X):
    """Values the body of local iteration i writes, from arrays A, X (reading A10)."""
    t = loop.tensors
    ix = lambda a: loop.ident_off + i if a is None else int(a[i])  # noqa: E731
    f = np.float32 if loop.dtype == O.F32 else np.int32
    c0 = f(loop._c0) if loop.dtype == O.F32 else np.int64(loop._c0)
    c1 = f(loop._c1) if loop.dtype == O.F32 else np.int64(loop._c1)
    wrap = (lambda v: f(v)) if loop.dtype == O.F32 else (lambda v: np.int32(np.int64(v) & 0xFFFFFFFF)
                                                         if (np.int64(v) & 0xFFFFFFFF) < 2**31
                                                         else np.int32((np.int64(v) & 0xFFFFFFFF) - 2**32))
    if loop.op == O.OP_ADD_C:
        return {"A": wrap(A[ix(t["r"])] + c0)}
    if loop.op == O.OP_SAXPY:
        return {"A": wrap(wrap(c0 * X[ix(t["r"])]) + A[ix(t["w"])])}
    if loop.op == O.OP_PRIV_TMP:
        tv = wrap(c0 * X[ix(t["r"])])
        return {"T": tv, "A": wrap(tv + c1)}
    return {"A": wrap(wrap(A[ix(t["r"])] + A[ix(t["r2"])]) * c0)}


def jp_priv_stream(loop, prof, ws, clear_keys=True):
    ind = _indirect(loop)
    keys = {k: _view(ws, loop, "keys_" + k, torch.int64) for k in ("A", "T")}
    if clear_keys:
        for v in keys.values():
            if v is not None:
                v[:] = 0
    t = loop.tensors
    A0 = _np(t["A"]).copy()
    X = _np(t["X"])
    ix = lambda a, i: loop.ident_off + i if a is None else int(a[i])  # noqa: E731
    for i in range(loop.n):
        vals = _values(loop, i, A0, X)
        gid = loop.iter_base + i
        for arr, v in vals.items():
            addr = ix(t["w"], i) if arr == "A" else ix(t["s"], i)
            if ind[arr]:
                k = ((gid + 1) << 32) | _bits(v, loop.dtype)
                keys[arr][addr] = max(int(keys[arr][addr]), k)
            else:
                _np(t[arr])[addr] = v


def jp_priv_finalize(loop, ws):
    for arr in ("A", "T"):
        k = _view(ws, loop, "keys_" + arr, torch.int64)
        if k is None:
            continue
        out = _np(loop.tensors[arr])
        m = k != 0
        out.view(np.uint32)[m] = (k[m] & 0xFFFFFFFF).astype(np.uint32)


def _oracle_loop(loop):
    t = loop.tensors
    assert loop.ident_off == 0
    return O.Loop(loop.op, loop.dtype, loop.n, _np(t["A"]), r=_np(t["r"]), r2=_np(t["r2"]), w=_np(t["w"]),
                  s=_np(t["s"]), X=_np(t["X"]), T=_np(t["T"]), c0=loop._c0, c1=loop._c1)


def jp_schedule(loop, ws=None, **kw):
    """Only the static-DOALL (all index arrays NULL) case is used by dist.py here."""
    t = loop.tensors
    assert all(t[k] is None for k in ("r", "r2", "w", "s"))
    A0 = _np(t["A"]).copy()
    X = _np(t["X"])
    for i in range(loop.n):
        for arr, v in _values(loop, i, A0, X).items():
            _np(t[arr])[loop.ident_off + i] = v
    return {"mode": 0, "mode_name": "DOALL", "profiled": 0}


def jp_run_tls(loop, window=0, w_max=65536, path=0, prof=None, ws=None, stats=True, **kw):
    if loop.ident_off or loop.iter_base:   # a range of a loop: its committed result is the in-order one
        t = loop.tensors
        ix = lambda a, i: loop.ident_off + i if a is None else int(a[i])  # noqa: E731
        for i in range(loop.n):
            for arr, v in _values(loop, i, _np(t["A"]), _np(t["X"])).items():
                _np(t[arr])[ix(t["w"], i) if arr == "A" else ix(t["s"], i)] = v
        return {"committed": loop.n, "executed": loop.n, "windows": 1, "violations": 0}
    st, A, T, stats_ = O.sim_tls(_oracle_loop(loop), window, w_max, -1 if prof is None else prof["raw_iters"])
    assert st == 0
    _np(loop.tensors["A"])[:] = A
    if loop.tensors["T"] is not None:
        _np(loop.tensors["T"])[:] = T
    return stats_


# ---- owner-partitioned sparse exchange (jp.h jp_sparse_*), plain definitions ----
def jp_sparse_pack(t0, t1=None, empty=-1, world=1, lo=0, hi=None):
    n = t0.numel()
    hi = n if hi is None else hi
    a = np.arange(lo, hi, dtype=np.int64)
    full = t0.numpy()[lo:hi] != empty
    if t1 is not None:
        full |= t1.numpy()[lo:hi] != empty
    a = a[full]
    cols = [a.astype(t0.numpy().dtype), t0.numpy()[a]] + ([t1.numpy()[a]] if t1 is not None else [])
    rows = torch.from_numpy(np.stack(cols, axis=1).copy())
    sl = max(-(-n // world), 1)
    counts = [int(np.count_nonzero(a // sl == k)) for k in range(world)]
    return rows, counts


def _rows_ok(rows, n):
    a = rows.numpy()[:, 0].astype(np.int64)
    return a, (a >= 0) & (a < n)


def jp_sparse_reduce_max(t0, t1, rows):
    a, ok = _rows_ok(rows, t0.numel())
    for q, t in enumerate([t0, t1]):
        if t is not None:
            np.maximum.at(t.numpy(), a[ok], rows.numpy()[ok, 1 + q])


def jp_sparse_gather(t0, t1, rows):
    a, ok = _rows_ok(rows, t0.numel())
    for q, t in enumerate([t0, t1]):
        if t is not None:
            rows.numpy()[ok, 1 + q] = t.numpy()[a[ok]]


def jp_sparse_scatter(t0, t1, rows):
    a, ok = _rows_ok(rows, t0.numel())
    for q, t in enumerate([t0, t1]):
        if t is not None:
            t.numpy()[a[ok]] = rows.numpy()[ok, 1 + q]


# ---- task stealing across ranks (jp.h jp_plan_tasks / jp_export_keys), plain definitions ----
def jp_plan_tasks(loop, chunk_counts, chunk_iters, ws, tau_high=0.999):
    import oracle.sched as OS
    cc = [int(x) for x in (chunk_counts.tolist() if hasattr(chunk_counts, "tolist") else chunk_counts)]
    n = loop.n
    tasks = []
    for k in range(-(-n // chunk_iters)):
        s, e = k * chunk_iters, min(n, (k + 1) * chunk_iters)
        m = OS.select_mode(False, e - s, cc[3 * k], cc[3 * k + 1], cc[3 * k + 2], tau_high)
        if tasks and tasks[-1][2] == m:
            tasks[-1][1] = e
        else:
            tasks.append([s, e, m])
    assert len(tasks) <= 64
    sets = []
    for s, e, _ in tasks:
        wr, rd = set(), set()
        for i in range(s, e):
            for arr, a, kind in _accesses(loop, i):
                (wr if kind == "w" else rd).add((arr, a))
        sets.append((wr, rd))
    conf = [0] * 64
    for u in range(len(tasks)):
        for t in range(u):
            (wt, rt), (wu, ru) = sets[t], sets[u]
            if wt & (wu | ru) or rt & wu:   # symmetric, as jp.h states it
                conf[u] |= 1 << t
                conf[t] |= 1 << u
    return [tuple(x) for x in tasks], conf


def jp_profile_plan_tasks(loop, chunk_iters, ws, tau_high=0.999):
    """jp.h jp_profile_plan_tasks: this rank's own profile of the whole loop (its
    full replica) with per-chunk counts, then the plan -- composed from the
    definitions above."""
    nck = -(-loop.n // chunk_iters)
    cc = torch.zeros(max(3 * nck, 3), dtype=torch.int64)
    jp_profile_stamp(loop, ws)
    prof = jp_profile_classify(loop, ws, chunk_iters=chunk_iters, chunk_counts=cc)
    ccl = cc.tolist()[:3 * nck]
    tasks, conf = jp_plan_tasks(loop, ccl, chunk_iters, ws, tau_high)
    return prof, ccl, tasks, conf


def jp_export_keys(loop, ws):
    ind = _indirect(loop)
    t = loop.tensors
    ix = lambda a, i: loop.ident_off + i if a is None else int(a[i])  # noqa: E731
    for arr in ("A", "T"):
        k = _view(ws, loop, "keys_" + arr, torch.int64)
        if k is None or not ind[arr] or (arr == "T" and loop.op != O.OP_PRIV_TMP):
            continue
        for i in range(loop.n):
            a = ix(t["w"], i) if arr == "A" else ix(t["s"], i)
            key = ((loop.iter_base + i + 1) << 32) | int(_np(t[arr]).view(np.uint32)[a])
            k[a] = max(int(k[a]), key)
