"""Shared test helpers: workload <-> oracle/jp conversions and random loops."""
from __future__ import annotations

import numpy as np
import torch

import oracle as O
import synth


def to_oracle(wl) -> O.Loop:
    a = lambda t: None if t is None else t.cpu().numpy()  # noqa: E731
    return O.Loop(wl.op, wl.dtype, wl.n, a(wl.A), r=a(wl.r), r2=a(wl.r2), w=a(wl.w), s=a(wl.s), X=a(wl.X),
                  T=a(wl.T), c0=wl.c0, c1=wl.c1)


def random_loop(seed: int, op: int, dtype: int, n: int, len_a: int | None = None, null_prob=0.2,
                dup_writes=True, slots=None) -> synth.Workload:
    """Random loop of any opcode; lengths are chosen so identity indices stay in range."""
    g = np.random.default_rng(seed)
    # decide which index arrays are NULL first: identity accesses need len >= n
    null = {k: g.random() < null_prob for k in ("r", "w", "r2", "s")}
    a_ident = (null["w"] or (op in (O.OP_ADD_C, O.OP_STENCIL2) and null["r"])
               or (op == O.OP_STENCIL2 and null["r2"]))
    la = len_a if len_a is not None else max(n, 8)
    if a_ident:
        la = max(la, n)
    lx = max(n, 8)
    lt = slots or max(8, n // 16)
    if op == O.OP_PRIV_TMP and null["s"]:
        lt = max(lt, n)
    el = np.int32 if dtype == O.I32 else np.float32

    def idx(key, hi):
        if null[key]:
            return None
        if dup_writes or hi < n:
            return torch.from_numpy(g.integers(0, hi, size=n).astype(np.int32))
        return torch.from_numpy(g.permutation(hi)[:n].astype(np.int32))

    def data(m):
        if dtype == O.I32:
            return torch.from_numpy(g.integers(-2**31, 2**31, size=m, dtype=np.int64).astype(np.int32))
        return torch.from_numpy(((g.integers(0, 2**23, size=m) * 2.0**-22) - 1).astype(el))

    r = idx("r", lx if op in (O.OP_SAXPY, O.OP_PRIV_TMP) else la)
    w = idx("w", la)
    r2 = idx("r2", la) if op == O.OP_STENCIL2 else None
    s = idx("s", lt) if op == O.OP_PRIV_TMP else None
    c0 = np.float32(1.1) if dtype == O.F32 else 7
    c1 = np.float32(0.3) if dtype == O.F32 else -3
    return synth.Workload("random", op, dtype, n, data(la), r=r, r2=r2, w=w, s=s,
                          X=data(lx) if op in (O.OP_SAXPY, O.OP_PRIV_TMP) else None,
                          T=data(lt) if op == O.OP_PRIV_TMP else None, c0=float(c0), c1=float(c1))


def bits_to_flags(raw_bits: torch.Tensor, n: int) -> np.ndarray:
    b = raw_bits.cpu().numpy().view(np.uint32)
    out = np.zeros(n, dtype=np.uint8)
    for k in range(n):
        out[k] = (b[k >> 5] >> (k & 31)) & 1
    return out


def region_workload(wl, b: int, e: int, name: str = None):
    """Iterations [b, e) of an indirect loop as a loop of its own (same arrays,
    index arrays sliced), e.g. config 5's privatized tail or DOALL head."""
    import synth
    return synth.Workload(name or f"{wl.name}[{b}:{e}]", wl.op, wl.dtype, e - b, wl.A.clone(),
                          r=None if wl.r is None else wl.r[b:e].clone(),
                          r2=None if wl.r2 is None else wl.r2[b:e].clone(),
                          w=None if wl.w is None else wl.w[b:e].clone(),
                          s=None if wl.s is None else wl.s[b:e].clone(),
                          X=wl.X, T=None if wl.T is None else wl.T.clone(), c0=wl.c0, c1=wl.c1)


def seq_mixed(n: int = 3 * 4096, seed: int = 9):
    """ADD_C int32 over three equal regions with disjoint addresses: a permutation
    (DOALL), a dependence chain r[i] = w[i-1] (d_raw = 100%: Fig. 2(b) mode C),
    and a permutation again."""
    assert n % 3 == 0
    m = n // 3
    g = np.random.default_rng(seed)
    w = np.concatenate([g.permutation(m), m + np.arange(m), 2 * m + g.permutation(m)]).astype(np.int32)
    r = w.copy()
    r[m + 1:2 * m] = w[m:2 * m - 1]
    A = g.integers(0, 1 << 20, size=n).astype(np.int32)
    return synth.Workload("seq_mixed", O.OP_ADD_C, O.I32, n, torch.from_numpy(A), r=torch.from_numpy(r),
                          w=torch.from_numpy(w), c0=7)
