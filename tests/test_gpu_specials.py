"""GPU parity on IEEE binary32 specials through every mode and kernel family
(reading A12: RN-even, two rounded ops, no contraction, no FTZ/DAZ; reading
A12b: a NaN result compares as NaN -- the payload is not part
of the contract, since x86 SSE propagates an operand's payload and sm_100
returns the canonical NaN -- every other result compares bit for bit, so +0 and
-0 differ and subnormals must survive).

Inputs mix +-0, +-inf, quiet NaNs with payloads, subnormals and near-overflow
values (synth.f32_specials) into the usual data; expected values come from
oracle/ only.
"""
import itertools

import numpy as np
import pytest
import torch

import oracle as O
import synth
from helpers import to_oracle

pytestmark = pytest.mark.gpu

if torch.cuda.is_available():
    import paper_conf_icpp_hanzlw13_b200 as jp
    DEV = torch.device("cuda:0")
else:  # collected on CPU boxes, never run there
    jp = None
    DEV = None

OPS = [O.OP_ADD_C, O.OP_SAXPY, O.OP_PRIV_TMP, O.OP_STENCIL2]
C0S = [1.1, -0.0, float(np.float32(1e-40)), float("inf")]


def nan_eq(got: torch.Tensor, exp: np.ndarray):
    g = got.cpu().numpy().astype(np.float32, copy=False)
    e = np.asarray(exp, dtype=np.float32)
    gn, en = np.isnan(g), np.isnan(e)
    bad = np.flatnonzero(gn != en)
    if bad.size:
        return False, bad[:8]
    gb, eb = g.view(np.uint32), e.view(np.uint32)
    bad = np.flatnonzero((gb != eb) & ~gn)
    return bad.size == 0, bad[:8]


def check(g, A, T):
    ok, where = nan_eq(g.A, A)
    assert ok, f"A differs at {where}: got {g.A.cpu().numpy()[where]} want {A[where]}"
    if T is not None:
        ok, where = nan_eq(g.T, T)
        assert ok, f"T differs at {where}"


def sp(seed, stream, n):
    return synth.f32_specials(seed, stream, n)


def special_loop(op, n, seed, r=None, r2=None, w=None, s=None, la=None, lt=None, c0=1.1, c1=-0.0):
    la = la or n
    return synth.Workload(f"specials{op}", op, O.F32, n, sp(seed, 1, la), r=r, r2=r2, w=w, s=s,
                          X=sp(seed, 2, max(n, la)) if op in (O.OP_SAXPY, O.OP_PRIV_TMP) else None,
                          T=sp(seed, 3, lt or max(8, n // 16)) if op == O.OP_PRIV_TMP else None, c0=c0, c1=c1)


@pytest.fixture(params=[0, 1], ids=["ldg128", "tma"])
def doall_kernel(request):
    old = jp.jp_doall_kernel(-1)
    jp.jp_doall_kernel(request.param)
    yield request.param
    jp.jp_doall_kernel(old)


@pytest.mark.parametrize("op,c0", list(itertools.product(OPS, C0S)))
def test_specials_doall_affine(op, c0, doall_kernel):
    n = (1 << 20) + 3
    wl = special_loop(op, n, 11 + op, c0=c0, lt=n)
    _, A, T = O.run_seq(to_oracle(wl))
    g = wl.to(DEV)
    res = jp.jp_schedule(jp.Loop.from_workload(g))
    torch.cuda.synchronize()
    assert res["mode"] == jp.JP_MODE_DOALL
    check(g, A, T)


@pytest.mark.parametrize("generic", ["0", "1"])
@pytest.mark.parametrize("op", OPS)
def test_specials_doall_indirect(op, generic, monkeypatch):
    if generic == "1":
        monkeypatch.setenv("JP_DOALL_GENERIC", "1")
    n = 300001
    g0 = np.random.default_rng(op)
    pi = torch.from_numpy(g0.permutation(n).astype(np.int32))
    kw = dict(w=pi)
    if op == O.OP_ADD_C:
        kw["r"] = pi
    elif op == O.OP_STENCIL2:
        kw.update(r=pi, r2=pi)
    else:
        kw["r"] = torch.from_numpy(g0.permutation(n).astype(np.int32))
    if op == O.OP_PRIV_TMP:
        kw["s"] = torch.from_numpy(g0.permutation(n).astype(np.int32))
    wl = special_loop(op, n, 21 + op, lt=n, **kw)
    _, A, T = O.run_seq(to_oracle(wl))
    g = wl.to(DEV)
    L = jp.Loop.from_workload(g)
    res = jp.jp_schedule(L, jp.workspace(L), static_check=1)
    torch.cuda.synchronize()
    assert res["mode"] == jp.JP_MODE_DOALL
    check(g, A, T)


@pytest.mark.parametrize("c0", C0S)
def test_specials_privatized_config4_shape(c0, doall_kernel):
    """PRIV_TMP (config 4's shape: identity X / Y, s over 1024 slots) -- the
    streamed kernels (bulk-copy staged and 16-B vector)."""
    n = (1 << 20) + 77
    s = (synth.rnd(1004, 3, torch.arange(n, dtype=torch.int64)) & 1023).to(torch.int32)
    wl = special_loop(O.OP_PRIV_TMP, n, 31, s=s, lt=1024, c0=c0)
    _, A, T = O.run_seq(to_oracle(wl))
    g = wl.to(DEV)
    L = jp.Loop.from_workload(g)
    res = jp.jp_schedule(L, jp.workspace(L))
    torch.cuda.synchronize()
    assert res["mode"] == jp.JP_MODE_PRIVATIZED
    check(g, A, T)


def generic_priv_loop(op, n):
    """Raw-free loops with WAR and WAW: w 2-to-1 onto [0, n/2) (WAW); an odd i
    reads ahead the address the next (even) iteration writes first (WAR); even
    iterations read the read-only region [n/2 + 2, n + 2).  PRIV_TMP: scratch
    slots reused every 97 iterations (WAR and WAW through T)."""
    ar = torch.arange(n, dtype=torch.int64)
    if op == O.OP_PRIV_TMP:
        pi = torch.from_numpy(np.random.default_rng(5).permutation(n).astype(np.int32))
        return special_loop(op, n, 41, r=pi, w=pi, s=(ar % 97).to(torch.int32), lt=97)
    w = (ar // 2).to(torch.int32)
    ro = n // 2 + 2
    r = torch.where(ar % 2 == 1, (ar + 1) // 2, ro + ar // 2).clamp(max=n + 1).to(torch.int32)
    r2 = (ro + (ar * 7) % (n + 2 - ro)).to(torch.int32) if op == O.OP_STENCIL2 else None
    return special_loop(op, n, 41, r=r, r2=r2, w=w, la=n + 2)


@pytest.mark.parametrize("op", [O.OP_ADD_C, O.OP_STENCIL2, O.OP_PRIV_TMP])
def test_specials_privatized_generic(op):
    """The generic privatized kernel (packed last-writer keys) on specials."""
    wl = generic_priv_loop(op, 200003)
    ref = to_oracle(wl)
    p = O.profile(ref)
    assert p["raw_iters"] == 0 and p["waw_iters"] > 0 and p["war_iters"] > 0, p
    _, A, T = O.run_seq(ref)
    g = wl.to(DEV)
    L = jp.Loop.from_workload(g)
    res = jp.jp_schedule(L, jp.workspace(L))
    torch.cuda.synchronize()
    assert res["mode"] == jp.JP_MODE_PRIVATIZED
    check(g, A, T)


def tls_loop(op, n, d, seed):
    """Write-once loop with RAW at density d (the config-3 recipe) over fp32 specials."""
    r, w, _ = synth.dep_region(seed, n, 0, d, 64)
    kw = dict(r=r, w=w)
    if op == O.OP_STENCIL2:
        kw["r2"] = torch.roll(r, 1)
    if op == O.OP_SAXPY:
        kw["r"] = torch.from_numpy(np.random.default_rng(seed).permutation(n).astype(np.int32))
    if op == O.OP_PRIV_TMP:
        kw["s"] = torch.from_numpy(np.random.default_rng(seed + 1).permutation(n).astype(np.int32))
        kw["r"] = kw["s"]
    return special_loop(op, n, seed, lt=n, **kw)


@pytest.mark.parametrize("path,window", [(1, 1024), (2, 8192), (3, 4096)])
@pytest.mark.parametrize("op", OPS)
def test_specials_tls_restart(op, path, window):
    wl = tls_loop(op, 50000, 0.05, 51 + op)
    ref = to_oracle(wl)
    st, A, T, stats = O.sim_tls(ref, window)
    g = wl.to(DEV)
    L = jp.Loop.from_workload(g)
    got = jp.jp_run_tls(L, window=window, path=path, ws=jp.workspace(L))
    torch.cuda.synchronize()
    check(g, A, T)
    assert got == stats


@pytest.mark.parametrize("path", [5, 6])
@pytest.mark.parametrize("op", OPS)
def test_specials_tls_onchip(op, path):
    wl = tls_loop(op, 60000, 0.05, 61 + op)
    ref = to_oracle(wl)
    g = wl.to(DEV)
    L = jp.Loop.from_workload(g)
    ws = jp.workspace(L)
    p = jp.jp_profile_density(L, ws)
    assert p["waw_iters"] == 0
    W = 8192 if path == 5 else 0
    got = jp.jp_run_tls(L, window=W, prof=p, ws=ws, recovery=jp.JP_TLS_ONCHIP, path=path)
    torch.cuda.synchronize()
    st, A, T, stats = O.sim_tls_fwd(ref, W if W else jp.jp_tls_grid_window())
    check(g, A, T)
    assert got == stats


@pytest.mark.parametrize("op", OPS)
def test_specials_serial_and_tiny(op):
    """Path 7 (one warp, program order) on a dependence chain, and the one-CTA
    tiny schedule (n <= 4096) through jp_schedule."""
    n = 20000
    ar = torch.arange(n, dtype=torch.int32)
    kw = dict(r=torch.clamp(ar - 1, min=0).to(torch.int32), w=ar.clone())
    if op == O.OP_STENCIL2:
        kw["r2"] = torch.clamp(ar + 1, max=n - 1).to(torch.int32)
    if op in (O.OP_SAXPY, O.OP_PRIV_TMP):
        kw["s"] = ar.clone() if op == O.OP_PRIV_TMP else None
    wl = special_loop(op, n, 71 + op, lt=n, **kw)
    ref = to_oracle(wl)
    _, A, T = O.run_seq(ref)
    g = wl.to(DEV)
    L = jp.Loop.from_workload(g)
    jp.jp_run_tls(L, path=7, ws=jp.workspace(L))
    torch.cuda.synchronize()
    check(g, A, T)
    for d in (0.0, 0.05):
        wt = tls_loop(op, 4096, d, 81 + op)
        _, A, T = O.run_seq(to_oracle(wt))
        g = wt.to(DEV)
        L = jp.Loop.from_workload(g)
        jp.jp_schedule(L, jp.workspace(L))
        torch.cuda.synchronize()
        check(g, A, T)
