"""GPU parity of TLS with on-chip recovery (JP_TLS_ONCHIP, reading B7)
against oracle/jpo.c jpo_sim_tls_fwd: every output array byte-equal and the
statistics (windows, violations, executed, committed) exact, through the C ABI.

Loops must write no address twice (profile waw_iters == 0), so the cases are
the dependent-set generator of configs 1/3 (w a permutation), write-once
random loops of every opcode, and the full-length dependence chains
(prefix chain, Gauss-Seidel) that make every iteration of a window wait on
its predecessor's forwarded value.
"""
import numpy as np
import pytest
import torch

import oracle as O
import synth
from helpers import random_loop, to_oracle

pytestmark = pytest.mark.gpu

if torch.cuda.is_available():
    import paper_conf_icpp_hanzlw13_b200 as jp
    DEV = torch.device("cuda:0")
else:  # collected on CPU boxes, never run there
    jp = None
    DEV = None

OPS = [O.OP_ADD_C, O.OP_SAXPY, O.OP_PRIV_TMP, O.OP_STENCIL2]
DTS = [O.I32, O.F32]


def same(t: torch.Tensor, a: np.ndarray) -> bool:
    return t.cpu().numpy().tobytes() == a.tobytes()


def grid_w():
    return jp.jp_tls_grid_window()


def fwd_case(wl, window, cluster=0, guided=False, view=None, path=5):
    """Profile -> (guide) -> on-chip TLS on path 5 (cluster) or 6 (every SM);
    compare with the oracle.  window = 0: the path's own window."""
    ref = to_oracle(wl)
    g = wl.to(DEV)
    L = jp.Loop.from_workload(g) if view is None else view(g)
    ws = jp.workspace(L)
    p = jp.jp_profile_density(L, ws)
    assert p["waw_iters"] == 0
    if guided:
        jp.jp_tls_guide(L, ws)
    got = jp.jp_run_tls(L, window=window, prof=p, ws=ws, cluster=cluster, guided=guided,
                        recovery=jp.JP_TLS_ONCHIP, path=path)
    torch.cuda.synchronize()
    W = window
    if W == 0 and path == 6:
        W = grid_w()
    elif W == 0:
        c = cluster
        if c == 0:
            c = 1
            while c < 16 and 2048 * c < wl.n:
                c *= 2
        W = 2048 * c
    st, A, T, stats = O.sim_tls_fwd(ref, W)
    assert st == O.OK
    assert same(g.A, A), f"A differs at {np.flatnonzero(g.A.cpu().numpy() != A)[:10]}"
    if T is not None:
        assert same(g.T, T)
    assert got == stats, (got, stats)
    return got


@pytest.mark.parametrize("window", [1, 32, 100, 1000, 2048, 4096, 0])
@pytest.mark.parametrize("d", [0.0, 0.05])
@pytest.mark.parametrize("path", [5, 6])
def test_fwd_config1(window, d, path):
    fwd_case(synth.config1(d), window, path=path)


@pytest.mark.parametrize("cluster", [1, 2, 4, 8, 16])
def test_fwd_cluster_sizes(cluster):
    wl = synth.config3(0.05, n=(1 << 15) + 77)
    for window in (96, 1000, 2048 * cluster):
        fwd_case(wl, window, cluster=cluster)
        fwd_case(wl, window, cluster=cluster, guided=True)


@pytest.mark.parametrize("d", [0.001, 0.01, 0.05, 0.10])
@pytest.mark.parametrize("guided", [False, True])
def test_fwd_config3_reduced(d, guided):
    wl = synth.config3(d, n=(1 << 17) + 11)
    for window in (4096, 32768, 0):
        fwd_case(wl, window, guided=guided)
    for window in (4096, 100000, 0):
        fwd_case(wl, window, guided=guided, path=6)


@pytest.mark.parametrize("op,dt", [(op, dt) for op in OPS for dt in DTS])
def test_fwd_random_write_once(op, dt):
    """Write-once random loops (w a partial permutation; PRIV_TMP's s too) of every
    opcode and dtype, NULL indices included, several windows and clusters."""
    n = 7001
    wl = random_loop(1300 + op * 10 + dt, op, dt, n, len_a=3 * n, null_prob=0.2, dup_writes=False,
                     slots=2 * n)
    for window, cluster in ((64, 0), (1500, 0), (2048, 1), (4096, 2), (0, 0)):
        fwd_case(wl, window, cluster=cluster)
        if op != O.OP_PRIV_TMP:
            fwd_case(wl, window, cluster=cluster, guided=True)
    for window in (64, 2500, 0):
        fwd_case(wl, window, path=6)
        if op != O.OP_PRIV_TMP:
            fwd_case(wl, window, guided=True, path=6)


def test_fwd_chains():
    """Every iteration depends on the previous one (prefix chain, Gauss-Seidel):
    each window resolves a dependence chain as long as the window."""
    n = 40000
    A0 = torch.arange(n, dtype=torch.int32) * 3
    ar = torch.arange(n, dtype=torch.int32)
    pc = synth.Workload("pc", O.OP_ADD_C, O.I32, n, A0.clone(), r=torch.clamp(ar - 1, min=0), w=ar.clone(), c0=7)
    for window in (100, 2048, 32768):
        st = fwd_case(pc, window)
        assert st["violations"] == n - -(-n // window)
    gs = synth.Workload("gs", O.OP_STENCIL2, O.F32, n, (A0.float() * 0.01).clone(), r=torch.clamp(ar - 1, min=0),
                        r2=torch.clamp(ar + 1, max=n - 1), w=ar.clone(), c0=0.4)
    for window in (777, 32768):
        fwd_case(gs, window)
        fwd_case(gs, window, guided=True)
    for window in (1000, 40000):
        assert fwd_case(pc, window, path=6)["violations"] == n - -(-n // window)
        fwd_case(gs, window, path=6, guided=True)


def test_fwd_unaligned_views():
    """Index streams that start 3 entries into their tensors."""
    n = 9000
    wl = synth.config3(0.05, n=n + 3)
    sl = lambda t: None if t is None else t[3:]  # noqa: E731
    sub = synth.Workload("sub", wl.op, wl.dtype, n, wl.A.clone(), r=sl(wl.r), w=sl(wl.w), c0=wl.c0)
    view = lambda g: jp.Loop(wl.op, wl.dtype, n, g.A, r=sl(g.r), w=sl(g.w), c0=wl.c0)  # noqa: E731
    ref = to_oracle(sub)
    g = wl.to(DEV)
    L = view(g)
    ws = jp.workspace(L)
    p = jp.jp_profile_density(L, ws)
    got = jp.jp_run_tls(L, window=1000, prof=p, ws=ws, recovery=jp.JP_TLS_ONCHIP)
    torch.cuda.synchronize()
    _, A, _, stats = O.sim_tls_fwd(ref, 1000)
    assert same(g.A, A) and got == stats


def test_fwd_repeatability():
    """Races in the write log or the shadow-slot polls would show as run-to-run differences."""
    wl = synth.config3(0.10, n=1 << 20)
    ref = to_oracle(wl)
    _, A, _, stats = O.sim_tls_fwd(ref, 32768)
    g = wl.to(DEV)
    A0 = g.A.clone()
    L = jp.Loop.from_workload(g)
    ws = jp.workspace(L)
    p = jp.jp_profile_density(L, ws)
    jp.jp_tls_guide(L, ws)
    for rep in range(10):
        g.A.copy_(A0)
        got = jp.jp_run_tls(L, window=32768, prof=p, ws=ws, guided=bool(rep & 1), recovery=jp.JP_TLS_ONCHIP,
                            path=5 + (rep & 2) // 2)
        torch.cuda.synchronize()
        assert same(g.A, A) and got == stats, rep


def test_fwd_needs_write_once_profile():
    wl = random_loop(5, O.OP_ADD_C, O.I32, 3000, len_a=64, null_prob=0.0)
    g = wl.to(DEV)
    L = jp.Loop.from_workload(g)
    ws = jp.workspace(L)
    with pytest.raises(jp.JPError):          # no profile
        jp.jp_run_tls(L, window=64, ws=ws, recovery=jp.JP_TLS_ONCHIP)
    p = jp.jp_profile_density(L, ws)
    assert p["waw_iters"] > 0
    with pytest.raises(jp.JPError):          # profile with WAW
        jp.jp_run_tls(L, window=64, prof=p, ws=ws, recovery=jp.JP_TLS_ONCHIP)
    wl3 = synth.config3(0.01, n=1 << 16).to(DEV)
    L3 = jp.Loop.from_workload(wl3)
    p3 = jp.jp_profile_density(L3, jp.workspace(L3))
    with pytest.raises(jp.JPError):          # window larger than a 16-CTA cluster holds
        jp.jp_run_tls(L3, window=2048 * 16 + 1, prof=p3, ws=jp.workspace(L3), recovery=jp.JP_TLS_ONCHIP, path=5)
    with pytest.raises(jp.JPError):          # window larger than the given cluster holds
        jp.jp_run_tls(L3, window=4097, cluster=2, prof=p3, ws=jp.workspace(L3), recovery=jp.JP_TLS_ONCHIP)


@pytest.mark.parametrize("d", [0.001, 0.01, 0.05, 0.10])
def test_fwd_config3_full_size_schedule(d):
    """BASELINE size N=2^24 through jp_schedule (profile -> Fig. 2(b) TLS -> guide ->
    on-chip recovery, the default for write-once loops): full arrays and stats."""
    wl = synth.config3(d)
    ref = to_oracle(wl)
    g = wl.to(DEV)
    L = jp.Loop.from_workload(g)
    res = jp.jp_schedule(L, jp.workspace(L))
    torch.cuda.synchronize()
    # write-once, WAR-free ADD_C: one window of the whole loop, DC from the guide (path 8)
    assert res["mode"] == jp.JP_MODE_TLS and res["tls_recovery"] == jp.JP_TLS_ONCHIP and res["tls_path"] == 8
    assert res["tls_w_max"] == wl.n and res["tls_guided"] == 1
    _, A, _, stats = O.sim_tls_fwd(ref, res["tls_w_max"])
    assert same(g.A, A)
    assert res["tls"] == stats, (res["tls"], stats)


def test_fwd_grid_window_cap():
    wl = synth.config3(0.01, n=1 << 16).to(DEV)
    L = jp.Loop.from_workload(wl)
    ws = jp.workspace(L)
    p = jp.jp_profile_density(L, ws)
    with pytest.raises(jp.JPError):
        jp.jp_run_tls(L, window=grid_w() + 1, prof=p, ws=ws, recovery=jp.JP_TLS_ONCHIP, path=6)
    with pytest.raises(jp.JPError):          # not an on-chip path
        jp.jp_run_tls(L, window=100, prof=p, ws=ws, recovery=jp.JP_TLS_ONCHIP, path=1)


@pytest.mark.parametrize("case", ["c3_0", "c3_1", "c3_10", "stencil", "saxpy_null"])
def test_schedule_fused_guide_bits(case):
    """jp_schedule writes the guide bitmaps in its classify pass (no jp_tls_guide):
    raw words == the oracle's raw flags, source words == oracle raw_sources, for
    write-once loops (the only loops a guided run accepts); the run is exact."""
    from helpers import bits_to_flags
    if case.startswith("c3"):
        wl = synth.config3({"c3_0": 0.0, "c3_1": 0.01, "c3_10": 0.10}[case], n=(1 << 16) + 9)
    elif case == "stencil":
        wl = random_loop(77, O.OP_STENCIL2, O.F32, 5000, len_a=15000, null_prob=0.0, dup_writes=False)
    else:
        wl = random_loop(78, O.OP_ADD_C, O.I32, 5003, len_a=15000, null_prob=0.5, dup_writes=False)
    ref = to_oracle(wl)
    _, A, _ = O.run_seq(ref)
    g = wl.to(DEV)
    L = jp.Loop.from_workload(g)
    ws = jp.workspace(L)
    res = jp.jp_schedule(L, ws)
    torch.cuda.synchronize()
    assert same(g.A, A)
    off, nb = jp.jp_ws_region(L, "guide")
    if nb == 0:
        return
    nw = (wl.n + 31) // 32
    words = ws[off:off + 8 * nw].view(torch.int32)
    assert np.array_equal(bits_to_flags(words[:nw], wl.n), O.profile(ref)["flags"] & 1)
    assert np.array_equal(bits_to_flags(words[nw:], wl.n), O.raw_sources(ref))
    if res["mode"] == jp.JP_MODE_TLS:
        assert res["tls"] == O.sim_tls_fwd(ref, res["tls_w_max"])[3]


def flow_case(wl, monkey_buckets=None):
    """jp_run_tls path 8 (one window, DC from the guide) after a profile and the
    guide on the same workspace: arrays == sequential, stats == jpo_sim_tls_fwd
    with W = n (one window; violations = raw iterations; executed = n + raw)."""
    ref = to_oracle(wl)
    g = wl.to(DEV)
    L = jp.Loop.from_workload(g)
    ws = jp.workspace(L)
    p = jp.jp_profile_density(L, ws)
    jp.jp_tls_guide(L, ws)
    got = jp.jp_run_tls(L, window=0, prof=p, ws=ws, guided=True, recovery=jp.JP_TLS_ONCHIP, path=8)
    torch.cuda.synchronize()
    st, A, _, stats = O.sim_tls_fwd(ref, max(wl.n, 1))
    assert same(g.A, A), f"A differs at {np.flatnonzero(g.A.cpu().numpy() != A)[:10]}"
    assert got == stats, (got, stats)
    assert got["violations"] == O.profile(ref)["raw_iters"]
    return got


@pytest.mark.parametrize("d", [0.0, 0.001, 0.05, 0.5, 1.0])
@pytest.mark.parametrize("delta", [1, 64, 1024])
def test_flow_config3_shapes(d, delta):
    """Densities up to chains (delta = 1, d = 1: every iteration waits on the previous one)."""
    n = (1 << 16) + 7 if d < 0.5 or delta > 1 else 5000
    flow_case(synth.config3(d, n=n, delta=delta))


@pytest.mark.parametrize("dt", [O.I32, O.F32])
@pytest.mark.parametrize("seed", range(3))
def test_flow_random_write_once(dt, seed):
    """Write-once ADD_C loops (w a permutation) whose reads are either an earlier
    iteration's write (RAW) or the iteration's own address -- WAR-free."""
    g0 = np.random.default_rng(40 + seed)
    n = [777, 20000, 300001][seed]
    w = g0.permutation(n).astype(np.int32)
    r = w.copy()
    dep = g0.random(n) < 0.3
    back = np.maximum(np.arange(n) - g0.integers(1, 2000, n), 0)
    r[dep] = w[back[dep]]
    A = g0.integers(-1000, 1000, n).astype(np.int32) if dt == O.I32 else g0.standard_normal(n).astype(np.float32)
    wl = synth.Workload("flow", O.OP_ADD_C, dt, n, torch.from_numpy(A), r=torch.from_numpy(r), w=torch.from_numpy(w),
                        c0=(3 if dt == O.I32 else 1.1))
    p = O.profile(to_oracle(wl))
    assert p["waw_iters"] == 0 and p["war_iters"] == 0
    flow_case(wl)


def test_flow_preconditions():
    """Path 8 refuses loops it cannot run exactly: WAR present, STENCIL2, no guide."""
    n = 4000
    ar = torch.arange(n, dtype=torch.int32)
    ahead = synth.Workload("ahead", O.OP_ADD_C, O.I32, n, torch.arange(n + 1, dtype=torch.int32), r=ar + 1, w=ar.clone(),
                           c0=1)     # reads ahead: WAR
    g = ahead.to(DEV)
    L = jp.Loop.from_workload(g)
    ws = jp.workspace(L)
    p = jp.jp_profile_density(L, ws)
    assert p["war_iters"] > 0 and p["waw_iters"] == 0
    jp.jp_tls_guide(L, ws)
    with pytest.raises(jp.JPError):
        jp.jp_run_tls(L, prof=p, ws=ws, guided=True, recovery=jp.JP_TLS_ONCHIP, path=8)
    wl = synth.config3(0.01, n=n)
    g = wl.to(DEV)
    L = jp.Loop.from_workload(g)
    ws = jp.workspace(L)
    p = jp.jp_profile_density(L, ws)
    with pytest.raises(jp.JPError):       # no guide words
        jp.jp_run_tls(L, prof=p, ws=ws, guided=False, recovery=jp.JP_TLS_ONCHIP, path=8)
    with pytest.raises(jp.JPError):       # a fixed window shorter than the loop
        jp.jp_tls_guide(L, ws)
        jp.jp_run_tls(L, window=100, prof=p, ws=ws, guided=True, recovery=jp.JP_TLS_ONCHIP, path=8)


def test_schedule_flow_and_windowed_agree(monkeypatch):
    """jp_schedule picks path 8 for config 3; JP_TLS_NO_FLOW=1 keeps the windowed
    all-SM kernel (path 6); both reach the sequential state with their own stats."""
    wl = synth.config3(0.05, n=(1 << 20) + 3)
    ref = to_oracle(wl)
    _, A, _ = O.run_seq(ref)
    for env, path in (("0", 8), ("1", 6)):
        if env == "1":
            monkeypatch.setenv("JP_TLS_NO_FLOW", "1")
        g = wl.to(DEV)
        L = jp.Loop.from_workload(g)
        res = jp.jp_schedule(L, jp.workspace(L))
        torch.cuda.synchronize()
        assert res["tls_path"] == path, res
        assert same(g.A, A)
        assert res["tls"] == O.sim_tls_fwd(ref, res["tls_w_max"])[3]
