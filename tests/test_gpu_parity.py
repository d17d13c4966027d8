"""GPU parity: every mode of libjp.so against the CPU oracle (bit-exact).

Run on a B200 with ``pytest -m gpu``.  Every call goes through the C ABI
(paper_conf_icpp_hanzlw13_b200 -> libjp.so); the expected values come only from
oracle/ (test infrastructure) on the same seeded inputs.  Tolerance: none --
int32 bodies wrap and fp32 bodies are two separately rounded RN ops compiled
with -fmad=false on both sides (BASELINE.json north_star; reading A12), so the
bar is byte equality of every output array and exact integer statistics.
"""
import itertools
import os
import shutil
import subprocess
import sys

import numpy as np
import pytest
import torch

import oracle as O
import synth
from helpers import bits_to_flags, random_loop, to_oracle

pytestmark = pytest.mark.gpu

if torch.cuda.is_available():
    import paper_conf_icpp_hanzlw13_b200 as jp
    DEV = torch.device("cuda:0")
else:  # collected on CPU boxes, never run there
    jp = None
    DEV = None

OPS = [O.OP_ADD_C, O.OP_SAXPY, O.OP_PRIV_TMP, O.OP_STENCIL2]
DTS = [O.I32, O.F32]


def gpu(wl):
    return wl.to(DEV)


def same(t: torch.Tensor, a: np.ndarray) -> bool:
    return t.cpu().numpy().tobytes() == a.tobytes()


def check_arrays(g, A, T):
    assert same(g.A, A), f"A differs at {np.flatnonzero(g.A.cpu().numpy() != A)[:10]}"
    if T is not None:
        assert same(g.T, T), f"T differs at {np.flatnonzero(g.T.cpu().numpy() != T)[:10]}"


# ---------------------------------------------------------------------------
# profiler
# ---------------------------------------------------------------------------
def prof_case(wl):
    ref = O.profile(to_oracle(wl))
    g = gpu(wl)
    L = jp.Loop.from_workload(g)
    ws = jp.workspace(L, jp.JP_WS_PROFILE)
    bits = torch.zeros((wl.n + 31) // 32 + 1, dtype=torch.int32, device=DEV)
    p = jp.jp_profile_density(L, ws, raw_bits=bits)
    assert (p["raw_iters"], p["war_iters"], p["waw_iters"]) == (ref["raw_iters"], ref["war_iters"], ref["waw_iters"])
    assert p["first_raw_iter"] == ref["first_raw_iter"]
    assert np.array_equal(bits_to_flags(bits, wl.n), ref["flags"] & 1)
    return p, ref


@pytest.mark.parametrize("op,dt,seed", [(op, dt, s) for op in OPS for dt in DTS for s in range(3)])
def test_profile_random(op, dt, seed):
    n = [1, 37, 1000, 4099][seed % 4] if seed < 3 else 5000
    wl = random_loop(1000 * op + 10 * dt + seed, op, dt, n + 17 * seed, len_a=max(64, (n + 17 * seed) // 3))
    prof_case(wl)


@pytest.mark.parametrize("d", [0.0, 0.05])
def test_profile_config1(d):
    p, _ = prof_case(synth.config1(d))
    assert p["raw_iters"] == (205 if d else 0)


@pytest.mark.parametrize("d", [0.001, 0.01, 0.05, 0.10])
def test_profile_config3_reduced(d):
    prof_case(synth.config3(d, n=(1 << 18) + 5))


def test_profile_config4_and_5():
    prof_case(synth.config4(n=(1 << 18) + 3))
    prof_case(synth.config5(n=1 << 16))


@pytest.mark.parametrize("kernel", ["quad", "ballot"])
@pytest.mark.parametrize("chunk,n", [(1024, 1 << 16), (160, (1 << 16) + 77), (96, 40000), (32, 5000)])
def test_profile_chunk_counts(kernel, chunk, n, monkeypatch):
    """Per-chunk counts (the stealing scheduler's input): the quad kernel with
    warp-aggregated chunk atomics (chunk >= 128) and the ballot kernel
    (JP_CLASSIFY_BALLOT=1, and every chunk < 128) against the oracle's flags."""
    if kernel == "ballot":
        monkeypatch.setenv("JP_CLASSIFY_BALLOT", "1")
    wl = synth.config5(n=1 << 16) if n == 1 << 16 else random_loop(n, O.OP_STENCIL2, O.I32, n, len_a=n // 2)
    ref = O.profile(to_oracle(wl))
    g = gpu(wl)
    L = jp.Loop.from_workload(g)
    ws = jp.workspace(L)
    nck = -(-wl.n // chunk)
    cc = torch.full((nck * 3,), -7, dtype=torch.int64, device=DEV)
    jp.jp_profile_density(L, ws, chunk_iters=chunk, chunk_counts=cc)
    cc = cc.cpu().numpy().reshape(-1, 3)
    f = np.concatenate([ref["flags"], np.zeros(nck * chunk - wl.n, dtype=ref["flags"].dtype)]).reshape(-1, chunk)
    assert np.array_equal(cc[:, 0], (f & 1).sum(1))
    assert np.array_equal(cc[:, 1], ((f >> 1) & 1).sum(1))
    assert np.array_equal(cc[:, 2], ((f >> 2) & 1).sum(1))


def test_profile_partitioned_equals_whole():
    """C1: stamp each rank's range with global ids, MAX-combine the int32 tables,
    classify each range; the summed counts equal the single-GPU profile."""
    wl = synth.config3(0.05, n=1 << 16)
    ref = O.profile(to_oracle(wl))
    g = gpu(wl)
    k = 3
    rg = jp.jp_plan_sharing(wl.n, k)
    loops, wss = [], []
    for (s, e) in rg:
        L = jp.Loop(g.op, g.dtype, e - s, g.A, r=g.r[s:e], w=g.w[s:e], c0=g.c0, iter_base=s)
        loops.append(L)
        wss.append(jp.workspace(L, jp.JP_WS_PROFILE))
        jp.jp_profile_stamp(L, wss[-1])
    torch.cuda.synchronize()
    for reg in ("minW_A", "minR_A"):
        off, nb = jp.jp_ws_region(loops[0], reg)
        views = [w[off:off + nb].view(torch.int32) for w in wss]
        m = views[0].clone()
        for v in views[1:]:
            m = torch.maximum(m, v)
        for v in views:
            v.copy_(m)
    tot = [0, 0, 0]
    for L, w in zip(loops, wss):
        p = jp.jp_profile_classify(L, w)
        tot = [tot[0] + p["raw_iters"], tot[1] + p["war_iters"], tot[2] + p["waw_iters"]]
    assert tot == [ref["raw_iters"], ref["war_iters"], ref["waw_iters"]]


def test_index_error_no_side_effects():
    wl = synth.config1(0.05)
    wl.w[100] = 4096   # out of range
    g = gpu(wl)
    A0 = g.A.clone()
    L = jp.Loop.from_workload(g)
    ws = jp.workspace(L)
    with pytest.raises(jp.JPError) as e:
        jp.jp_profile_density(L, ws)
    assert e.value.status == -5
    for fn in (lambda: jp.jp_run_doall(L, None, ws), lambda: jp.jp_run_privatized(L, None, ws),
               lambda: jp.jp_run_tls(L, 256, ws=ws), lambda: jp.jp_schedule(L, ws)):
        with pytest.raises(jp.JPError) as e:
            fn()
        assert e.value.status == -5
    torch.cuda.synchronize()
    assert torch.equal(g.A, A0)
    assert jp.jp_validate(L, ws) == 1


@pytest.mark.parametrize("case", ["c4", "c4_w", "saxpy_r", "c4_tail"])
def test_structural_raw_free_schedule(case, doall_kernel):
    """Reading B11: PRIV_TMP (X read-only, T's read covered) and SAXPY with
    identity writes are run without a profile (profiled = 0) -- results equal the
    oracle; an out-of-range indirect index gives JP_ERR_INDEX with every array
    untouched (the run launched behind the device check exits at once)."""
    n = (1 << 20) + 77
    g0 = np.random.default_rng(3)
    if case == "c4":
        wl, mode = synth.config4(n=n), jp.JP_MODE_PRIVATIZED
    elif case == "c4_tail":   # one 4096-iteration tile and a ragged element tail (beyond the tiny path)
        n = 4096 + 3001
        wl, mode = synth.config4(n=n), jp.JP_MODE_PRIVATIZED
    elif case == "c4_w":   # Y written through a 2-to-1 index: WAW on Y as well
        wl, mode = synth.config4(n=n), jp.JP_MODE_PRIVATIZED
        wl.w = torch.from_numpy((g0.permutation(n) // 2).astype(np.int32))
    else:
        wl, mode = random_loop(9, O.OP_SAXPY, O.F32, n, null_prob=0.0), jp.JP_MODE_DOALL
        wl.w = None
    _, A, T = O.run_seq(to_oracle(wl))
    g = gpu(wl)
    L = jp.Loop.from_workload(g)
    ws = jp.workspace(L)
    res = jp.jp_schedule(L, ws)
    torch.cuda.synchronize()
    assert res["mode"] == mode and res["profiled"] == 0, res
    check_arrays(g, A, T)
    # the same loop with one bad indirect index: nothing modified
    g = gpu(wl)
    idx = g.s if case.startswith("c4") else g.r
    idx[n // 2] = 1 << 30
    A0, T0 = g.A.clone(), None if g.T is None else g.T.clone()
    L = jp.Loop.from_workload(g)
    with pytest.raises(jp.JPError) as e:
        jp.jp_schedule(L, ws)
    assert e.value.status == -5
    torch.cuda.synchronize()
    assert torch.equal(g.A, A0) and (T0 is None or torch.equal(g.T, T0))
    # a good call on the same workspace right after the aborted one (whose
    # keys were flushed before the abort): the run clears what it uses
    g = gpu(wl)
    L = jp.Loop.from_workload(g)
    res = jp.jp_schedule(L, ws)
    torch.cuda.synchronize()
    assert res["mode"] == mode and res["profiled"] == 0, res
    check_arrays(g, A, T)
    # static_check = 1: the profile decides (Fig. 2(b)), same arrays
    g = gpu(wl)
    L = jp.Loop.from_workload(g)
    res = jp.jp_schedule(L, ws, static_check=1)
    torch.cuda.synchronize()
    assert res["profiled"] == 1 and res["prof"]["raw_iters"] == 0
    check_arrays(g, A, T)


@pytest.mark.parametrize("mirror", [1, 0])
def test_structural_priv_side_stream(mirror, monkeypatch):
    """The structural privatized call returns once its index check is published
    (mapped host words; JP_STRUCT_NO_MIRROR=1: a device-to-host copy): the
    X -> Y phase is ordered on the caller's stream, so the arrays equal the
    oracle after that stream -- back-to-back calls on one workspace with
    different inputs, one of them with a bad index in between."""
    if not mirror:
        monkeypatch.setenv("JP_STRUCT_NO_MIRROR", "1")
    st = torch.cuda.Stream()
    ws = None
    for k in range(4):
        wl = synth.config4(n=(1 << 19) + 13 * k, slots=(1024, 256, 4096, 512)[k])
        _, A, T = O.run_seq(to_oracle(wl))
        g = gpu(wl)
        torch.cuda.synchronize()
        L = jp.Loop.from_workload(g)
        ws = jp.workspace(L) if ws is None or ws.numel() < jp.workspace(L).numel() else ws
        if k == 2:
            g.s[7] = -1
            A0 = g.A.clone()
            torch.cuda.synchronize()
            with pytest.raises(jp.JPError) as e:
                jp.jp_schedule(L, ws, stream=st)
            assert e.value.status == -5
            st.synchronize()
            assert torch.equal(g.A, A0)
            continue
        res = jp.jp_schedule(L, ws, stream=st)
        st.synchronize()
        assert res["mode"] == jp.JP_MODE_PRIVATIZED and res["profiled"] == 0, res
        check_arrays(g, A, T)


def test_illegal_modes_and_workspace():
    wl = synth.config1(0.05)
    g = gpu(wl)
    L = jp.Loop.from_workload(g)
    ws = jp.workspace(L)
    p = jp.jp_profile_density(L, ws)
    with pytest.raises(jp.JPError) as e:
        jp.jp_run_doall(L, p, ws)
    assert e.value.status == -4
    with pytest.raises(jp.JPError) as e:
        jp.jp_run_privatized(L, p, ws)
    assert e.value.status == -4
    small = torch.empty(1024, dtype=torch.uint8, device=DEV)
    with pytest.raises(jp.JPError) as e:
        jp.jp_profile_density(L, small)
    assert e.value.status == -3


# ---------------------------------------------------------------------------
# DOALL
# ---------------------------------------------------------------------------
@pytest.fixture(params=[0, 1], ids=["ldg128", "tma"])
def doall_kernel(request):
    """Both affine DOALL kernels (jp_doall_kernel): LDG/STG.128 stream and bulk-copy staged."""
    old = jp.jp_doall_kernel(-1)
    jp.jp_doall_kernel(request.param)
    yield request.param
    jp.jp_doall_kernel(old)


@pytest.mark.parametrize("op,dt", list(itertools.product(OPS, DTS)))
@pytest.mark.parametrize("n", [(1 << 20) + 3, 4096 * 5, 100, 4096 * 149 + 17])
def test_doall_affine(op, dt, n, doall_kernel):
    wl = random_loop(77 + op * 2 + dt, op, dt, n, null_prob=1.0)   # all indices NULL
    _, A, T = O.run_seq(to_oracle(wl))
    g = gpu(wl)
    res = jp.jp_schedule(jp.Loop.from_workload(g))
    assert res["mode"] == jp.JP_MODE_DOALL and res["profiled"] == 0
    torch.cuda.synchronize()
    check_arrays(g, A, T)


def test_doall_misaligned_scalar_path():
    n = 4099
    wl = synth.config2(n=n + 1)
    g = gpu(wl)
    A_off, X_off = g.A[1:], g.X[1:]         # 4-byte offset: not 16-byte aligned
    ref = O.Loop(1, 1, n, wl.A[1:].numpy(), X=wl.X[1:].numpy(), c0=wl.c0)
    exp = O.run_seq(ref)[1]
    jp.jp_run_doall(jp.Loop(1, 1, n, A_off, X=X_off, c0=wl.c0))
    torch.cuda.synchronize()
    assert same(A_off, exp)


@pytest.mark.parametrize("op,dt", list(itertools.product(OPS, DTS)))
def test_doall_indirect_permutation(op, dt):
    n = 50000
    g0 = np.random.default_rng(op * 10 + dt)
    wl = random_loop(5 + op * 2 + dt, op, dt, n, len_a=n, dup_writes=False, null_prob=0.0, slots=n)
    pi = torch.from_numpy(g0.permutation(n).astype(np.int32))
    wl.w = pi
    if op in (O.OP_ADD_C,):
        wl.r = pi
    if op == O.OP_STENCIL2:
        wl.r, wl.r2 = pi, pi
    if op == O.OP_PRIV_TMP:
        wl.s = torch.from_numpy(g0.permutation(n).astype(np.int32))
    ref = to_oracle(wl)
    p = O.profile(ref)
    assert (p["raw_iters"], p["war_iters"], p["waw_iters"]) == (0, 0, 0)
    _, A, T = O.run_seq(ref)
    g = gpu(wl)
    L = jp.Loop.from_workload(g)
    res = jp.jp_schedule(L, jp.workspace(L))
    if op == O.OP_PRIV_TMP:   # reading B11: RAW-free by its access sets, privatized without a profile
        assert res["mode"] == jp.JP_MODE_PRIVATIZED and res["profiled"] == 0
    else:
        assert res["mode"] == jp.JP_MODE_DOALL and res["profiled"] == 1
    torch.cuda.synchronize()
    check_arrays(g, A, T)


def test_config2_full_size_sampled(doall_kernel):
    """BASELINE size N=2^28 in the bench's launch configuration; outputs sampled
    and recomputed one by one by the oracle."""
    n = 1 << 28
    wl = synth.config2(n=n, device=DEV)
    Y0 = wl.A.clone()
    jp.jp_schedule(jp.Loop.from_workload(wl))
    torch.cuda.synchronize()
    idx = torch.cat([torch.arange(0, 4096), torch.randint(0, n, (1 << 16,), generator=torch.Generator().manual_seed(1)),
                     torch.arange(n - 4096, n)]).to(DEV)
    x, y0, y = wl.X[idx].cpu().numpy(), Y0[idx].cpu().numpy(), wl.A[idx].cpu().numpy()
    ref = O.Loop(1, 1, len(idx), y0, X=x, c0=wl.c0)
    assert y.tobytes() == O.run_seq(ref)[1].tobytes()


# ---------------------------------------------------------------------------
# privatized
# ---------------------------------------------------------------------------
@pytest.mark.parametrize("n", [1, 31, 4096 + 7, 4096 * 3, (1 << 20) + 5, 4096 * 300 + 4099])
def test_priv_config4(n, doall_kernel):
    wl = synth.config4(n=n)
    ref = to_oracle(wl)
    _, A, T = O.run_seq(ref)
    _, A2, T2 = O.sim_priv(ref)
    assert A.tobytes() == A2.tobytes() and T.tobytes() == T2.tobytes()
    g = gpu(wl)
    L = jp.Loop.from_workload(g)
    ws = jp.workspace(L)
    res = jp.jp_schedule(L, ws)
    torch.cuda.synchronize()
    if n > 1024 + 64:
        assert res["mode"] == jp.JP_MODE_PRIVATIZED
    check_arrays(g, A, T)


@pytest.mark.parametrize("op,dt,seed", [(op, dt, s) for op in OPS for dt in DTS for s in range(2)])
def test_priv_random_raw_free(op, dt, seed):
    """Random loops made RAW-free by construction: exposed reads only from
    addresses no iteration writes (or identity/self)."""
    n = 20000 + seed * 4097
    wl = random_loop(300 + op * 10 + dt * 3 + seed, op, dt, n, len_a=2 * n, null_prob=0.1,
                     slots=[7, 3000][seed])
    g0 = np.random.default_rng(seed)
    if wl.w is not None:
        wl.w = torch.from_numpy(g0.integers(0, n, size=n).astype(np.int32))      # writes in [0, n): WAW
    if op in (O.OP_ADD_C, O.OP_STENCIL2):
        wl.r = torch.from_numpy(g0.integers(n, 2 * n, size=n).astype(np.int32))  # reads in [n, 2n)
        if op == O.OP_STENCIL2:
            wl.r2 = torch.from_numpy(g0.integers(n, 2 * n, size=n).astype(np.int32))
        if wl.w is None:
            wl.w = torch.from_numpy(g0.integers(0, n, size=n).astype(np.int32))
    if op == O.OP_SAXPY and wl.w is not None:
        wl.w = torch.from_numpy(g0.permutation(2 * n)[:n].astype(np.int32))     # Y read = write: must be unique
    ref = to_oracle(wl)
    p = O.profile(ref)
    assert p["raw_iters"] == 0
    _, A, T = O.run_seq(ref)
    g = gpu(wl)
    L = jp.Loop.from_workload(g)
    ws = jp.workspace(L)
    jp.jp_run_privatized(L, None, ws)
    torch.cuda.synchronize()
    check_arrays(g, A, T)


def test_priv_split_merge_equals_whole():
    """C4: two ranges privatized into separate key tables, int64 MAX-combined,
    applied once -- equals the sequential result (global last writer)."""
    wl = synth.config4(n=(1 << 18) + 9)
    _, A, T = O.run_seq(to_oracle(wl))
    g = gpu(wl)
    rg = jp.jp_plan_sharing(wl.n, 2)
    keys = []
    for (s, e) in rg:
        L = jp.Loop(g.op, g.dtype, e - s, g.A[s:e], s=g.s[s:e], X=g.X[s:e], T=g.T, c0=g.c0, c1=g.c1, iter_base=s)
        ws = jp.workspace(L, jp.JP_WS_PRIV)
        jp.jp_priv_stream(L, {"n": e - s, "raw_iters": 0, "war_iters": 1, "waw_iters": 1, "first_raw_iter": -1,
                              "d_raw": 0.0, "d_war": 0.0, "d_waw": 0.0}, ws)
        off, nb = jp.jp_ws_region(L, "keys_T")
        keys.append(ws[off:off + nb].view(torch.int64))
    torch.cuda.synchronize()
    merged = torch.maximum(keys[0], keys[1])
    jp.jp_merge_apply(g.T, merged)
    torch.cuda.synchronize()
    check_arrays(g, A, T)


def test_config4_full_size(doall_kernel):
    """BASELINE size N=2^26 (bench launch configuration), compared in full."""
    wl = synth.config4()
    _, A, T = O.run_seq(to_oracle(wl))
    g = gpu(wl)
    L = jp.Loop.from_workload(g)
    ws = jp.workspace(L)
    res = jp.jp_schedule(L, ws)
    torch.cuda.synchronize()
    assert res["mode"] == jp.JP_MODE_PRIVATIZED
    check_arrays(g, A, T)


# ---------------------------------------------------------------------------
# TLS
# ---------------------------------------------------------------------------
def tls_case(wl, window, path, w_max=65536, with_prof=False, cluster=0, guided=False):
    ref = to_oracle(wl)
    prof_raw = O.profile(ref)["raw_iters"] if (with_prof or guided) else -1
    st, A, T, stats = O.sim_tls(ref, window, w_max, prof_raw)
    g = gpu(wl)
    L = jp.Loop.from_workload(g)
    ws = jp.workspace(L)
    p = jp.jp_profile_density(L, ws) if (with_prof or guided) else None
    if guided:
        jp.jp_tls_guide(L, ws)
    got = jp.jp_run_tls(L, window=window, w_max=w_max, path=path, prof=p, ws=ws, cluster=cluster, guided=guided)
    torch.cuda.synchronize()
    check_arrays(g, A, T)
    assert got == stats, (got, stats)
    return got


@pytest.mark.parametrize("window,path", [(32, 1), (100, 1), (1024, 1), (2048, 1), (4096, 1),
                                         (32, 2), (1000, 2), (8192, 2),
                                         (65536, 2), (32, 3), (100, 3), (1000, 3), (4096, 3), (65536, 3)])
@pytest.mark.parametrize("d", [0.0, 0.05])
def test_tls_config1(window, path, d):
    tls_case(synth.config1(d), window, path)


@pytest.mark.parametrize("d", [0.001, 0.01, 0.10])
@pytest.mark.parametrize("path", [1, 2, 3])
def test_tls_config3_reduced(d, path):
    tls_case(synth.config3(d, n=(1 << 17) + 11), 4096, path)


@pytest.mark.parametrize("op,dt,seed", [(op, dt, s) for op in OPS for dt in DTS for s in range(3)])
def test_tls_random(op, dt, seed):
    n = [200, 3000, 9001][seed]
    wl = random_loop(500 + op * 10 + dt * 3 + seed, op, dt, n, len_a=max(32, n // [1, 4, 2][seed]))
    for window, path in ((64, 1), (1000, 1), (1000, 2), (64, 3), (1000, 3)):
        tls_case(wl, window, path)


@pytest.mark.parametrize("path", [1, 2, 3])
def test_tls_adaptive(path):
    wl = synth.config3(0.01, n=1 << 16)
    w_max = 4096 if path == 1 else 65536
    tls_case(wl, 0, path, w_max=w_max, with_prof=True)
    tls_case(synth.config3(0.05, n=1 << 16), 0, path, w_max=w_max, with_prof=False)


def test_tls_gauss_seidel_and_prefix_chain():
    n = 3000
    A0 = torch.arange(n, dtype=torch.int32)
    ar = torch.arange(n, dtype=torch.int32)
    gs = synth.Workload("gs", 3, 0, n, A0.clone(), r=torch.clamp(ar - 1, min=0), r2=torch.clamp(ar + 1, max=n - 1),
                        w=ar.clone(), c0=3)
    st = tls_case(gs, 256, 1)
    assert st["windows"] == n and st["violations"] == n - 1
    pc = synth.Workload("pc", 0, 0, n, A0.clone(), r=torch.clamp(ar - 1, min=0), w=ar.clone(), c0=7)
    st = tls_case(pc, 1000, 2)
    assert st["windows"] == n and st["violations"] == n - 1


def test_config3_full_size_stats():
    """BASELINE size N=2^24 at d=1%, W=4096 (bench configuration): full arrays and stats."""
    tls_case(synth.config3(0.01), 4096, 1)
    tls_case(synth.config3(0.01), 4096, 3)


@pytest.mark.parametrize("cluster", [1, 2, 4, 8, 16])
def test_tls_cluster_sizes(cluster):
    """The cluster path at every cluster size (incl. a non power of two), fixed
    and adaptive windows, with and without the WAW commit (profile or not)."""
    wl = synth.config3(0.05, n=(1 << 15) + 77)
    for window in (96, 1000, 4096):
        if window <= 32 * (144 * cluster - 1):
            tls_case(wl, window, 3, cluster=cluster)
            tls_case(wl, window, 3, cluster=cluster, with_prof=True)
    tls_case(wl, 0, 3, w_max=4096, cluster=cluster, with_prof=True)


@pytest.mark.parametrize("op,dt", [(op, dt) for op in OPS for dt in DTS])
def test_tls_cluster_waw_unaligned(op, dt):
    """In-window WAW (many writers per address, len_A = 64) and index streams
    that are not 16-byte aligned (views starting 3 entries in): the 4-byte ring
    fill and the __match_any_sync commit groups of the cluster path."""
    n = 5000
    wl = random_loop(900 + op * 10 + dt, op, dt, n + 3, len_a=64, null_prob=0.0)
    sl = lambda t: None if t is None else t[3:]  # noqa: E731
    sub = synth.Workload("sub", wl.op, wl.dtype, n, wl.A.clone(), r=sl(wl.r), r2=sl(wl.r2), w=sl(wl.w),
                         s=sl(wl.s), X=wl.X, T=None if wl.T is None else wl.T.clone(), c0=wl.c0, c1=wl.c1)
    for window in (64, 1000):
        _, A, T, stats = O.sim_tls(to_oracle(sub), window, 65536, -1)
        g = gpu(wl)
        L = jp.Loop(wl.op, wl.dtype, n, g.A, r=sl(g.r), w=sl(g.w), r2=sl(g.r2), s=sl(g.s), X=g.X, T=g.T,
                    c0=wl.c0, c1=wl.c1)
        got = jp.jp_run_tls(L, window=window, path=3, ws=jp.workspace(L))
        torch.cuda.synchronize()
        check_arrays(g, A, T)
        assert got == stats, (window, got, stats)


def test_tls_cluster_size_must_be_pow2():
    wl = gpu(synth.config1(0.05))
    L = jp.Loop.from_workload(wl)
    with pytest.raises(jp.JPError):
        jp.jp_run_tls(L, window=64, path=3, cluster=3, ws=jp.workspace(L))


# ---------------------------------------------------------------------------
# profile-guided TLS
# ---------------------------------------------------------------------------
def guide_case(wl):
    """The guide bitmaps equal the oracle's raw flags and RAW-source flags."""
    ref = to_oracle(wl)
    g = gpu(wl)
    L = jp.Loop.from_workload(g)
    ws = jp.workspace(L)
    jp.jp_profile_density(L, ws)
    jp.jp_tls_guide(L, ws)
    torch.cuda.synchronize()
    off, nb = jp.jp_ws_region(L, "guide")
    nw = (wl.n + 31) // 32
    words = ws[off:off + 8 * nw].view(torch.int32)
    raw = bits_to_flags(words[:nw], wl.n)
    src = bits_to_flags(words[nw:], wl.n)
    assert np.array_equal(raw, O.profile(ref)["flags"] & 1)
    assert np.array_equal(src, O.raw_sources(ref))


@pytest.mark.parametrize("op,dt,seed", [(op, dt, s) for op in (O.OP_ADD_C, O.OP_SAXPY, O.OP_STENCIL2)
                                        for dt in DTS for s in range(2)])
def test_guide_bits_random(op, dt, seed):
    n = [777, 5000][seed]
    guide_case(random_loop(700 + op * 10 + dt * 3 + seed, op, dt, n, len_a=max(64, n // 3), null_prob=0.0))


@pytest.mark.parametrize("d", [0.0, 0.001, 0.05, 0.10])
def test_guide_bits_config3(d):
    guide_case(synth.config3(d, n=(1 << 16) + 9))


@pytest.mark.parametrize("path", [1, 3])
@pytest.mark.parametrize("d", [0.001, 0.01, 0.05, 0.10])
def test_tls_guided_config3_reduced(d, path):
    wl = synth.config3(d, n=(1 << 17) + 11)
    wm = 4096
    for window in (96, 1000, wm):
        tls_case(wl, window, path, guided=True)
    tls_case(wl, 0, path, w_max=wm, guided=True)


@pytest.mark.parametrize("op,dt", [(op, dt) for op in (O.OP_ADD_C, O.OP_SAXPY, O.OP_STENCIL2) for dt in DTS])
def test_tls_guided_random_waw_free(op, dt):
    """Write-once loops (w a partial permutation: no WAW) of every opcode with
    exposed reads, guided on both paths; the result equals the unguided run."""
    n = 6000
    wl = random_loop(300 + op * 10 + dt, op, dt, n, len_a=3 * n, null_prob=0.0, dup_writes=False)
    for path in (1, 3):
        for window in (64, 1500):
            tls_case(wl, window, path, guided=True)


def test_tls_guided_needs_waw_free_profile():
    wl = gpu(random_loop(5, O.OP_ADD_C, O.I32, 3000, len_a=64, null_prob=0.0))
    L = jp.Loop.from_workload(wl)
    ws = jp.workspace(L)
    p = jp.jp_profile_density(L, ws)
    assert p["waw_iters"] > 0
    with pytest.raises(jp.JPError):
        jp.jp_run_tls(L, window=64, prof=p, ws=ws, guided=True)


@pytest.mark.parametrize("d", [0.001, 0.01, 0.10])
def test_config3_full_size_guided(d):
    """BASELINE size N=2^24 through jp_schedule (profile -> guide -> TLS with restart
    recovery, tls_recovery = 1), full arrays and stats."""
    wl = synth.config3(d)
    ref = to_oracle(wl)
    g = gpu(wl)
    L = jp.Loop.from_workload(g)
    res = jp.jp_schedule(L, jp.workspace(L), tls_recovery=1)
    torch.cuda.synchronize()
    assert res["mode"] == jp.JP_MODE_TLS and res["tls_recovery"] == jp.JP_TLS_RESTART
    # the cap and path come from the profile's distance-hazard plan; the statistics
    # are reading A8's adaptive policy under that cap, exactly
    raw = O.profile(ref)["raw_iters"]
    wm = res["tls_w_max"]
    assert res["tls_path"] in (1, 2, 3) and wm >= 32
    _, A, _, stats = O.sim_tls(ref, 0, wm, raw)
    check_arrays(g, A, None)
    assert res["tls"] == stats, (res["tls"], stats)


# ---------------------------------------------------------------------------
# scheduler
# ---------------------------------------------------------------------------
def test_schedule_modes_fig2b():
    cases = [(synth.config1(0.0), jp.JP_MODE_DOALL), (synth.config1(0.05), jp.JP_MODE_TLS),
             (synth.config4(n=1 << 14), jp.JP_MODE_PRIVATIZED)]
    n = 2048
    ar = torch.arange(n, dtype=torch.int32)
    gs = synth.Workload("gs", 3, 0, n, torch.arange(n, dtype=torch.int32), r=torch.clamp(ar - 1, min=0),
                        r2=torch.clamp(ar + 1, max=n - 1), w=ar.clone(), c0=3)
    cases.append((gs, jp.JP_MODE_SEQ_RECOMMENDED))
    for wl, mode in cases:
        _, A, T = O.run_seq(to_oracle(wl))
        g = gpu(wl)
        L = jp.Loop.from_workload(g)
        res = jp.jp_schedule(L, jp.workspace(L))
        assert res["mode"] == mode, (wl.name, res)
        torch.cuda.synchronize()
        check_arrays(g, A, T)


@pytest.mark.parametrize("n,chunk", [(1 << 16, 1024), ((1 << 18), 4096), ((1 << 20), 1 << 16)])
@pytest.mark.parametrize("recovery", [0, 1])
def test_schedule_stealing_config5(n, chunk, recovery):
    """recovery 0 (auto): the write-once TLS task runs with on-chip recovery on a
    cluster beside the partitioned tasks; 1: restart recovery on one SM."""
    wl = synth.config5(n=n)
    ref = to_oracle(wl)
    _, A, T = O.run_seq(ref)
    g = gpu(wl)
    L = jp.Loop.from_workload(g)
    res = jp.jp_schedule(L, jp.workspace(L), scheme=jp.JP_SCHED_STEALING, chunk_iters=chunk, tls_recovery=recovery)
    torch.cuda.synchronize()
    check_arrays(g, A, T)
    assert res["task_mode_iters"][jp.JP_MODE_DOALL] == n // 2
    assert res["task_mode_iters"][jp.JP_MODE_TLS] == n // 4
    assert res["task_mode_iters"][jp.JP_MODE_PRIVATIZED] == n // 4
    assert res["n_batches"] == 1
    b, e = n // 2, 3 * n // 4   # the TLS task, as a loop of its own
    mid = O.Loop(ref.op, ref.dtype, e - b, ref.A, r=ref.r[b:e], w=ref.w[b:e], c0=ref.c0)
    if recovery == 0:
        assert res["tls_recovery"] == jp.JP_TLS_ONCHIP and res["tls_path"] in (5, 6, 8) and res["tls_guided"] == 1
        assert res["tls"] == O.sim_tls_fwd(mid, res["tls_w_max"])[3]
    else:
        assert res["tls_recovery"] == jp.JP_TLS_RESTART and res["tls_path"] == 1
        raw = O.profile(mid)["raw_iters"]
        assert res["tls"] == O.sim_tls(mid, 0, res["tls_w_max"], raw)[3]


def test_schedule_stealing_dependent_tasks():
    """Tasks that share addresses must be ordered (2MM/Crypt-style dependent batches)."""
    n, chunk = 1 << 14, 1024
    ar = torch.arange(n, dtype=torch.int32)
    r = ar.clone()
    w = ar.clone()
    # second half reads what the first half wrote, far back (RAW across tasks, TLS-free inside)
    r[n // 2:] = ar[: n // 2]
    w[n // 2:] = ar[n // 2:]
    wl = synth.Workload("dep", 0, 0, n, torch.arange(n, dtype=torch.int32) * 3, r=r, w=w, c0=5)
    _, A, T = O.run_seq(to_oracle(wl))
    g = gpu(wl)
    L = jp.Loop.from_workload(g)
    res = jp.jp_schedule(L, jp.workspace(L), scheme=jp.JP_SCHED_STEALING, chunk_iters=chunk)
    torch.cuda.synchronize()
    check_arrays(g, A, T)


def test_schedule_host_e2e():
    wl = synth.config1(0.05)
    _, A, _ = O.run_seq(to_oracle(wl))
    h = {k: (v.pin_memory() if v is not None else None) for k, v in wl.arrays().items()}
    L = jp.Loop(wl.op, wl.dtype, wl.n, h["A"], r=h["r"], w=h["w"], c0=wl.c0)
    stage = torch.empty(jp.jp_stage_bytes(L), dtype=torch.uint8, device=DEV)
    Ld = jp.Loop.from_workload(gpu(wl))
    ws = jp.workspace(Ld)
    res = jp.jp_schedule_host(L, stage, ws)
    assert res["mode"] == jp.JP_MODE_TLS
    assert h["A"].numpy().tobytes() == A.tobytes()


def test_launch_count_and_version():
    n0 = jp.jp_launch_count()
    g = gpu(synth.config2(n=4096))
    jp.jp_schedule(jp.Loop.from_workload(g))
    torch.cuda.synchronize()
    assert jp.jp_launch_count() == n0 + 1
    assert "sm_100a" in jp.jp_version()


@pytest.mark.parametrize("waw", [False, True])
def test_tls_cta_repeatability(waw):
    """The single-CTA window loops are timing sensitive (TLS
    barrier): run the densest reduced config-3 loop 12 times per kernel."""
    wl = synth.config3(0.10, n=(1 << 17) + 11)
    ref = to_oracle(wl)
    exp = {w: O.sim_tls(ref, w) for w in (1024, 4096)}
    prof = None
    for rep in range(12):
        for path, window in ((1, 1024), (1, 4096)):
            g = gpu(wl)
            L = jp.Loop.from_workload(g)
            ws = jp.workspace(L)
            if not waw and prof is None:
                prof = jp.jp_profile_density(L, ws)
            _, A, _, stats = exp[window]
            got = jp.jp_run_tls(L, window=window, w_max=window, path=path, prof=None if waw else prof, ws=ws)
            torch.cuda.synchronize()
            assert got == stats, (rep, path, got, stats)
            check_arrays(g, A, None)


# ---------------------------------------------------------------------------
# tiny loops: the whole schedule in one CTA (jp_tiny.cu)
# ---------------------------------------------------------------------------
def tiny_case(wl, expect_mode=None, **kw):
    """kw: jp_sched_cfg fields (tls_recovery: 0 auto = on chip for write-once
    loops, 1 restart; tls_window)."""
    ref = to_oracle(wl)
    _, A, T = O.run_seq(ref)
    p = O.profile(ref)
    g = gpu(wl)
    L = jp.Loop.from_workload(g)
    n0 = jp.jp_launch_count()
    res = jp.jp_schedule(L, jp.workspace(L), **kw)
    torch.cuda.synchronize()
    assert jp.jp_launch_count() == n0 + 1           # one launch does profile + mode + run
    check_arrays(g, A, T)
    got = (res["prof"]["raw_iters"], res["prof"]["war_iters"], res["prof"]["waw_iters"], res["prof"]["first_raw_iter"])
    assert got == (p["raw_iters"], p["war_iters"], p["waw_iters"], p["first_raw_iter"])
    if expect_mode is not None:
        assert res["mode"] == expect_mode
    if res["mode"] in (jp.JP_MODE_TLS, jp.JP_MODE_SEQ_RECOMMENDED):
        assert res["tls_path"] == 4
        onchip = p["waw_iters"] == 0 and kw.get("tls_recovery", 0) != 1
        assert res["tls_recovery"] == (jp.JP_TLS_ONCHIP if onchip else jp.JP_TLS_RESTART)
        if onchip:
            stats = O.sim_tls_fwd(ref, res["tls_w_max"])[3]
        elif kw.get("tls_window", 0) > 0:
            stats = O.sim_tls(ref, kw["tls_window"])[3]
        else:
            stats = O.sim_tls(ref, 0, res["tls_w_max"], p["raw_iters"])[3]
        assert res["tls"] == stats, (res["tls"], stats)
    return res


@pytest.mark.parametrize("d", [0.0, 0.05])
def test_tiny_config1(d):
    res = tiny_case(synth.config1(d), jp.JP_MODE_DOALL if d == 0 else jp.JP_MODE_TLS)
    if d:
        assert res["prof"]["raw_iters"] == 205


@pytest.mark.parametrize("op,dt,seed", [(op, dt, s) for op in OPS for dt in DTS for s in range(4)])
def test_tiny_random(op, dt, seed):
    """Random tiny loops of every opcode: every mode appears (duplicate writes ->
    WAW, small arrays -> RAW/WAR, permutations -> DOALL)."""
    n = [37, 1000, 4096, 3000][seed]
    la = [64, 8192, 4096, 3 * 3000][seed] if op != O.OP_PRIV_TMP else max(n, 64)
    wl = random_loop(4000 + op * 10 + dt * 5 + seed, op, dt, n, len_a=min(la, 8192), null_prob=0.15,
                     dup_writes=seed != 3, slots=[4, 64, 4096, 1000][seed])
    tiny_case(wl)


def test_tiny_modes_all_reached():
    """Fig. 2(b) branches inside the tiny kernel: DOALL, PRIVATIZED, TLS, SEQ_RECOMMENDED."""
    n = 2048
    ar = torch.arange(n, dtype=torch.int32)
    perm = torch.from_numpy(np.random.default_rng(3).permutation(n).astype(np.int32))
    cases = [(synth.Workload("doall", 0, 0, n, ar.clone(), r=perm, w=perm, c0=3), jp.JP_MODE_DOALL),
             (synth.Workload("war", 0, 0, n, ar.clone(), r=torch.clamp(ar + 1, max=n - 1), w=ar.clone(), c0=3),
              jp.JP_MODE_PRIVATIZED),
             (synth.config1(0.05), jp.JP_MODE_TLS),
             (synth.Workload("chain", 0, 0, n, ar.clone(), r=torch.clamp(ar - 1, min=0), w=ar.clone(), c0=3),
              jp.JP_MODE_SEQ_RECOMMENDED)]
    for wl, mode in cases:
        tiny_case(wl, mode)


def test_tiny_bad_index_no_side_effects():
    wl = synth.config1(0.05)
    wl.r = wl.r.clone()
    wl.r[100] = 4096   # out of range
    g = gpu(wl)
    A0 = g.A.clone()
    L = jp.Loop.from_workload(g)
    with pytest.raises(jp.JPError) as e:
        jp.jp_schedule(L, jp.workspace(L))
    assert e.value.status == -5
    torch.cuda.synchronize()
    assert torch.equal(g.A, A0)


@pytest.mark.parametrize("kw", [dict(tls_recovery=1), dict(tls_window=100), dict(tls_window=100, tls_recovery=1),
                                dict(tls_window=1)])
def test_tiny_recovery_and_windows(kw):
    """The one-CTA schedule with on-chip recovery (fixed windows) and with restart recovery."""
    res = tiny_case(synth.config1(0.05), jp.JP_MODE_TLS, **kw)
    if kw.get("tls_window"):
        assert res["tls"]["windows"] >= -(-4096 // kw["tls_window"])
    tiny_case(random_loop(41, O.OP_STENCIL2, O.F32, 3000, len_a=6000, null_prob=0.0, dup_writes=False), **kw)


@pytest.mark.parametrize("cross", [False, True])
def test_schedule_stealing_many_tasks(cross):
    """32 alternating DOALL / TLS chunk tasks (64-bit task masks; <= 8 tasks use
    byte masks): disjoint address blocks give one batch; with `cross`, each TLS
    chunk also reads what the previous DOALL chunk wrote, ordering the tasks."""
    n, chunk = 32768, 1024
    g = np.random.default_rng(9)
    r = np.empty(n, np.int32)
    w = np.empty(n, np.int32)
    for c in range(n // chunk):
        base = c * chunk
        if c % 2 == 0:   # DOALL: a permutation of the block, read = write address
            p = g.permutation(chunk).astype(np.int32) + base
            r[base:base + chunk] = p
            w[base:base + chunk] = p
        else:            # TLS: a prefix chain inside the block
            w[base:base + chunk] = np.arange(base, base + chunk, dtype=np.int32)
            r[base:base + chunk] = np.maximum(np.arange(base - 1, base + chunk - 1, dtype=np.int32), base)
            if cross:
                r[base] = base - chunk + 5   # the previous (DOALL) block's write
    wl = synth.Workload("alt", O.OP_ADD_C, O.I32, n, torch.arange(n, dtype=torch.int32) * 5,
                        r=torch.from_numpy(r), w=torch.from_numpy(w), c0=3)
    _, A, T = O.run_seq(to_oracle(wl))
    gw = gpu(wl)
    L = jp.Loop.from_workload(gw)
    res = jp.jp_schedule(L, jp.workspace(L), scheme=jp.JP_SCHED_STEALING, chunk_iters=chunk)
    torch.cuda.synchronize()
    check_arrays(gw, A, T)
    assert res["n_tasks"] == n // chunk
    assert res["n_batches"] == (2 if cross else 1)


@pytest.mark.parametrize("pass_mb", ["1", "3"])
def test_profile_address_windows(pass_mb, monkeypatch):
    """The stamp pass in L2-sized address windows (forced small with
    JP_STAMP_PASS_MB): counts and the first raw iteration equal the oracle's;
    a whole jp_schedule (fused guide bitmaps, on-chip TLS) stays exact."""
    monkeypatch.setenv("JP_STAMP_PASS_MB", pass_mb)
    for wl in (synth.config3(0.05, n=(1 << 19) + 5), synth.config5(n=1 << 19),
               random_loop(61, O.OP_STENCIL2, O.F32, 300000, len_a=1 << 19, null_prob=0.0),
               random_loop(62, O.OP_SAXPY, O.I32, 300000, len_a=1 << 19, null_prob=0.0)):
        ref = to_oracle(wl)
        pr = O.profile(ref)
        g = gpu(wl)
        L = jp.Loop.from_workload(g)
        ws = jp.workspace(L)
        p = jp.jp_profile_density(L, ws)
        assert (p["raw_iters"], p["war_iters"], p["waw_iters"], p["first_raw_iter"]) == \
            (pr["raw_iters"], pr["war_iters"], pr["waw_iters"], pr["first_raw_iter"])
        _, A, T = O.run_seq(ref)
        res = jp.jp_schedule(L, ws)
        torch.cuda.synchronize()
        check_arrays(g, A, T)
        assert res["prof"]["raw_iters"] == pr["raw_iters"]


def test_profile_config3_full_size():
    """BASELINE size (N = 2^24, tables 2 x 64 MiB: the windowed passes) against the oracle."""
    wl = synth.config3(0.05)
    pr = O.profile(to_oracle(wl))
    g = gpu(wl)
    L = jp.Loop.from_workload(g)
    p = jp.jp_profile_density(L, jp.workspace(L))
    assert (p["raw_iters"], p["war_iters"], p["waw_iters"], p["first_raw_iter"]) == \
        (pr["raw_iters"], pr["war_iters"], pr["waw_iters"], pr["first_raw_iter"])


@pytest.mark.parametrize("pairs", ["1", "0"])
@pytest.mark.parametrize("op", [O.OP_ADD_C, O.OP_SAXPY, O.OP_STENCIL2])
@pytest.mark.parametrize("seed", [3, 4])
def test_schedule_profile_interleaved_tables(op, seed, pairs, monkeypatch):
    """jp_schedule's classify pass on tables beyond 2^20 entries reads an
    interleaved {minW, minR} copy (JP_CLASSIFY_PAIRS=1, the default) or the two
    tables (0): the profile equals the oracle's either way, and so does the
    result of the mode it selects."""
    monkeypatch.setenv("JP_CLASSIFY_PAIRS", pairs)
    wl = random_loop(seed * 10 + op, op, O.F32 if op != O.OP_ADD_C else O.I32, 60001, len_a=(1 << 20) + 3)
    ref = to_oracle(wl)
    p = O.profile(ref)
    g = gpu(wl)
    L = jp.Loop.from_workload(g)
    res = jp.jp_schedule(L, jp.workspace(L), tls_recovery=1, static_check=1)
    torch.cuda.synchronize()
    assert (res["prof"]["raw_iters"], res["prof"]["war_iters"], res["prof"]["waw_iters"],
            res["prof"]["first_raw_iter"]) == (p["raw_iters"], p["war_iters"], p["waw_iters"], p["first_raw_iter"])
    _, A, T = O.run_seq(ref)
    check_arrays(g, A, T)


# ---------------------------------------------------------------------------
# mode C on the device: one warp in program order (jp_tls_cfg.path 7)
# ---------------------------------------------------------------------------
def _chain(n, op=O.OP_ADD_C, dtype=O.I32, stride=1):
    """Every iteration reads what iteration i - stride wrote (d_raw ~ 100%)."""
    ar = torch.arange(n, dtype=torch.int32)
    g = np.random.default_rng(n)
    A = torch.from_numpy(g.integers(0, 1 << 20, size=n).astype(np.int32)) if dtype == O.I32 else \
        torch.from_numpy(((g.integers(0, 2**23, size=n) * 2.0**-22) - 1).astype(np.float32))
    r = torch.clamp(ar - stride, min=0)
    if op == O.OP_STENCIL2:
        return synth.Workload("gs", op, dtype, n, A, r=r, r2=torch.clamp(ar + 1, max=n - 1), w=ar.clone(),
                              c0=float(np.float32(0.5)) if dtype == O.F32 else 3)
    return synth.Workload("chain", op, dtype, n, A, r=r, w=ar.clone(), c0=7 if dtype == O.I32 else 1.1)


@pytest.mark.parametrize("op", [O.OP_ADD_C, O.OP_SAXPY, O.OP_PRIV_TMP, O.OP_STENCIL2])
@pytest.mark.parametrize("dtype", [O.I32, O.F32])
@pytest.mark.parametrize("n,len_a,seed", [(1, 8, 1), (33, 16, 2), (1000, 64, 3), (5000, 4096, 4),
                                          (70001, 3000, 5), (40000, 1 << 16, 6)])
def test_serial_warp_matches_oracle(op, dtype, n, len_a, seed):
    """path 7 on random loops (in-batch RAW chains, WAW, identity streams):
    arrays equal the sequential oracle, stats count batches."""
    wl = random_loop(seed * 13 + op * 3 + dtype, op, dtype, n, len_a=len_a)
    ref = to_oracle(wl)
    _, A, T = O.run_seq(ref)
    g = gpu(wl)
    L = jp.Loop.from_workload(g)
    st = jp.jp_run_tls(L, path=7, ws=jp.workspace(L))
    torch.cuda.synchronize()
    check_arrays(g, A, T)
    assert st["committed"] == n and st["executed"] == n and st["windows"] == -(-n // 32)
    # violations = iterations whose exposed A read was written earlier in the same 32-iteration batch
    ix = lambda a: np.arange(n) if a is None else a.numpy().astype(np.int64)  # noqa: E731
    w = ix(wl.w)
    reads = {O.OP_ADD_C: [ix(wl.r)], O.OP_SAXPY: [w], O.OP_PRIV_TMP: [],
             O.OP_STENCIL2: [ix(wl.r), ix(wl.r2)]}[op]
    fwd = 0
    for i in range(n):
        b0 = i - i % 32
        fwd += any(np.any(w[b0:i] == rd[i]) for rd in reads)
    assert st["violations"] == fwd


@pytest.mark.parametrize("case", ["chain1", "chain3", "gs_f32", "gs_i32", "chain_saxpy"])
def test_schedule_mode_c_runs_serial(case):
    """A loop above tau_high (mode C) runs on the one-warp path through
    jp_schedule and ends in the sequential state; larger than the tiny path."""
    n = (1 << 16) + 17
    wl = {"chain1": lambda: _chain(n), "chain3": lambda: _chain(n, stride=3),
          "gs_f32": lambda: _chain(n, O.OP_STENCIL2, O.F32), "gs_i32": lambda: _chain(n, O.OP_STENCIL2, O.I32),
          "chain_saxpy": lambda: _chain(n, O.OP_SAXPY, O.F32)}[case]()
    if wl.op == O.OP_SAXPY:
        wl.X = wl.A.clone()
        wl.w = wl.r.clone()   # Y[w] = c0 X[r] + Y[w]: SAXPY reads its own write address
    ref = to_oracle(wl)
    _, A, T = O.run_seq(ref)
    g = gpu(wl)
    L = jp.Loop.from_workload(g)
    res = jp.jp_schedule(L, jp.workspace(L))
    torch.cuda.synchronize()
    check_arrays(g, A, T)
    if O.profile(ref)["raw_iters"] > 0.999 * n:
        assert res["mode"] == jp.JP_MODE_SEQ_RECOMMENDED and res["tls_path"] == 7, res
        assert res["task_mode_iters"][jp.JP_MODE_SEQ_RECOMMENDED] == n


@pytest.mark.parametrize("masks_always", ["0", "1"])
@pytest.mark.parametrize("seed", range(6))
def test_plan_tasks_matches_definition(seed, masks_always, monkeypatch):
    """jp_plan_tasks (tasks = maximal same-mode chunk runs, PDG from per-address
    task masks) against its plain definition (tests/fake_engine.py: Fig. 2(b)
    per chunk via oracle/sched.select_mode, address sets per task, pairwise
    intersection) on loops mixing DOALL / privatized / TLS regions."""
    import fake_engine as fe
    if masks_always == "1":   # skip the address-range prefilter: the masks pass decides every pair
        monkeypatch.setenv("JP_TASK_MASKS_ALWAYS", "1")
    g = np.random.default_rng(seed)
    n, chunk = 8192, 1024
    if seed % 2:
        wl = synth.config5(n=n, delta=64)
    else:
        wl = random_loop(seed, O.OP_ADD_C, O.I32, n, len_a=3 * n)
        # perturb: some chunks independent permutations (DOALL), others dense
        for k in range(0, n // chunk, 2):
            perm = torch.from_numpy((g.permutation(chunk) + k * chunk).astype(np.int32))
            wl.r[k * chunk:(k + 1) * chunk] = perm
            wl.w[k * chunk:(k + 1) * chunk] = perm
    gw = gpu(wl)
    L = jp.Loop.from_workload(gw)
    ws = jp.workspace(L)
    cc = torch.zeros(3 * (n // chunk), dtype=torch.int64, device="cuda")
    jp.jp_profile_density(L, ws, chunk_iters=chunk, chunk_counts=cc)
    tasks, conf = jp.jp_plan_tasks(L, cc.cpu(), chunk, ws)
    Lc = jp.Loop.from_workload(wl)
    et, ec = fe.jp_plan_tasks(Lc, cc.cpu(), chunk, None)
    assert tasks == et
    assert conf[:len(tasks)] == ec[:len(tasks)]


@pytest.mark.parametrize("op,dtype", [(O.OP_SAXPY, O.F32), (O.OP_ADD_C, O.I32), (O.OP_PRIV_TMP, O.F32),
                                      (O.OP_STENCIL2, O.F32)])
@pytest.mark.parametrize("n,chunk", [((1 << 22) * 3 + 77, None), (10000, "1024"), (5, "1024")])
def test_schedule_host_pipelined_doall(op, dtype, n, chunk, monkeypatch):
    """Determined-DOALL loops through jp_schedule_host: chunked H2D / kernel /
    D2H on three streams (pre-staging overlapped with execution)
    gives the sequential result, ragged last chunk included."""
    if chunk:
        monkeypatch.setenv("JP_STAGE_CHUNK", chunk)
    g = np.random.default_rng(n + op)
    el = np.int32 if dtype == O.I32 else np.float32
    mk = lambda: torch.from_numpy((g.integers(-9, 9, size=n) if dtype == O.I32  # noqa: E731
                                   else g.standard_normal(n)).astype(el))
    wl = synth.Workload("aff", op, dtype, n, mk(), X=mk() if op in (O.OP_SAXPY, O.OP_PRIV_TMP) else None,
                        T=mk() if op == O.OP_PRIV_TMP else None, c0=3 if dtype == O.I32 else 1.1, c1=0.3)
    _, A, T = O.run_seq(to_oracle(wl))
    h = {k: v.pin_memory() for k, v in wl.arrays().items()}
    L = jp.Loop(op, dtype, n, h["A"], X=h.get("X"), T=h.get("T"), c0=wl.c0, c1=wl.c1)
    stage = torch.empty(jp.jp_stage_bytes(L), dtype=torch.uint8, device=DEV)
    res = jp.jp_schedule_host(L, stage, None)
    assert res["mode"] == jp.JP_MODE_DOALL and res["profiled"] == 0
    assert h["A"].numpy().tobytes() == A.tobytes()
    if T is not None:
        assert h["T"].numpy().tobytes() == T.tobytes()


def test_schedule_stealing_mode_c_task():
    """A chunk run above tau_high becomes a mode-C task of the stealing scheme and
    runs on the one-warp program-order path beside the partitioned tasks."""
    from helpers import seq_mixed
    wl = seq_mixed(3 * 8192)
    _, A, _ = O.run_seq(to_oracle(wl))
    g = gpu(wl)
    L = jp.Loop.from_workload(g)
    res = jp.jp_schedule(L, jp.workspace(L), scheme=jp.JP_SCHED_STEALING, chunk_iters=2048)
    torch.cuda.synchronize()
    check_arrays(g, A, None)
    assert res["task_mode_iters"][jp.JP_MODE_SEQ_RECOMMENDED] == 8192 and res["tls_path"] == 7, res


@pytest.mark.skipif(shutil.which("compute-sanitizer") is None or os.environ.get("JP_RUN_SANITIZER") != "1",
                    reason="compute-sanitizer is closed on the GPU pool (runs under it left GPUs needing a reset); "
                           "JP_RUN_SANITIZER=1 runs it where allowed (profiles/r01d_sanitizers.md has the round-1 runs)")
def test_memcheck_clean():
    """compute-sanitizer memcheck over every kernel family at small N (scripts/sanitize.py):
    no out-of-bounds or misaligned access, and every case still equals the oracle."""
    root = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
    out = subprocess.run(["compute-sanitizer", "--tool", "memcheck", "--print-limit", "5", sys.executable,
                          os.path.join(root, "scripts", "sanitize.py")], capture_output=True, text=True, timeout=900)
    assert "DONE fails=0" in out.stdout, out.stdout[-2000:] + out.stderr[-2000:]
    assert "ERROR SUMMARY: 0 errors" in out.stdout + out.stderr, out.stdout[-2000:]


def test_schedule_stealing_two_grid_tls_tasks():
    """Two TLS regions (each beyond a 16-CTA cluster: the all-SM on-chip path)
    separated by DOALL regions, all on disjoint addresses: one batch whose two
    grid TLS tasks run back to back -- the first reuses the profile's pair table
    as its clean write log, the second must reset it."""
    m = 1 << 16
    parts_r, parts_w = [], []
    g = np.random.default_rng(4)
    for k in range(4):
        base = k * m
        if k % 2 == 0:
            p = torch.from_numpy((g.permutation(m) + base).astype(np.int32))
            parts_r.append(p)
            parts_w.append(p.clone())
        else:
            r, w, _ = synth.gen.dep_region(1100 + k, m, base, 0.05, 512)
            parts_r.append(r)
            parts_w.append(w)
    n = 4 * m
    A = torch.from_numpy(g.integers(0, 1 << 20, size=n).astype(np.int32))
    wl = synth.Workload("two_tls", O.OP_ADD_C, O.I32, n, A, r=torch.cat(parts_r), w=torch.cat(parts_w), c0=7)
    _, Aexp, _ = O.run_seq(to_oracle(wl))
    gw = gpu(wl)
    L = jp.Loop.from_workload(gw)
    res = jp.jp_schedule(L, jp.workspace(L), scheme=jp.JP_SCHED_STEALING, chunk_iters=4096)
    torch.cuda.synchronize()
    check_arrays(gw, Aexp, None)
    assert res["n_tasks"] == 4 and res["task_mode_iters"][jp.JP_MODE_TLS] == 2 * m and res["tls_path"] in (6, 8), res


@pytest.mark.parametrize("full", ["0", "1"])
@pytest.mark.parametrize("seed,n,slots", [(1, 5000, 64), (2, 70001, 1024), (3, 100, 4096), (4, 300000, 8192)])
def test_priv_tmp_slot_count_profile(seed, n, slots, full, monkeypatch):
    """PRIV_TMP with identity Y: war = waw = n - #slots first-written in the range,
    from the T table alone (JP_CLASSIFY_FULL=1: the classify pass) -- both equal
    the oracle, for the whole loop and for a range of it."""
    if full == "1":
        monkeypatch.setenv("JP_CLASSIFY_FULL", "1")
    g = np.random.default_rng(seed)
    wl = synth.Workload("pt", O.OP_PRIV_TMP, O.F32, n, torch.from_numpy(g.standard_normal(n).astype(np.float32)),
                        s=torch.from_numpy(g.integers(0, slots, size=n).astype(np.int32)),
                        X=torch.from_numpy(g.standard_normal(n).astype(np.float32)),
                        T=torch.from_numpy(g.standard_normal(slots).astype(np.float32)), c0=1.1, c1=0.3)
    ref = O.profile(to_oracle(wl))
    gw = gpu(wl)
    L = jp.Loop.from_workload(gw)
    p = jp.jp_profile_density(L, jp.workspace(L))
    assert (p["raw_iters"], p["war_iters"], p["waw_iters"], p["first_raw_iter"]) == \
        (ref["raw_iters"], ref["war_iters"], ref["waw_iters"], -1)
    # a range [b, e) of the loop (stamped alone: its own first writers)
    b, e = n // 3, n - n // 5
    sub = synth.Workload("pt_sub", O.OP_PRIV_TMP, O.F32, e - b, wl.A[b:e].clone(), s=wl.s[b:e].clone(),
                         X=wl.X[b:e].clone(), T=wl.T.clone(), c0=1.1, c1=0.3)
    rs = O.profile(to_oracle(sub))
    Ls = jp.Loop.from_workload(gpu(sub))
    ps = jp.jp_profile_density(Ls, jp.workspace(Ls))
    assert (ps["war_iters"], ps["waw_iters"]) == (rs["war_iters"], rs["waw_iters"])
    # ranges with iter_base > 0 whose first writers lie partly OUTSIDE the range:
    # stamp [0, b) and [b, n) into their own workspaces, MAX-combine the T tables
    # (the C1 all-reduce of profile_partitioned), classify each range; the sum is
    # the whole loop's profile
    Lw = jp.Loop.from_workload(gw)
    parts = [Lw.range(0, b), Lw.range(b, n)]
    wss = [jp.workspace(P) for P in parts]
    for P, W_ in zip(parts, wss):
        jp.jp_profile_stamp(P, W_)
    for name in ("minW_T", "minR_T"):
        offs = [jp.jp_ws_region(P, name) for P in parts]
        if offs[0][1] == 0:
            continue
        views = [W_[o:o + nb].view(torch.int32) for W_, (o, nb) in zip(wss, offs)]
        m = torch.maximum(views[0], views[1])
        for v in views:
            v.copy_(m)
    got = [jp.jp_profile_classify(P, W_) for P, W_ in zip(parts, wss)]
    assert sum(q["raw_iters"] for q in got) == 0
    assert sum(q["war_iters"] for q in got) == ref["war_iters"]
    assert sum(q["waw_iters"] for q in got) == ref["waw_iters"]


def _bucket_cases():
    n = (1 << 20) + 77
    g = np.random.default_rng(8)
    out = []
    # config 3's recipe at 5% (write-once: the guide words are defined)
    out.append(("c3", synth.config3(0.05, n=n)))
    # random ADD_C with duplicate writes and reads anywhere (WAW, WAR, RAW)
    out.append(("rand", synth.Workload("rand", O.OP_ADD_C, O.I32, n, torch.from_numpy(g.integers(0, 99, n).astype(np.int32)),
                                       r=torch.from_numpy(g.integers(0, n, n).astype(np.int32)),
                                       w=torch.from_numpy(g.integers(0, n, n).astype(np.int32)), c0=3)))
    # identity read, indirect writes into a larger A; n < len_A
    la = (1 << 21) + 5
    out.append(("r_ident", synth.Workload("r_ident", O.OP_ADD_C, O.I32, n, torch.from_numpy(g.integers(0, 99, la).astype(np.int32)),
                                          w=torch.from_numpy(g.integers(0, la, n).astype(np.int32)), c0=3)))
    # identity write, reads behind (RAW at distance <= 300)
    rr = np.maximum(np.arange(n) - g.integers(0, 300, n), 0).astype(np.int32)
    out.append(("w_ident", synth.Workload("w_ident", O.OP_ADD_C, O.I32, n, torch.from_numpy(g.integers(0, 99, n).astype(np.int32)),
                                          r=torch.from_numpy(rr), c0=3)))
    # SAXPY with indirect Y writes (raw = war = waw = "not the first writer")
    out.append(("saxpy", synth.Workload("saxpy", O.OP_SAXPY, O.F32, n, torch.from_numpy(g.standard_normal(n).astype(np.float32)),
                                        r=torch.from_numpy(g.integers(0, n, n).astype(np.int32)),
                                        w=torch.from_numpy(g.integers(0, n, n).astype(np.int32)),
                                        X=torch.from_numpy(g.standard_normal(n).astype(np.float32)), c0=1.1)))
    # in-place updates (r[i] == w[i], one access record for both) for a random
    # half of the iterations, random reads and duplicate writes for the rest
    wm = g.integers(0, n, n).astype(np.int32)
    rm = np.where(g.random(n) < 0.5, wm, g.integers(0, n, n)).astype(np.int32)
    out.append(("inplace_mix", synth.Workload("inplace_mix", O.OP_ADD_C, O.I32, n,
                                              torch.from_numpy(g.integers(0, 99, n).astype(np.int32)),
                                              r=torch.from_numpy(rm), w=torch.from_numpy(wm), c0=3)))
    return out


@pytest.mark.parametrize("buckets", ["1", "0"])
@pytest.mark.parametrize("case", range(6))
def test_schedule_bucket_profile(case, buckets, monkeypatch):
    """jp_schedule's profile of a large A by address buckets (jp_bucket.cu) --
    and, with JP_PROFILE_BUCKETS=0, the stamp/classify profile it replaces --
    against the oracle: counts, first raw iteration, the guide's raw words
    (raw flags of every iteration) and, for write-once loops, its RAW-source
    words; the arrays after the run."""
    monkeypatch.setenv("JP_PROFILE_BUCKETS", buckets)
    name, wl = _bucket_cases()[case]
    ref = to_oracle(wl)
    p = O.profile(ref)
    g = gpu(wl)
    L = jp.Loop.from_workload(g)
    ws = jp.workspace(L)
    res = jp.jp_schedule(L, ws, static_check=1, tls_recovery=1)
    torch.cuda.synchronize()
    assert (res["prof"]["raw_iters"], res["prof"]["war_iters"], res["prof"]["waw_iters"],
            res["prof"]["first_raw_iter"]) == (p["raw_iters"], p["war_iters"], p["waw_iters"], p["first_raw_iter"]), name
    off, nb = jp.jp_ws_region(L, "guide")
    nw = (wl.n + 31) // 32
    words = ws[off:off + 8 * nw].view(torch.int32)
    assert np.array_equal(bits_to_flags(words[:nw], wl.n), p["flags"] & 1), name
    if p["waw_iters"] == 0:
        assert np.array_equal(bits_to_flags(words[nw:], wl.n), O.raw_sources(ref)), name
    _, A, T = O.run_seq(ref)
    check_arrays(g, A, T)


def _gate_cases():
    n = (1 << 20) + 77
    c3 = synth.config3(0.05, n=n)
    raw = O.profile(to_oracle(c3))["raw_iters"]
    cases = _bucket_cases()
    return [("c3", c3, {}), ("doall", synth.config3(0.0, n=n), {}), ("rand_waw", cases[1][1], {}),
            ("w_ident", cases[3][1], {}), ("seq", c3, {"tau_high": 0.01}),
            ("tau_edge_tls", c3, {"tau_high": raw / n}), ("tau_edge_seq", c3, {"tau_high": (raw - 1) / n}),
            ("forced_restart", c3, {"tls_recovery": 1})]


@pytest.mark.parametrize("case", range(8))
def test_schedule_gated_path8(case, monkeypatch):
    """Path 8 launched behind the profile and gated on its header on the device
    (jp_schedule, large A): the kernel runs exactly when Fig. 2(b) gives mode B
    with war = waw = 0 -- the same result fields as the host-decided call
    (JP_NO_SPEC_FLOW=1), arrays equal to the oracle, for loops on both sides of
    the gate (DOALL, WAW, mode C, the tau_high edge, forced restart)."""
    name, wl, kw = _gate_cases()[case]
    _, A, T = O.run_seq(to_oracle(wl))
    out = []
    for spec in ("1", "0"):
        if spec == "0":
            monkeypatch.setenv("JP_NO_SPEC_FLOW", "1")
        monkeypatch.setenv("JP_FLOW_CHECK", "1")
        g = gpu(wl)
        L = jp.Loop.from_workload(g)
        ws = jp.workspace(L)
        res = jp.jp_schedule(L, ws, **kw)
        torch.cuda.synchronize()
        check_arrays(g, A, T)
        out.append(res)
    a, b = out
    assert a == b, (name, a, b)
    if name in ("c3", "w_ident", "tau_edge_tls"):
        assert a["mode_name"] == "TLS" and a["tls_path"] == 8, (name, a)
        assert a["tls"]["violations"] == a["prof"]["raw_iters"] and a["tls"]["windows"] == 1
    elif name in ("seq", "tau_edge_seq"):
        assert a["mode"] == jp.JP_MODE_SEQ_RECOMMENDED and a["tls_path"] == 7, (name, a)
    elif name == "doall":
        assert a["mode"] == jp.JP_MODE_DOALL, a
    else:
        assert a["tls_path"] != 8, (name, a)


def test_schedule_bucket_profile_bad_index():
    """An out-of-range index found by the bucket profile: JP_ERR_INDEX, nothing modified."""
    wl = synth.config3(0.01, n=(1 << 20) + 3)
    wl.r[12345] = -7
    g = gpu(wl)
    A0 = g.A.clone()
    L = jp.Loop.from_workload(g)
    for kw in (dict(), dict(scheme=jp.JP_SCHED_STEALING, chunk_iters=1 << 16)):
        with pytest.raises(jp.JPError) as e:
            jp.jp_schedule(L, jp.workspace(L), **kw)
        assert e.value.status == -5
        torch.cuda.synchronize()
        assert torch.equal(g.A, A0)


@pytest.mark.parametrize("masks_always", ["0", "1"])
def test_schedule_stealing_bucket_ranges_dependent(masks_always, monkeypatch):
    """Large A (the bucket profile) with chunks a multiple of its 16384-iteration
    tile: the task ranges come from the profile's per-chunk address ranges.  The
    second half reads what the first half wrote (a cross-task RAW): the PDG must
    order them; a third, disjoint region overlaps nothing."""
    if masks_always == "1":
        monkeypatch.setenv("JP_TASK_MASKS_ALWAYS", "1")
    q = 1 << 18
    n = 3 * q
    ar = torch.arange(n, dtype=torch.int32)
    g0 = np.random.default_rng(12)
    w = ar.clone()
    r = ar.clone()
    r[q:2 * q] = torch.from_numpy(g0.permutation(q).astype(np.int32))   # reads the first region's writes
    w[2 * q:] = torch.from_numpy((2 * q + g0.permutation(q)).astype(np.int32))
    r[2 * q:] = w[2 * q:]
    wl = synth.Workload("dep_big", O.OP_ADD_C, O.I32, n, torch.from_numpy(g0.integers(0, 99, n + (1 << 20)).astype(np.int32)),
                        r=r, w=w, c0=5)
    _, A, _ = O.run_seq(to_oracle(wl))
    g = gpu(wl)
    L = jp.Loop.from_workload(g)
    res = jp.jp_schedule(L, jp.workspace(L), scheme=jp.JP_SCHED_STEALING, chunk_iters=1 << 16)
    torch.cuda.synchronize()
    check_arrays(g, A, None)
    assert res["n_batches"] == 2, res
