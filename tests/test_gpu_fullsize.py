"""GPU parity at BASELINE.json's full sizes, in the launch configurations
bench.py times, compared with the oracle element by element (every output
byte), plus the multi-trip (grid-stride) path of the indirect DOALL kernel at
n >= 2^23 for every opcode and dtype.

Expected values come only from oracle/ (jpo_run_seq in C, one host thread) on
the same seeded inputs (synth/).  Bar: byte equality (reading A12: two RN ops,
no contraction, on both sides; reading A11: int32 wraps).
"""
import itertools

import numpy as np
import pytest
import torch

import oracle as O
import synth
from helpers import random_loop, to_oracle

pytestmark = pytest.mark.gpu

if torch.cuda.is_available():
    import paper_conf_icpp_hanzlw13_b200 as jp
    import paper_conf_icpp_hanzlw13_b200.dist as jd
    DEV = torch.device("cuda:0")
else:  # collected on CPU boxes, never run there
    jp = jd = None
    DEV = None

OPS = [O.OP_ADD_C, O.OP_SAXPY, O.OP_PRIV_TMP, O.OP_STENCIL2]
DTS = [O.I32, O.F32]


def equal_bytes(t: torch.Tensor, a: np.ndarray) -> bool:
    return torch.equal(t.cpu().view(torch.int32), torch.from_numpy(a.view(np.int32)))


def first_diff(t: torch.Tensor, a: np.ndarray):
    return np.flatnonzero(t.cpu().numpy().view(np.int32) != a.view(np.int32))[:10]


@pytest.fixture(params=[0, 1], ids=["ldg128", "tma"])
def doall_kernel(request):
    old = jp.jp_doall_kernel(-1)
    jp.jp_doall_kernel(request.param)
    yield request.param
    jp.jp_doall_kernel(old)


def test_config2_full_size_every_byte(doall_kernel):
    """Config 2 (SAXPY fp32, N = 2^28, X and Y 1 GiB each) through jp_schedule,
    the bench's step: all 2^28 outputs against jpo_run_seq."""
    n = 1 << 28
    wl = synth.config2(n=n, device=DEV)
    ref = O.Loop(O.OP_SAXPY, O.F32, n, wl.A.cpu().numpy(), X=wl.X.cpu().numpy(), c0=wl.c0)
    res = jp.jp_schedule(jp.Loop.from_workload(wl))
    torch.cuda.synchronize()
    assert res["mode"] == jp.JP_MODE_DOALL and res["profiled"] == 0
    st, Y, _ = O.run_seq(ref)
    assert st == O.OK
    assert equal_bytes(wl.A, Y), first_diff(wl.A, Y)


@pytest.mark.parametrize("recovery", [0, 1])
def test_config5_full_size_schedule(recovery):
    """Config 5 (N = 2^24: DOALL head 2^23, TLS middle 2^22 at 5%, privatized
    tail 2^22) through jp_schedule(STEALING), the bench's call: every byte of A."""
    wl = synth.config5()
    n = wl.n
    ref = to_oracle(wl)
    g = wl.to(DEV)
    L = jp.Loop.from_workload(g)
    res = jp.jp_schedule(L, jp.workspace(L), scheme=jp.JP_SCHED_STEALING, chunk_iters=1 << 16,
                         tls_recovery=recovery)
    torch.cuda.synchronize()
    _, A, _ = O.run_seq(ref)
    assert equal_bytes(g.A, A), first_diff(g.A, A)
    assert res["task_mode_iters"] == [n // 2, n // 4, n // 4, 0], res
    b, e = n // 2, 3 * n // 4
    mid = O.Loop(ref.op, ref.dtype, e - b, ref.A, r=ref.r[b:e], w=ref.w[b:e], c0=ref.c0)
    if recovery == 0:
        assert res["tls"] == O.sim_tls_fwd(mid, res["tls_w_max"])[3]
    else:
        assert res["tls"] == O.sim_tls(mid, 0, res["tls_w_max"], O.profile(mid)["raw_iters"])[3]


@pytest.mark.parametrize("dynamic,force", [(False, False), (False, True), (True, False)])
def test_config5_full_size_dist_world1(dynamic, force):
    """Config 5 at N = 2^24 through the multi-rank stealing driver at world 1
    (the bench's partitioned row; force: the multi-rank path instead of the
    one-rank delegation to jp_schedule): every byte of A."""
    wl = synth.config5()
    ref = to_oracle(wl)
    g = wl.to(DEV)
    L = jp.Loop.from_workload(g)
    res = jd.schedule_stealing(L, jp.workspace(L), chunk_iters=1 << 16, dynamic=dynamic, force_ranks=force)
    assert ("delegated" in res) == (not dynamic and not force)
    torch.cuda.synchronize()
    _, A, _ = O.run_seq(ref)
    assert equal_bytes(g.A, A), first_diff(g.A, A)
    p = O.profile(ref)
    assert (res["prof"]["raw_iters"], res["prof"]["war_iters"], res["prof"]["waw_iters"]) == \
        (p["raw_iters"], p["war_iters"], p["waw_iters"])


@pytest.mark.parametrize("generic", ["0", "1"])
@pytest.mark.parametrize("op,dt", list(itertools.product(OPS, DTS)))
def test_doall_indirect_multi_trip(op, dt, generic, monkeypatch):
    """k_doall_quad / k_doall_generic beyond one grid's worth of iterations
    (n = 2^23 + 2^21 + 5: several grid-stride trips plus a ragged tail), every
    opcode and dtype, dependence-free indirect loops (permutation writes)."""
    if generic == "1":
        monkeypatch.setenv("JP_DOALL_GENERIC", "1")
    n = (1 << 23) + (1 << 21) + 5
    g0 = np.random.default_rng(1000 + op * 2 + dt)
    wl = random_loop(7 + op * 2 + dt, op, dt, n, len_a=n, dup_writes=False, null_prob=0.0, slots=n)
    pi = torch.from_numpy(g0.permutation(n).astype(np.int32))
    wl.w = pi
    if op == O.OP_ADD_C:
        wl.r = pi
    if op == O.OP_STENCIL2:
        wl.r, wl.r2 = pi, pi
    if op == O.OP_PRIV_TMP:
        wl.s = torch.from_numpy(g0.permutation(n).astype(np.int32))
    ref = to_oracle(wl)
    _, A, T = O.run_seq(ref)
    g = wl.to(DEV)
    L = jp.Loop.from_workload(g)
    res = jp.jp_schedule(L, jp.workspace(L), static_check=1)   # profiled: Fig. 2(b) picks DOALL
    torch.cuda.synchronize()
    assert res["mode"] == jp.JP_MODE_DOALL and res["prof"]["raw_iters"] == 0
    assert equal_bytes(g.A, A), first_diff(g.A, A)
    if T is not None:
        assert equal_bytes(g.T, T)


@pytest.mark.parametrize("d,delta", [(0.01, 1024), (0.10, 1024), (0.01, 1 << 20), (0.10, 1 << 20)])
def test_config3_waw_full_size_restart(d, delta):
    """Config 3's shape with write-after-write (on-chip recovery illegal), N = 2^24,
    through jp_schedule with tls_recovery = 1 -- the bench's config3_waw restart
    rows: restart TLS under the distance-steered cap; every byte of A and the
    statistics of jpo_sim_tls under that cap (the default call runs path 9,
    tests/test_gpu_flow_waw.py)."""
    wl = synth.config3_waw(d, delta=delta)
    ref = to_oracle(wl)
    g = wl.to(DEV)
    L = jp.Loop.from_workload(g)
    res = jp.jp_schedule(L, jp.workspace(L), tls_recovery=1)
    torch.cuda.synchronize()
    assert res["mode"] == jp.JP_MODE_TLS and res["tls_recovery"] == jp.JP_TLS_RESTART, res
    p = O.profile(ref)
    assert (res["prof"]["raw_iters"], res["prof"]["waw_iters"]) == (p["raw_iters"], p["waw_iters"])
    st, A, _, stats = O.sim_tls(ref, 0, res["tls_w_max"], p["raw_iters"])
    assert equal_bytes(g.A, A), first_diff(g.A, A)
    assert res["tls"] == stats, (res["tls"], stats)


@pytest.mark.parametrize("split", [3, 5])
def test_schedule_ranges_of_config3(split):
    """A loop run as consecutive ranges (iter_base = ident_off = the range start),
    each through jp_schedule on the shared arrays -- the address-bucket profile,
    Fig. 2(b) and the one-window on-chip TLS of every range use global ids; the
    final A is the sequential one (ranges in order = program order)."""
    n = (1 << 21) + 13
    wl = synth.config3(0.05, n=n)
    _, A, _ = O.run_seq(to_oracle(wl))
    g = wl.to(DEV)
    full = jp.Loop.from_workload(g)
    cuts = [n * k // split for k in range(split + 1)]
    for b, e in zip(cuts[:-1], cuts[1:]):
        part = full.range(b, e)
        res = jp.jp_schedule(part, jp.workspace(part))
        torch.cuda.synchronize()
        assert res["mode"] in (jp.JP_MODE_TLS, jp.JP_MODE_DOALL, jp.JP_MODE_PRIVATIZED), res
    assert equal_bytes(g.A, A), first_diff(g.A, A)
