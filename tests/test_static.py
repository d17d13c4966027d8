"""Static analysis lite.

CPU: the exact affine dependence test (jp_affine_dependence, host-only C)
against a brute force over all pairs i != j.  GPU: jp_static_check's affine
detection and independence verdict against numpy and the oracle's pair
enumeration (jpo_pairs: a loop is conflict-free iff it has no RAW, WAR or WAW
pair), and jp_schedule running such loops as DOALL without a profile.
"""
import itertools

import numpy as np
import pytest
import torch

import oracle as O
import synth
import paper_conf_icpp_hanzlw13_b200 as jp
from helpers import to_oracle


def brute(af, bf, ag, bg, n):
    f = {af * i + bf: i for i in range(n)}
    gs = {}
    for j in range(n):
        gs.setdefault(ag * j + bg, []).append(j)
    for i in range(n):
        for j in gs.get(af * i + bf, []):
            if i != j:
                return True
    return False


def test_affine_dependence_exhaustive_small():
    for af, ag in itertools.product(range(-3, 4), repeat=2):
        for bf, bg in itertools.product(range(-6, 7), repeat=2):
            for n in (0, 1, 2, 3, 7):
                assert jp.jp_affine_dependence(af, bf, ag, bg, n) == brute(af, bf, ag, bg, n), (af, bf, ag, bg, n)


def test_affine_dependence_random_large():
    g = np.random.default_rng(4)
    for _ in range(3000):
        af, ag = (int(x) for x in g.integers(-40, 41, 2))
        bf, bg = (int(x) for x in g.integers(-500, 501, 2))
        n = int(g.integers(1, 60))
        assert jp.jp_affine_dependence(af, bf, ag, bg, n) == brute(af, bf, ag, bg, n), (af, bf, ag, bg, n)


def test_affine_dependence_big_values():
    # i - j = 2^30: conflict iff n > 2^30
    assert jp.jp_affine_dependence(1, 0, 1, 1 << 30, (1 << 30) + 1)
    assert not jp.jp_affine_dependence(1, 0, 1, 1 << 30, 1 << 30)
    # 3i = 5j + 1 has solutions (i, j) = (2, 1), (7, 4), ...
    assert jp.jp_affine_dependence(3, 0, 5, 1, 3)
    assert not jp.jp_affine_dependence(3, 0, 5, 1, 2)
    # 2i = 2j + 1: parity, never
    assert not jp.jp_affine_dependence(2, 0, 2, 1, 1 << 30)


# ---------------------------------------------------------------------------
# GPU
# ---------------------------------------------------------------------------
OPS = [O.OP_ADD_C, O.OP_SAXPY, O.OP_PRIV_TMP, O.OP_STENCIL2]


def affine_loop(seed, op, n):
    g = np.random.default_rng(seed)
    la = 4 * n + 64

    def arr():
        if g.random() < 0.2:
            return None
        a = int(g.integers(-3, 4))
        b = int(g.integers(0, la)) if a >= 0 else int(g.integers(0, la))
        if g.random() < 0.15:   # sometimes out of range on purpose
            b = la - 1 if a > 0 else 0 if a < 0 else b
        return torch.from_numpy((a * np.arange(n, dtype=np.int64) + b).astype(np.int32))
    r, w = arr(), arr()
    r2 = arr() if op == O.OP_STENCIL2 else None
    s = arr() if op == O.OP_PRIV_TMP else None
    A0 = torch.from_numpy(g.integers(-1000, 1000, la).astype(np.int32))
    X = torch.from_numpy(g.integers(-1000, 1000, la).astype(np.int32)) if op in (O.OP_SAXPY, O.OP_PRIV_TMP) else None
    T = torch.zeros(la, dtype=torch.int32) if op == O.OP_PRIV_TMP else None
    return synth.Workload("affine", op, O.I32, n, A0, r=r, r2=r2, w=w, s=s, X=X, T=T, c0=3, c1=2)


@pytest.mark.gpu
@pytest.mark.parametrize("op", OPS)
def test_static_check_random_affine(op):
    dev = torch.device("cuda:0")
    for seed in range(40):
        n = [1, 2, 5, 37, 300, 1000][seed % 6]
        wl = affine_loop(1000 * op + seed, op, n)
        g = wl.to(dev)
        L = jp.Loop.from_workload(g)
        ws = jp.workspace(L)
        s = jp.jp_static_check(L, ws)
        assert s["affine"] == 1
        for q, t in enumerate((wl.r, wl.r2, wl.w, wl.s)):
            if t is not None:
                assert s["beta"][q] == int(t[0]) and (n == 1 or s["alpha"][q] == int(t[1]) - int(t[0]))
        ref = to_oracle(wl)
        inr = O.run_seq(ref)[0] == O.OK
        assert s["in_range"] == int(inr), (seed, s)
        if inr:
            pr = O.pairs(ref)
            free = pr["raw_pairs"] == 0 and pr["war_pairs"] == 0 and pr["waw_pairs"] == 0
            assert s["independent"] == int(free), (seed, s, pr)


@pytest.mark.gpu
def test_static_check_not_affine_and_schedule():
    dev = torch.device("cuda:0")
    # a permutation is not affine: the profiler decides
    wl = synth.config1(0.0)
    L = jp.Loop.from_workload(wl.to(dev))
    assert jp.jp_static_check(L, jp.workspace(L))["affine"] == 0
    # stride-2 read / write halves: affine, conflict-free -> DOALL without a profile
    n = 1 << 20
    i = torch.arange(n, dtype=torch.int32)
    wl = synth.Workload("even_odd", O.OP_ADD_C, O.I32, n, torch.arange(2 * n, dtype=torch.int32),
                        r=2 * i + 1, w=2 * i, c0=5)
    _, A, _ = O.run_seq(to_oracle(wl))
    for sc, profiled in ((0, 0), (1, 1)):
        g = wl.to(dev)
        L = jp.Loop.from_workload(g)
        res = jp.jp_schedule(L, jp.workspace(L), static_check=sc)
        torch.cuda.synchronize()
        assert res["mode"] == jp.JP_MODE_DOALL and res["profiled"] == profiled
        assert g.A.cpu().numpy().tobytes() == A.tobytes()
    # shifted read of the written range (i reads i-1's write): affine but dependent -> profiled, TLS
    wl = synth.Workload("shift", O.OP_ADD_C, O.I32, 5000, torch.arange(6000, dtype=torch.int32),
                        r=torch.arange(5000, dtype=torch.int32), w=torch.arange(1, 5001, dtype=torch.int32), c0=1)
    _, A, _ = O.run_seq(to_oracle(wl))
    g = wl.to(dev)
    L = jp.Loop.from_workload(g)
    s = jp.jp_static_check(L, jp.workspace(L))
    assert s["affine"] == 1 and s["independent"] == 0
    res = jp.jp_schedule(L, jp.workspace(L))
    torch.cuda.synchronize()
    assert res["profiled"] == 1 and res["mode"] in (jp.JP_MODE_TLS, jp.JP_MODE_SEQ_RECOMMENDED)
    assert g.A.cpu().numpy().tobytes() == A.tobytes()
