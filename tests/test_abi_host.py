"""CPU-side checks of the C ABI (-m "not gpu"): libjp.so loads, exports every
symbol include/jp.h declares, and its host-only logic (workspace layout, the
Fig. 2(b) decision, the task-sharing / task-stealing plans) matches the plain
restatements in oracle/sched.py.  No compute call is made without a GPU, except
to check that one fails loudly with JP_ERR_CUDA (no CPU fallback)."""
import ctypes as C
import os
import random
import re

import numpy as np
import pytest
import torch

import oracle as O
import oracle.sched as S
import paper_conf_icpp_hanzlw13_b200 as jp
from paper_conf_icpp_hanzlw13_b200 import _abi

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def header_functions():
    src = open(os.path.join(ROOT, "include", "jp.h")).read()
    src = re.sub(r"/\*.*?\*/", "", src, flags=re.S)
    return sorted(set(re.findall(r"\b(jp_[a-z0-9_]+)\s*\(", src)))


def test_library_exports_every_header_symbol():
    lib = jp.lib()
    names = header_functions()
    assert len(names) >= 20
    for name in names:
        assert hasattr(lib, name), name
    assert sorted(n for n, _, _ in _abi.SIGNATURES) == names


def test_version_and_launch_counter():
    assert "sm_100a" in jp.jp_version()
    assert jp.jp_launch_count() >= 0


def cpu_loop(op=0, n=1000, la=1000, r=True, w=True, s=False, lt=16):
    A = torch.zeros(la, dtype=torch.int32)
    idx = torch.zeros(n, dtype=torch.int32)
    return jp.Loop(op, 0, n, A, r=idx if r else None, w=idx if w else None, s=idx if s else None,
                   X=torch.zeros(max(n, 8), dtype=torch.int32) if op in (1, 2) else None,
                   T=torch.zeros(lt, dtype=torch.int32) if op == 2 else None)


def test_workspace_layout_fixed_offsets():
    L = cpu_loop()
    sizes = {u: jp.jp_workspace_bytes(L, u) for u in (0, 1, 2, 4, 8, 15, 16, 31)}
    assert sizes[0] == 4096
    assert sizes[1] < sizes[2] < sizes[4] < sizes[8] == sizes[15] < sizes[16] == sizes[31]
    # regions are disjoint, 256-aligned and inside the total
    spans = []
    for name in _abi.REGIONS:
        off, nb = jp.jp_ws_region(L, name)
        assert off % 256 == 0
        if nb:
            spans.append((off, off + nb))
            assert off + nb <= sizes[31]
    spans.sort()
    for a, b in zip(spans, spans[1:]):
        assert a[1] <= b[0]
    # identity-only arrays need no tables
    La = cpu_loop(r=False, w=False)
    assert jp.jp_ws_region(La, "minW_A")[1] == 0 and jp.jp_ws_region(La, "keys_A")[1] == 0
    Lt = cpu_loop(op=2, r=False, w=False, s=True, lt=1024)
    assert jp.jp_ws_region(Lt, "minW_T")[1] == 4 * 1024 and jp.jp_ws_region(Lt, "keys_T")[1] == 8 * 1024
    assert jp.jp_ws_region(Lt, "keys_A")[1] == 0
    # guide regions: maxRx over A and two bitmaps of ceil(n/32) words (opcodes with exposed A reads)
    assert jp.jp_ws_region(L, "maxRx_A")[1] == 4 * 1000 and jp.jp_ws_region(L, "guide")[1] == 8 * 32
    assert jp.jp_ws_region(Lt, "guide")[1] == 0


@pytest.mark.parametrize("seed", range(200))
def test_select_mode_matches_fig2b(seed):
    g = random.Random(seed)
    n = g.choice([1, 100, 4096])
    raw = g.choice([0, 0, 1, n // 100, n // 10, n // 3, n])
    war, waw = g.choice([0, 0, 5]), g.choice([0, 0, 7])
    all_null = g.random() < 0.15
    L = cpu_loop(r=not all_null, w=not all_null)
    p = {"n": n, "raw_iters": raw, "war_iters": war, "waw_iters": waw, "first_raw_iter": -1,
         "d_raw": raw / n, "d_war": war / n, "d_waw": waw / n}
    tau = g.choice([0.25, 0.05, 0.5])
    assert jp.jp_select_mode(L, p, tau) == S.select_mode(all_null, n, raw, war, waw, tau)


def test_select_mode_paper_cases():
    """P:L624-629 (BlackScholes, DD ~ 0.012 -> GPU-TLS, mode B)
    (CFD/Sepia: no TD, some FD -> mode D); P:L611-613 (Gauss-Seidel, high -> C)."""
    L = cpu_loop()
    mk = lambda n, r, a, b: {"n": n, "raw_iters": r, "war_iters": a, "waw_iters": b, "first_raw_iter": -1,  # noqa
                             "d_raw": r / n, "d_war": a / n, "d_waw": b / n}
    assert jp.jp_select_mode(L, mk(1000, 12, 0, 0)) == jp.JP_MODE_TLS
    assert jp.jp_select_mode(L, mk(1000, 0, 900, 900)) == jp.JP_MODE_PRIVATIZED
    assert jp.jp_select_mode(L, mk(10000, 9999, 9999, 0)) == jp.JP_MODE_SEQ_RECOMMENDED   # Gauss-Seidel
    assert jp.jp_select_mode(L, mk(1000, 999, 999, 0)) == jp.JP_MODE_TLS   # 0.999: not above tau_high
    assert jp.jp_select_mode(L, mk(1000, 0, 0, 0)) == jp.JP_MODE_DOALL
    assert jp.jp_select_mode(cpu_loop(r=False, w=False), None) == jp.JP_MODE_DOALL


def test_boundary_formula_paper_hardware():
    """P:L354-358 with the paper's platform: 12 cores at 2.66 GHz
    and 448 GPU cores; the M2050 clock 1.15 GHz is NOT in the paper (external)."""
    b = S.boundary(448, 1.15, 12, 2.66)
    assert abs(b - 515.2 / 547.12) < 1e-12
    n = 10_000_000
    rg = jp.jp_plan_sharing(n, 2, [448 * 1.15, 12 * 2.66])
    assert rg[0] == (0, int(n * b)) and rg[1] == (int(n * b), n)


@pytest.mark.parametrize("seed", range(50))
def test_plan_sharing_matches_oracle(seed):
    g = random.Random(seed)
    world = g.randint(1, 8)
    n = g.choice([0, 1, 7, 1 << 28, g.randint(0, 10**9)])
    weights = None if g.random() < 0.3 else [g.uniform(0.1, 5.0) for _ in range(world)]
    got = jp.jp_plan_sharing(n, world, weights)
    assert got == S.sharing_ranges(n, weights or [1.0] * world)
    assert got[0][0] == 0 and got[-1][1] == n
    for a, b in zip(got, got[1:]):
        assert a[1] == b[0]
    if weights is None and n % world == 0:
        assert all(e - s == n // world for s, e in got)   # closed form 1/k on identical GPUs


@pytest.mark.parametrize("seed", range(60))
def test_plan_stealing_matches_oracle(seed):
    g = random.Random(seed)
    world = g.randint(1, 8)
    pos, tasks = 0, []
    for _ in range(g.randint(1, 6)):
        ln = g.randint(1, 50000)
        tasks.append((pos, pos + ln, g.choice([0, 0, 1, 2])))
        pos += ln
    chunk = g.choice([1024, 4096, 65536])
    speed = None if g.random() < 0.4 else [g.uniform(0.5, 3.0) for _ in range(world)]
    st = g.uniform(0.01, 1.0)
    got, stolen = jp.jp_plan_stealing(tasks, world, chunk, speed, st)
    exp, estolen = S.stealing_plan(tasks, world, chunk, speed, st)
    assert got == exp and stolen == estolen
    # every iteration of every task is owned exactly once; TLS stays on rank 0
    cover = sorted((c[0], c[1]) for c in got)
    assert cover[0][0] == 0 and cover[-1][1] == pos
    for a, b in zip(cover, cover[1:]):
        assert a[1] == b[0]
    assert all(c[3] == 0 for c in got if c[2] == 2)
    assert all(0 <= c[3] < world for c in got)


def test_stealing_bicg_mechanism():
    """P:L633-641 (BICG): eight equal sub-loops all land in one queue at first;
    the empty worker gets one and then steals.  Two equal-speed workers here:
    the mechanism (dealing + tail stealing) must leave both busy.  The paper's
    62.5% CPU share depends on unreported speeds: parity unpinned."""
    tasks = [(k * 1000, (k + 1) * 1000, 0) for k in range(8)]
    chunks, stolen = jp.jp_plan_stealing(tasks, 2, 1000, [1.0, 1.0], 1.0)
    owners = [c[3] for c in chunks]
    assert owners.count(0) == owners.count(1) == 4 and stolen == 0
    chunks, stolen = jp.jp_plan_stealing(tasks, 2, 1000, [3.0, 1.0], 1.0)
    owners = [c[3] for c in chunks]
    assert owners.count(0) > owners.count(1)   # faster worker ends up with more sub-loops
    # a TLS task pinned to rank 0 makes rank 1 steal rank 0's DOALL chunks
    tasks = [(0, 8000, 2)] + [(8000 + k * 1000, 9000 + k * 1000, 0) for k in range(8)]
    chunks, stolen = jp.jp_plan_stealing(tasks, 2, 1000, [1.0, 1.0], 1.0)
    assert stolen >= 3 and sum(1 for c in chunks if c[3] == 1) >= 7


@pytest.mark.skipif(torch.cuda.is_available(), reason="checks the no-GPU failure path")
def test_compute_calls_fail_loudly_without_gpu():
    L = cpu_loop()
    with pytest.raises(jp.JPError) as e:
        jp.jp_run_doall(L)
    assert e.value.status == _abi.JP_ERR_CUDA
    with pytest.raises(jp.JPError) as e:
        jp.jp_schedule(L, torch.zeros(1 << 20, dtype=torch.uint8))
    assert e.value.status == _abi.JP_ERR_CUDA
    Y = torch.zeros(64, dtype=torch.float32)
    with pytest.raises(jp.JPError) as e:
        jp.jp_run_doall_spill([jp.Loop(1, 1, 64, Y, X=Y.clone(), c0=2.0)], 0, 16, torch.zeros(1, dtype=torch.int64))
    assert e.value.status == _abi.JP_ERR_CUDA
    t = torch.zeros(100, dtype=torch.int32)
    with pytest.raises(jp.JPError) as e:
        jp.jp_sparse_pack(t, None, -1, 2)
    assert e.value.status == _abi.JP_ERR_CUDA
    with pytest.raises(jp.JPError) as e:
        jp.jp_sparse_reduce_max(t, None, torch.zeros((3, 2), dtype=torch.int32))
    assert e.value.status == _abi.JP_ERR_CUDA


def test_sparse_exchange_bad_arguments():
    """Argument errors of the NEXT-2 entry points are decided on the host."""
    lib = _abi.lib()
    cnt = (C.c_int64 * 2)()
    buf = C.create_string_buffer(1 << 12)
    p = C.addressof(buf)
    assert lib.jp_sparse_pack(p, None, 3, 10, 0, 10, -1, 2, p, 10, cnt, p, 4096, None) == _abi.JP_ERR_ARG
    assert lib.jp_sparse_pack(p, None, 4, 10, 5, 11, -1, 2, p, 10, cnt, p, 4096, None) == _abi.JP_ERR_ARG
    assert lib.jp_sparse_pack(p, None, 4, 10, 0, 10, -1, 0, p, 10, cnt, p, 4096, None) == _abi.JP_ERR_ARG
    assert lib.jp_sparse_pack(p, None, 4, 10, 0, 10, -1, 2, p, 10, cnt, p, 0, None) == _abi.JP_ERR_WORKSPACE
    assert lib.jp_sparse_pack(p, None, 4, 1 << 31, 0, 10, -1, 2, p, 10, cnt, p, 4096, None) == _abi.JP_ERR_ARG
    assert lib.jp_sparse_reduce_max(p, None, 8, 10, p, -1, None) == _abi.JP_ERR_ARG
    assert lib.jp_sparse_gather(None, None, 4, 10, p, 3, None) == _abi.JP_ERR_ARG
    assert lib.jp_sparse_scatter(p, None, 4, 10, None, 3, None) == _abi.JP_ERR_ARG
    assert lib.jp_sparse_scratch_bytes(1 << 24, 8) >= 8 * (2 * ((1 << 24) // 4096) + 8)
    assert lib.jp_sparse_scratch_bytes(-1, 8) == 0


def test_bad_arguments():
    with pytest.raises(jp.JPError) as e:
        jp.jp_plan_sharing(10, 2, [0.0, 0.0])
    assert e.value.status == _abi.JP_ERR_ARG
    A = torch.zeros(10, dtype=torch.int32)
    L = jp.Loop(0, 0, 11, A)          # identity index past len_A
    with pytest.raises(jp.JPError) as e:
        jp.jp_ws_region(L, "header")
    assert e.value.status == _abi.JP_ERR_INDEX


@pytest.mark.parametrize("n,raw", [(1 << 24, 16777), (1 << 24, 167772), (1 << 24, 1677722), (4096, 205), (100, 0),
                                   (100, -1), (1000, 3), (7, 7), (1 << 20, 1)])
def test_tls_next_window_matches_oracle(n, raw):
    """The library's reading-A8 policy (the C function every TLS kernel uses)
    equals the oracle's, for the first window and for every step."""
    for w_max in (32, 4096, 65536):
        assert jp.jp_tls_next_window(n, raw, -1, w_max) == O.tls_next_window(n, raw, -1, w_max)
        for prev in (0, 1, 15, 16, 17, 100, 4095, 4096, 70000):
            assert jp.jp_tls_next_window(n, raw, prev, w_max) == O.tls_next_window(n, raw, prev, w_max)
    assert jp.jp_tls_next_window(-1, raw, -1, 4096) == -1
    assert jp.jp_tls_next_window(n, raw, -1, 16) == -1


@pytest.mark.parametrize("seed", range(12))
def test_plan_matches_oracle_composition(seed):
    """jp_plan (host split plan of SURVEY 8(b)): chunk modes by Fig. 2(b), maximal
    same-mode runs, then the sharing split or the Alg. 1 plan -- against the
    oracle's select_mode / sharing_ranges / stealing_plan composed in Python."""
    import oracle.sched as OS
    g = np.random.default_rng(seed)
    chunk = 1024
    nck = int(g.integers(1, 40))
    n = nck * chunk - int(g.integers(0, chunk))
    world = int(g.integers(1, 5))
    profs, modes = [], []
    for k in range(nck):
        m = min(chunk, n - k * chunk)
        kind = g.integers(0, 4)
        raw = 0 if kind in (0, 1) else int(g.integers(1, m // 2 if kind == 2 else m))
        war = int(g.integers(0, m)) if kind == 1 else 0
        waw = int(g.integers(0, m)) if kind == 1 else 0
        profs.append({"n": m, "raw_iters": raw, "war_iters": war, "waw_iters": waw, "first_raw_iter": -1,
                      "d_raw": raw / m, "d_war": war / m, "d_waw": waw / m})
        modes.append(OS.select_mode(False, m, raw, war, waw, 0.25))
    tasks = []
    for k, md in enumerate(modes):
        s, e = k * chunk, min(n, (k + 1) * chunk)
        if tasks and tasks[-1][2] == md:
            tasks[-1][1] = e
        else:
            tasks.append([s, e, md])
    A = torch.zeros(n, dtype=torch.int32)
    L = jp.Loop(0, 0, n, A, r=torch.zeros(n, dtype=torch.int32), w=torch.zeros(n, dtype=torch.int32))
    got = jp.jp_plan(L, profs, world, scheme=jp.JP_SCHED_STEALING, chunk_iters=chunk, tau_high=0.25)
    exp, _ = OS.stealing_plan([tuple(t) for t in tasks], world, chunk, None, 1.0)
    assert [tuple(int(x) for x in r) for r in got] == [tuple(int(x) for x in r) for r in exp]
    got = jp.jp_plan(L, profs, world, scheme=jp.JP_SCHED_SHARING, chunk_iters=chunk, tau_high=0.25)
    rg = OS.sharing_ranges(n, [1.0] * world)
    exp = [(max(s, b), min(e, ee), md, k) for k, (b, ee) in enumerate(rg) for s, e, md in tasks
           if max(s, b) < min(e, ee)]
    assert [tuple(int(x) for x in r) for r in got] == exp
