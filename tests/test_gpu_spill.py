"""Task sharing with cross-boundary spill (
P:L350-353): jp_run_doall_spill against the oracle's sequential result.

Single process: the ranks' launches run concurrently on separate streams of
cuda:0 over shards in separate buffers, the slow "ranks" capped to one or two
CTAs so that the fast one drains their ranges from the tail.  Two processes:
dist.SpillGroup maps the peer shard and the counter table through CUDA IPC
(jp_ipc_export / jp_ipc_import) and runs the same kernel on each rank."""
import os
import socket
import sys

import numpy as np
import pytest
import torch
import torch.distributed as dist
import torch.multiprocessing as mp

import oracle as O
import paper_conf_icpp_hanzlw13_b200 as jp
import synth
from helpers import to_oracle

pytestmark = pytest.mark.gpu
ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def _whole(op, dt, n):
    """A whole affine loop of opcode op and its sequential result (oracle)."""
    g = np.random.default_rng(n + 31 * op + dt)
    el = np.int32 if dt == O.I32 else np.float32
    mk = lambda m: (g.integers(-1000, 1000, size=m).astype(el) if dt == O.I32  # noqa: E731
                    else g.standard_normal(m).astype(el))
    A, X = mk(n), mk(n)
    T = mk(n) if op == O.OP_PRIV_TMP else None
    c0 = 3 if dt == O.I32 else 1.25
    wl = synth.Workload("affine", op, dt, n, torch.from_numpy(A), X=torch.from_numpy(X),
                        T=None if T is None else torch.from_numpy(T), c0=c0, c1=c0)
    _, A_exp, T_exp = O.run_seq(to_oracle(wl))
    return wl, A_exp, T_exp


def _shards(wl, world):
    rg = jp.jp_plan_sharing(wl.n, world)
    out = []
    for b, e in rg:
        sl = lambda t: None if t is None else t[b:e].clone().cuda()  # noqa: E731
        out.append((b, e, jp.Loop(wl.op, wl.dtype, e - b, sl(wl.A), X=sl(wl.X), T=sl(wl.T), c0=wl.c0, c1=wl.c1,
                                  iter_base=b)))
    return out


@pytest.mark.parametrize("op,dt", [(O.OP_SAXPY, O.F32), (O.OP_ADD_C, O.I32), (O.OP_PRIV_TMP, O.F32),
                                   (O.OP_STENCIL2, O.F32)])
@pytest.mark.parametrize("world,n,chunk", [(2, 1 << 20, 1 << 14), (3, (1 << 20) + 7, 4099), (8, 300001, 1000),
                                           (2, 5, 2), (4, 1 << 22, 1 << 16)])
def test_spill_streams_match_oracle(op, dt, world, n, chunk):
    wl, A_exp, T_exp = _whole(op, dt, n)
    sh = _shards(wl, world)
    views = [s[2] for s in sh]
    ctr = torch.zeros(world, dtype=torch.int64, device="cuda")
    stats = [torch.zeros(3, dtype=torch.int64, device="cuda") for _ in range(world)]
    streams = [torch.cuda.Stream() for _ in range(world)]
    torch.cuda.synchronize()
    for k in range(world):
        jp.jp_run_doall_spill(views, k, chunk, ctr, stats[k], max_ctas=0 if k == 0 else 1 + (k % 2),
                              stream=streams[k])
    torch.cuda.synchronize()
    for (b, e, L) in sh:
        assert L.tensors["A"].cpu().numpy().tobytes() == A_exp[b:e].tobytes()
        if op == O.OP_PRIV_TMP:
            assert L.tensors["T"].cpu().numpy().tobytes() == T_exp[b:e].tobytes()
    st = torch.stack(stats).cpu().numpy()
    assert int(st[:, 0].sum() + st[:, 1].sum()) == n          # every iteration exactly once
    nch = [-(-(e - b) // chunk) for b, e, _ in sh]
    c = ctr.cpu().numpy().astype(np.uint64)
    claimed = [int(c[k] & 0xFFFFFFFF) + int(c[k] >> 32) for k in range(world)]
    assert all(claimed[k] >= nch[k] for k in range(world))


def test_spill_single_rank_is_plain_doall():
    wl, A_exp, _ = _whole(O.OP_SAXPY, O.F32, (1 << 18) + 3)
    (b, e, L), = _shards(wl, 1)
    ctr = torch.zeros(1, dtype=torch.int64, device="cuda")
    stats = torch.zeros(3, dtype=torch.int64, device="cuda")
    jp.jp_run_doall_spill([L], 0, 1 << 12, ctr, stats)
    torch.cuda.synchronize()
    assert L.tensors["A"].cpu().numpy().tobytes() == A_exp.tobytes()
    assert stats.tolist() == [wl.n, 0, 0]


def test_spill_rejects_indirect_and_mixed_views():
    wl = synth.config1(0.0, n=4096).to("cuda")
    L = jp.Loop.from_workload(wl)
    ctr = torch.zeros(1, dtype=torch.int64, device="cuda")
    with pytest.raises(jp.JPError) as e:
        jp.jp_run_doall_spill([L], 0, 1024, ctr)
    assert e.value.status == jp._abi.JP_ERR_UNSUPPORTED
    a, _, _ = _whole(O.OP_SAXPY, O.F32, 64)
    (_, _, L1), = _shards(a, 1)
    L2 = jp.Loop(O.OP_SAXPY, O.F32, 64, L1.tensors["A"], X=L1.tensors["X"], c0=2.0)
    ctr = torch.zeros(2, dtype=torch.int64, device="cuda")
    with pytest.raises(jp.JPError) as e:
        jp.jp_run_doall_spill([L1, L2], 0, 16, ctr)
    assert e.value.status == jp._abi.JP_ERR_ARG


def _port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def _worker(rank, world, port, q):
    sys.path[:0] = [ROOT, os.path.join(ROOT, "tests")]
    os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        import oracle as O2
        import paper_conf_icpp_hanzlw13_b200 as jp2
        from paper_conf_icpp_hanzlw13_b200 import dist as jd
        import synth as S
        from helpers import to_oracle as tor
        n = (1 << 22) + 12
        b, e = jd.sharing_ranges(n, world)[rank]
        wl = S.config2(n=n, start=b, count=e - b).to("cuda:0")
        shard = jp2.Loop.from_workload(wl, iter_base=b)
        sg = jd.SpillGroup(shard)
        res = None
        for _ in range(2):   # the group is reusable: counters re-zeroed per run
            wl2 = S.config2(n=n, start=b, count=e - b)
            shard.tensors["A"].copy_(wl2.A.cuda())
            res = sg.run(chunk=1 << 16, max_ctas=0 if rank == 0 else 1)
        exp = O2.run_seq(tor(S.config2(n=n, start=b, count=e - b)))[1]
        ok = shard.tensors["A"].cpu().numpy().tobytes() == exp.tobytes()
        tot = torch.tensor([res["own_iters"] + res["stolen_iters"]])
        dist.all_reduce(tot)
        ok &= int(tot.item()) == n
        sg.close()
        q.put((rank, bool(ok), res))
    except Exception as ex:  # pragma: no cover
        q.put((rank, False, repr(ex)))
    finally:
        dist.destroy_process_group()


def test_spill_two_processes_ipc():
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _port()
    ps = [ctx.Process(target=_worker, args=(r, 2, port, q)) for r in range(2)]
    for p in ps:
        p.start()
    out = sorted(q.get(timeout=600) for _ in range(2))
    for p in ps:
        p.join(timeout=120)
    assert [o[1] for o in out] == [True, True], out


@pytest.mark.parametrize("world,chunk", [(2, 1024), (3, 4096), (4, 1000)])
def test_priv_claim_streams_match_oracle(world, chunk):
    """Device-side stealing of privatized chunks (jp_run_priv_claim): `world`
    replicas on concurrent streams share one counter table; the slow ranks are
    capped to one CTA.  The max over the replicas' key tables, applied, gives
    the sequential result of config 5's privatized tail; every chunk ran once."""
    from helpers import region_workload
    base = synth.config5(n=1 << 16)
    wl = region_workload(base, 3 << 14, 1 << 16)
    _, A_exp, _ = O.run_seq(to_oracle(wl))
    reps = [wl.to("cuda") for _ in range(world)]
    Ls = [jp.Loop.from_workload(r) for r in reps]
    wss = [jp.workspace(L) for L in Ls]
    keys = []
    for L, ws in zip(Ls, wss):
        off, nb = jp.jp_ws_region(L, "keys_A")
        k = ws[off:off + nb].view(torch.int64)
        k.zero_()
        keys.append(k)
    n = wl.n
    ch = [(s, min(n, s + chunk)) for s in range(0, n, chunk)]
    first = [len(ch) * k // world for k in range(world + 1)]
    dch = torch.tensor(ch, dtype=torch.int64, device="cuda")
    ctr = torch.zeros(world, dtype=torch.int64, device="cuda")
    stats = [torch.zeros(3, dtype=torch.int64, device="cuda") for _ in range(world)]
    sts = [torch.cuda.Stream() for _ in range(world)]
    torch.cuda.synchronize()
    for k in range(world):
        jp.jp_run_priv_claim(Ls[k], dch, first, k, ctr, wss[k], stats[k], max_ctas=0 if k == 0 else 1,
                             stream=sts[k])
    torch.cuda.synchronize()
    merged = torch.stack(keys).amax(0)
    jp.jp_merge_apply(reps[0].A, merged)
    torch.cuda.synchronize()
    assert reps[0].A.cpu().numpy().tobytes() == A_exp.tobytes()
    st = torch.stack(stats).cpu().numpy()
    assert int(st[:, 0].sum() + st[:, 1].sum()) == n


def test_p2p_merge_times_out_instead_of_hanging():
    """jp_keys_merge_p2p with a peer that never arrives: the device-side barrier
    gives up after ~4 s and sets the error flag (no hang, no strike)."""
    import time
    keys = torch.zeros(1024, dtype=torch.int64, device="cuda")
    bar = torch.zeros(1, dtype=torch.int64, device="cuda")
    err = torch.zeros(1, dtype=torch.int32, device="cuda")
    t0 = time.perf_counter()
    jp.jp_keys_merge_p2p([keys.data_ptr(), keys.data_ptr()], keys, bar, 1, err)   # world 2, one caller
    torch.cuda.synchronize()
    dt = time.perf_counter() - t0
    assert int(err.item()) == 1 and 3.0 < dt < 30.0, (int(err.item()), dt)
    # a single-rank merge (world 1) passes both barriers and applies the keys
    keys[5] = (7 << 32) | 42
    arr = torch.zeros(1024, dtype=torch.int32, device="cuda")
    err.zero_()
    bar.zero_()
    jp.jp_keys_merge_p2p([keys.data_ptr()], keys, bar, 1, err, arr=arr)
    torch.cuda.synchronize()
    assert int(err.item()) == 0 and int(arr[5].item()) == 42 and int(arr.sum().item()) == 42
