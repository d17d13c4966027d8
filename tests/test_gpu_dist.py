"""Multi-process partitioned runs with the REAL kernels: world_size 2 ranks share
cuda:0 over the gloo backend (the only GPU a test box has), each rank running
its task-sharing range through libjp.so and dist.py's collectives (C1, C3, C4,
TLS broadcast).  The NCCL/NVLink path uses the same code with backend "nccl"."""
import os
import socket
import sys

import pytest
import torch
import torch.distributed as dist
import torch.multiprocessing as mp

pytestmark = pytest.mark.gpu
ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def _port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def _worker(rank, world, port, case, q, exchange="dense"):
    sys.path[:0] = [ROOT, os.path.join(ROOT, "tests")]
    os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        import oracle as O
        import paper_conf_icpp_hanzlw13_b200 as jp
        from paper_conf_icpp_hanzlw13_b200 import dist as jd
        import synth
        from helpers import region_workload, to_oracle
        dev = torch.device("cuda:0")
        wl = {"c1_0": lambda: synth.config1(0.0), "c1_5": lambda: synth.config1(0.05),
              "c4": lambda: synth.config4(n=(1 << 18) + 5), "c3": lambda: synth.config3(0.01, n=1 << 16),
              "c5tail": lambda: synth.config5(n=1 << 14),
              "c5priv": lambda: region_workload(synth.config5(n=1 << 18), 3 << 16, 1 << 18),
              "c5head": lambda: region_workload(synth.config5(n=1 << 18), 0, 1 << 17)}[case]()
        ref = to_oracle(wl)
        _, A_exp, T_exp = O.run_seq(ref)
        g = wl.to(dev)
        full = jp.Loop.from_workload(g)
        b, e = jd.sharing_ranges(wl.n, world)[rank]
        loop = full.range(b, e)
        ws = jp.workspace(loop)
        jd.OWNER_MIN_LEN = 1 << 12
        res = jd.schedule_partitioned(loop, ws, full_loop=full, exchange=exchange)
        torch.cuda.synchronize()
        if wl.op == O.OP_PRIV_TMP:
            ok = g.A.cpu().numpy()[b:e].tobytes() == A_exp[b:e].tobytes() and \
                g.T.cpu().numpy().tobytes() == T_exp.tobytes()
        else:
            ok = g.A.cpu().numpy().tobytes() == A_exp.tobytes()
        p = O.profile(ref)
        ok &= (res["prof"]["raw_iters"], res["prof"]["war_iters"], res["prof"]["waw_iters"]) == \
            (p["raw_iters"], p["war_iters"], p["waw_iters"])
        q.put((rank, bool(ok), res["mode_name"]))
    except Exception as ex:  # pragma: no cover
        q.put((rank, False, repr(ex)))
    finally:
        dist.destroy_process_group()


@pytest.mark.parametrize("exchange", ["dense", "owner"])
@pytest.mark.parametrize("case,mode", [("c1_0", "DOALL"), ("c1_5", "TLS"), ("c4", "PRIVATIZED"), ("c3", "TLS"),
                                       ("c5tail", "TLS"), ("c5priv", "PRIVATIZED"), ("c5head", "DOALL")])
def test_two_ranks_one_gpu(case, mode, exchange):
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _port()
    ps = [ctx.Process(target=_worker, args=(r, 2, port, case, q, exchange)) for r in range(2)]
    for p in ps:
        p.start()
    out = sorted(q.get(timeout=600) for _ in range(2))
    for p in ps:
        p.join(timeout=120)
    assert [o[1] for o in out] == [True, True], out
    assert all(o[2] == mode for o in out), out


def _steal_worker(rank, world, port, case, exchange, q, dynamic=False):
    sys.path[:0] = [ROOT, os.path.join(ROOT, "tests")]
    os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        import oracle as O
        import paper_conf_icpp_hanzlw13_b200 as jp
        from paper_conf_icpp_hanzlw13_b200 import dist as jd
        import synth
        from helpers import to_oracle
        wl = {"c5": lambda: synth.config5(n=1 << 18), "c5big": lambda: synth.config5(n=1 << 20, density=0.01),
              "c4": lambda: synth.config4(n=(1 << 18) + 64, slots=1024)}[case]()
        ref = to_oracle(wl)
        _, A_exp, T_exp = O.run_seq(ref)
        g = wl.to("cuda:0")
        full = jp.Loop.from_workload(g)
        ws = jp.workspace(full)
        jd.OWNER_MIN_LEN = 1 << 12
        res = jd.schedule_stealing(full, ws, chunk_iters=1 << 14, exchange=exchange, dynamic=dynamic)
        torch.cuda.synchronize()
        if wl.op == O.OP_PRIV_TMP and dynamic:   # Y identity-written where the chunk was claimed
            ok = True
        elif wl.op == O.OP_PRIV_TMP:   # Y identity-written: each rank holds the chunks it ran
            A = g.A.cpu().numpy()
            ok = all(A[cs:ce].tobytes() == A_exp[cs:ce].tobytes() for cs, ce, _, ow in res["chunks"] if ow == rank)
        else:
            ok = g.A.cpu().numpy().tobytes() == A_exp.tobytes()
        if wl.T is not None:
            ok &= g.T.cpu().numpy().tobytes() == T_exp.tobytes()
        p = O.profile(ref)
        ok &= (res["prof"]["raw_iters"], res["prof"]["war_iters"], res["prof"]["waw_iters"]) == \
            (p["raw_iters"], p["war_iters"], p["waw_iters"])
        q.put((rank, bool(ok), res["n_tasks"], res["n_batches"], res["rank_work"]))
    except Exception as ex:  # pragma: no cover
        import traceback
        q.put((rank, False, traceback.format_exc(), 0, None))
    finally:
        dist.destroy_process_group()


@pytest.mark.parametrize("exchange,dynamic", [("dense", False), ("owner", False), ("dense", True), ("owner", True)])
@pytest.mark.parametrize("case", ["c5", "c5big", "c4"])
def test_stealing_two_ranks_one_gpu(case, exchange, dynamic):
    """Config 5 (DOALL head, TLS middle, privatized tail) under the multi-rank
    task-stealing scheme: every replica ends with the sequential result."""
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _port()
    ps = [ctx.Process(target=_steal_worker, args=(r, 2, port, case, exchange, q, dynamic)) for r in range(2)]
    for p in ps:
        p.start()
    out = sorted(q.get(timeout=600) for _ in range(2))
    for p in ps:
        p.join(timeout=120)
    assert [o[1] for o in out] == [True, True], out
    assert sum(o[4]["iters"] for o in out) == {"c5": 1 << 18, "c5big": 1 << 20, "c4": (1 << 18) + 64}[case]


def _p2p_worker(rank, world, port, q):
    sys.path[:0] = [ROOT, os.path.join(ROOT, "tests")]
    os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        import oracle as O
        import paper_conf_icpp_hanzlw13_b200 as jp
        from paper_conf_icpp_hanzlw13_b200 import dist as jd
        import synth
        from helpers import to_oracle
        wl = synth.config4(n=(1 << 18) + 64, slots=1024)
        _, A_exp, T_exp = O.run_seq(to_oracle(wl))
        g = wl.to("cuda:0")
        T0, A0 = g.T.clone(), g.A.clone()
        full = jp.Loop.from_workload(g)
        b, e = jd.sharing_ranges(wl.n, world)[rank]
        loop = full.range(b, e)
        ws = jp.workspace(loop)
        ok = True
        handles = jd.p2p_handles(loop, ws)   # collective: mapped once, reused by three epochs
        for ep in range(4):   # epochs 1..3 on the same counter and mappings, then one with handles of its own
            g.T.copy_(T0)
            g.A.copy_(A0)
            res = jd.schedule_partitioned(loop, ws, full_loop=full, exchange="p2p", p2p=handles if ep < 3 else None)
            torch.cuda.synchronize()
            ok &= g.T.cpu().numpy().tobytes() == T_exp.tobytes()
            ok &= g.A.cpu().numpy()[b:e].tobytes() == A_exp[b:e].tobytes()
            ok &= res["mode_name"] == "PRIVATIZED"
        m = handles["keys_T"]
        ok &= m.ok() and m.epoch == 3
        dist.barrier()
        for m in handles.values():
            m.close()
        q.put((rank, bool(ok)))
    except Exception:  # pragma: no cover
        import traceback
        q.put((rank, traceback.format_exc()))
    finally:
        dist.destroy_process_group()


def test_p2p_key_merge_two_ranks():
    """C4 over peer memory (jp_keys_merge_p2p through CUDA IPC, no NCCL): config 4's
    privatized slots merged and applied in one kernel per rank, three epochs."""
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _port()
    ps = [ctx.Process(target=_p2p_worker, args=(r, 2, port, q)) for r in range(2)]
    for p in ps:
        p.start()
    out = sorted(q.get(timeout=300) for _ in range(2))
    for p in ps:
        p.join(timeout=120)
    assert out == [(0, True), (1, True)], out
