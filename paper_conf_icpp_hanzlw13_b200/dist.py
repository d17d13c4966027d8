"""Multi-GPU driver: the paper's task-sharing and task-stealing schemes
(Sec. V) across the ranks of one node, one process per GPU.

The C library never calls NCCL (include/jp.h): this module issues the
collectives through ``torch.distributed`` between the split entry points of
libjp.so and lets the kernels consume the results.  Collectives used
(SURVEY.md Sec.2c):

  C1  all_reduce MAX int32  over the first-writer / first-reader tables of the
      partitioned profile (entries are INT32_MAX - gid, empty -1);
  C3  all_reduce SUM int64  over the per-rank raw/war/waw counts;
  C4  all_reduce MAX int64  over the packed last-writer keys (gid+1)<<32|bits
      of the privatized / partitioned writes;
  bcast                      of the in/out array after a TLS run (TLS windows
      stay ordered on one GPU: "replicas only", north_star).

``exchange="owner"`` replaces the dense C1 / C4
all_reduces of len-sized tables by an owner-partitioned sparse exchange
(jp_sparse_* in jp.h; owner(a) = a / ceil(len/world)):

  C1o  pack the touched (addr, minW, minR) rows by owner -> all_to_all -> the
       owner folds them (MAX) -> answers each row with the folded value ->
       all_to_all back -> scatter.  Every address a rank's classify looks up is
       one it touched, so it ends with exactly the dense all_reduce's values
       there;
  C4o  pack the nonzero (addr, key) rows by owner -> all_to_all -> the owner
       folds them -> all_gather of each owner's final nonzero rows (padded
       with address -1) -> scatter: every replica holds the merged keys.

The bytes moved scale with the addresses the loop touches, not with len.
Tables shorter than OWNER_MIN_LEN (e.g. the 1024-slot T of config 4) stay on
the dense all_reduce.

Iteration ranges come from ``jp_plan_sharing`` (boundary formula)
and ``jp_plan_stealing`` (Alg. 1).  Every compute step is a
libjp.so kernel; ``engine`` exists only so that the CPU tests can drive the
collective logic with gloo and a test double (there is no CPU path here).
"""
from __future__ import annotations

import torch
import torch.distributed as dist

from . import _abi


def _engine(engine):
    if engine is not None:
        return engine
    import paper_conf_icpp_hanzlw13_b200 as jp
    return jp


def world_rank(group=None) -> tuple[int, int]:
    if dist.is_available() and dist.is_initialized():
        return dist.get_world_size(group), dist.get_rank(group)
    return 1, 0


def sharing_ranges(n: int, world: int, weights=None, engine=None):
    """Task-sharing plan: rank k gets [floor(n*S_k), floor(n*S_{k+1}))."""
    return _engine(engine).jp_plan_sharing(n, world, weights)


def _region(ws: torch.Tensor, loop, name: str, dtype, engine=None):
    off, nb = _engine(engine).jp_ws_region(loop, name)
    if nb == 0:
        return None
    return ws[off:off + nb].view(dtype)


OWNER_MIN_LEN = 1 << 16
P2P_MAX_LEN = 16384


def _a2a_rows(rows, counts, group):
    """all_to_all of owner-bucketed rows; returns (received rows, received counts)."""
    sc = torch.tensor(counts, dtype=torch.int64, device=rows.device)
    rc = torch.empty_like(sc)
    dist.all_to_all_single(rc, sc, group=group)
    rcl = [int(x) for x in rc.tolist()]
    recv = rows.new_empty((sum(rcl), rows.shape[1]))
    dist.all_to_all_single(recv, rows.contiguous(), output_split_sizes=rcl, input_split_sizes=list(counts),
                           group=group)
    return recv, rcl


def owner_reduce_touched(t0, t1, empty, group=None, engine=None) -> dict:
    """C1o: every entry this rank touched (t0 or t1 != empty) ends holding the MAX
    over all ranks, as a dense all_reduce MAX would leave it there."""
    jp = _engine(engine)
    world, _ = world_rank(group)
    rows, counts = jp.jp_sparse_pack(t0, t1, empty, world)
    recv, rcl = _a2a_rows(rows, counts, group)
    jp.jp_sparse_reduce_max(t0, t1, recv)
    jp.jp_sparse_gather(t0, t1, recv)   # stream-ordered after every received row is folded
    back = torch.empty_like(rows)
    dist.all_to_all_single(back, recv, output_split_sizes=list(counts), input_split_sizes=rcl, group=group)
    jp.jp_sparse_scatter(t0, t1, back)
    return {"rows_sent": int(rows.shape[0]), "rows_recv": int(recv.shape[0]),
            "bytes_sent": 2 * rows.numel() * rows.element_size()}


def owner_reduce_replicate(t, empty, group=None, engine=None) -> dict:
    """C4o: t ends, on every rank, equal to the all_reduce MAX of t over the ranks
    at every address where some rank holds a non-empty entry."""
    jp = _engine(engine)
    world, rank = world_rank(group)
    rows, counts = jp.jp_sparse_pack(t, None, empty, world)
    recv, _ = _a2a_rows(rows, counts, group)
    jp.jp_sparse_reduce_max(t, None, recv)
    n = t.numel()
    sl = -(-n // world)
    fin, _ = jp.jp_sparse_pack(t, None, empty, 1, min(rank * sl, n), min((rank + 1) * sl, n))
    m = torch.tensor([fin.shape[0]], dtype=torch.int64, device=t.device)
    ms = [torch.empty_like(m) for _ in range(world)]
    dist.all_gather(ms, m, group=group)
    mx = max(int(x.item()) for x in ms)
    pad = torch.full((max(mx, 1), 2), -1, dtype=t.dtype, device=t.device)
    pad[:fin.shape[0]] = fin
    got = [torch.empty_like(pad) for _ in range(world)]
    dist.all_gather(got, pad, group=group)
    jp.jp_sparse_scatter(t, None, torch.cat(got))
    return {"rows_sent": int(rows.shape[0]) + world * pad.shape[0], "rows_recv": int(recv.shape[0]),
            "bytes_sent": (rows.numel() + world * pad.numel()) * t.element_size()}


class P2PMerge:
    """C4 for one small key table (<= 16384 slots) over NVLink peer memory
    (jp_keys_merge_p2p): every rank maps every rank's table and rank 0's
    barrier counter through CUDA IPC once; ``run`` merges (max per slot) and
    optionally applies the keys to ``arr`` inside one single-CTA kernel per rank
    -- no NCCL call, two device-side barriers."""

    def __init__(self, table, group=None):
        import paper_conf_icpp_hanzlw13_b200 as jp
        self.jp, self.group, self.table = jp, group, table
        self.world, self.rank = world_rank(group)
        dev = table.device
        self.bar = torch.zeros(1, dtype=torch.int64, device=dev)
        self.err = torch.zeros(1, dtype=torch.int32, device=dev)
        self.epoch = 0
        self._opened = []
        mine = (jp.jp_ipc_export(table), jp.jp_ipc_export(self.bar) if self.rank == 0 else None)
        allinfo = [None] * self.world
        dist.all_gather_object(allinfo, mine, group=group)
        self.ptrs = []
        for k, (h, _) in enumerate(allinfo):
            if k == self.rank:
                self.ptrs.append(table.data_ptr())
            else:
                p = jp.jp_ipc_import(*h)
                self._opened.append((p, h[1]))
                self.ptrs.append(p)
        self.bar_ref = self.bar
        if self.rank != 0:
            p = jp.jp_ipc_import(*allinfo[0][1])
            self._opened.append((p, allinfo[0][1][1]))
            self.bar_ref = _RawPtr(p)
        torch.cuda.synchronize()
        dist.barrier(group=group)

    def run(self, table=None, arr=None, stream=None):
        """Merge (and apply to ``arr``).  Raises if the device barrier timed out:
        the keys are then NOT merged and nothing was applied on this rank."""
        if table is not None and (table.data_ptr() != self.table.data_ptr() or table.numel() != self.table.numel()):
            raise ValueError("P2PMerge.run: this handle maps a different key table")
        self.epoch += 1
        self.jp.jp_keys_merge_p2p(self.ptrs, self.table, self.bar_ref, self.epoch, self.err, arr, stream)
        if not self.ok():
            raise RuntimeError(f"p2p key merge (epoch {self.epoch}): device barrier timed out on rank {self.rank}; "
                               "keys not merged")

    def ok(self) -> bool:
        return int(self.err.item()) == 0

    def close(self):
        for p, off in self._opened:
            self.jp.jp_ipc_close(p, off)
        self._opened = []


class PrivMerge:
    """Config 4 across the ranks in ONE kernel per rank and step
    (jp_priv_stream_merge): privatized stream of this rank's range, C4 by peer
    stores into every rank's inbox (CUDA IPC / NVLink), R2 -- no NCCL call, no
    second launch.  Collective to build (every rank maps every rank's inbox
    once); ``step()`` launches, ``check()`` synchronizes and raises if a merge
    timed out; ``graph()`` captures one step in a CUDA graph (same arguments
    every step: the epoch lives in the inbox) and returns a replay callable."""

    def __init__(self, loop, ws, group=None, engine=None):
        jp = _engine(engine)
        self.jp, self.loop, self.ws, self.group = jp, loop, ws, group
        self.world, self.rank = world_rank(group)
        nb = jp.jp_priv_inbox_bytes(loop, self.world)
        if nb == 0:
            raise ValueError("the fused merge needs the config-4 shape (PRIV_TMP, identity X/Y, indirect s, "
                             "len_T <= 4096)")
        dev = ws.device
        self.inbox = torch.zeros(nb // 8, dtype=torch.int64, device=dev)
        self.err = torch.zeros(1, dtype=torch.int32, device=dev)
        self._opened = []
        torch.cuda.synchronize()
        if self.world == 1:
            self.ptrs = [self.inbox.data_ptr()]
        else:
            allinfo = [None] * self.world
            dist.all_gather_object(allinfo, jp.jp_ipc_export(self.inbox), group=group)
            self.ptrs = []
            for k, h in enumerate(allinfo):
                if k == self.rank:
                    self.ptrs.append(self.inbox.data_ptr())
                else:
                    p = jp.jp_ipc_import(*h)
                    self._opened.append((p, h[1]))
                    self.ptrs.append(p)
            dist.barrier(group=group)

    def step(self, stream=None):
        self.jp.jp_priv_stream_merge(self.loop, self.ws, self.ptrs, self.rank, self.err, stream=stream)

    def check(self):
        torch.cuda.synchronize()
        if int(self.err.item()) != 0:
            raise RuntimeError(f"fused privatized merge: a peer's flag never arrived on rank {self.rank}")

    def graph(self):
        """One step captured in a CUDA graph (replayed with g.replay()); None if
        the driver refuses to capture the cooperative launch."""
        try:
            s = torch.cuda.Stream()
            g = torch.cuda.CUDAGraph()
            with torch.cuda.graph(g, stream=s):
                self.step()
            return g
        except Exception:   # pragma: no cover - capture support is driver-dependent
            return None

    def close(self):
        for p, off in self._opened:
            self.jp.jp_ipc_close(p, off)
        self._opened = []


def p2p_handles(loop, ws, group=None, engine=None) -> dict:
    """Collective: one P2PMerge per small key table of ``loop`` in ``ws`` (every
    rank must call it with its own replica).  The handles keep the tables (and
    so the workspaces) alive on every rank for as long as they live, so the
    peers' mapped pointers stay valid; pass them to ``privatized_partitioned``
    to reuse the mappings across calls, ``close()`` them when done."""
    jp = _engine(engine)
    out = {}
    for name in ("keys_A", "keys_T"):
        t = _region(ws, loop, name, torch.int64, jp)
        if t is not None and t.numel() <= P2P_MAX_LEN:
            out[name] = P2PMerge(t, group)
    return out


def _reduce_tables(tabs, empty, group, exchange, jp):
    """MAX of each table across the ranks: dense all_reduce, or the owner form."""
    tabs = [t for t in tabs if t is not None]
    if exchange == "owner" and tabs and tabs[0].numel() >= OWNER_MIN_LEN:
        return tabs
    for t in tabs:
        dist.all_reduce(t, op=dist.ReduceOp.MAX, group=group)
    return []


def profile_partitioned(loop, ws, group=None, engine=None, exchange: str = "dense", chunk_iters: int = 0,
                        chunk_counts=None) -> dict:
    """Profile of the whole loop from rank-local ranges (iter_base = global id of
    the rank's first iteration): stamp locally, C1 (dense or owner form),
    classify locally, C3.  The result equals the single-GPU profile exactly
    (tested)."""
    jp = _engine(engine)
    world, _ = world_rank(group)
    jp.jp_profile_stamp(loop, ws)
    if world > 1:
        left = _reduce_tables([_region(ws, loop, n, torch.int32, jp) for n in ("minW_A", "minR_A")], -1, group,
                              exchange, jp)
        if left:
            owner_reduce_touched(left[0], left[1] if len(left) > 1 else None, -1, group, jp)
        _reduce_tables([_region(ws, loop, n, torch.int32, jp) for n in ("minW_T", "minR_T")], -1, group, "dense", jp)
    if chunk_counts is None:
        p = jp.jp_profile_classify(loop, ws)
    else:
        p = jp.jp_profile_classify(loop, ws, chunk_iters=chunk_iters, chunk_counts=chunk_counts)
    if world > 1:
        dev = ws.device
        c = torch.tensor([p["n"], p["raw_iters"], p["war_iters"], p["waw_iters"]], dtype=torch.int64, device=dev)
        dist.all_reduce(c, group=group)
        f = torch.tensor([p["first_raw_iter"] if p["first_raw_iter"] >= 0 else (1 << 62)], dtype=torch.int64,
                         device=dev)
        dist.all_reduce(f, op=dist.ReduceOp.MIN, group=group)
        n, raw, war, waw = (int(x) for x in c.tolist())
        fr = int(f.item())
        p = {"n": n, "raw_iters": raw, "war_iters": war, "waw_iters": waw,
             "first_raw_iter": -1 if fr >= (1 << 62) else fr,
             "d_raw": raw / n if n else 0.0, "d_war": war / n if n else 0.0, "d_waw": waw / n if n else 0.0}
    return p


def privatized_partitioned(loop, ws, prof, group=None, engine=None, exchange: str = "dense", p2p=None):
    """PE(V) over rank-local ranges: keys locally, C4 (MAX over packed keys), then
    every rank applies the merged keys -- each rank ends with the sequential
    result in its replica of the keyed arrays; identity-indexed outputs stay
    sharded (each rank holds its own range).  ``exchange="p2p"``: small key
    tables merge over peer memory, through ``p2p`` (from ``p2p_handles``) or
    through handles built (collectively) and closed inside this call."""
    jp = _engine(engine)
    world, _ = world_rank(group)
    jp.jp_priv_stream(loop, prof, ws, clear_keys=True)
    applied = 0
    tabs = [(name, _region(ws, loop, name, torch.int64, jp)) for name in ("keys_A", "keys_T")]
    tabs = [(n_, t) for n_, t in tabs if t is not None]
    if world > 1:
        own = None
        if exchange == "p2p" and p2p is None and any(t.numel() <= P2P_MAX_LEN for _, t in tabs):
            p2p = own = p2p_handles(loop, ws, group, jp)
        try:
            for name, t in tabs:
                if exchange == "p2p" and t.numel() <= P2P_MAX_LEN:
                    arr = loop.tensors["A" if name == "keys_A" else "T"]
                    p2p[name].run(t, arr=arr.view(torch.int32) if arr is not None else None)
                    applied += 1
                    continue
                for t2 in _reduce_tables([t], 0, group, "owner" if exchange == "owner" else "dense", jp):
                    owner_reduce_replicate(t2, 0, group, jp)
        finally:
            if own is not None:
                torch.cuda.synchronize()
                dist.barrier(group=group)   # no peer still reads a table before it is unmapped
                for h in own.values():
                    h.close()
    if applied < len(tabs) or not tabs:
        jp.jp_priv_finalize(loop, ws)


def schedule_partitioned(loop, ws, group=None, tau_high: float = _abi.TAU_HIGH, tls_window: int = 0, tls_w_max: int = 2048,
                         full_loop=None, engine=None, exchange: str = "dense", p2p=None) -> dict:
    """Task sharing of one loop across the ranks (P:L342-358 generalised to k
    devices).  ``loop`` is this rank's range (iter_base = its first global id,
    index arrays offset, element arrays shared-address replicas).

      * all index arrays NULL: determined DOALL, each rank runs its shard, no
        collective (outputs stay sharded);
      * else partitioned profile (C1+C3), Fig. 2(b) mode, then
        DOALL / PRIVATIZED: privatized kernels + C4 merge (a DOALL loop is the
        dependence-free special case of PE(V));
        TLS / SEQ_RECOMMENDED: rank 0 runs the windows over ``full_loop`` and
        broadcasts the in/out arrays (replicas only).
    ``exchange``: "dense" (all_reduce of the tables), "owner" (NEXT-2) or "p2p"
    (small key tables over peer memory; ``p2p`` = handles from ``p2p_handles``).
    """
    jp = _engine(engine)
    world, rank = world_rank(group)
    if loop.tensors["r"] is None and loop.tensors["w"] is None and loop.tensors["r2"] is None \
            and loop.tensors["s"] is None:
        res = jp.jp_schedule(loop, ws)
        res["scheme"] = "sharing"
        return res
    if exchange not in ("dense", "owner", "p2p"):
        raise ValueError(f"exchange must be 'dense', 'owner' or 'p2p', not {exchange!r}")
    prof = profile_partitioned(loop, ws, group, jp, "owner" if exchange == "owner" else "dense")
    mode = jp.jp_select_mode(loop, prof, tau_high)
    res = {"mode": mode, "mode_name": _abi.MODE_NAMES[mode], "profiled": 1, "prof": prof, "scheme": "sharing"}
    if mode in (_abi.JP_MODE_DOALL, _abi.JP_MODE_PRIVATIZED):
        privatized_partitioned(loop, ws, prof, group, jp, exchange, p2p)
    else:
        if full_loop is None:
            raise ValueError("TLS needs the whole loop on rank 0 (full_loop)")
        if rank == 0:
            res["tls"] = jp.jp_run_tls(full_loop, window=tls_window, w_max=tls_w_max, prof=prof, ws=ws)
        if world > 1:
            for name in ("A", "T"):
                t = full_loop.tensors[name]
                if t is not None:
                    dist.broadcast(t, src=0, group=group)
    return res


def _levels(conf, nt):
    """Topological batch of every task: 1 + the highest batch it depends on."""
    lv = [0] * nt
    for u in range(nt):
        for t in range(u):
            if (conf[u] >> t) & 1:
                lv[u] = max(lv[u], lv[t] + 1)
    return lv


def schedule_stealing(full, ws, group=None, chunk_iters: int = 65536, tau_high: float = _abi.TAU_HIGH, speed=None,
                      speed_tls: float = 1.0, exchange: str = "dense", engine=None, timings: bool = False,
                      dynamic: bool = False, force_ranks: bool = False, profile: str = "replicated") -> dict:
    """Task stealing of one loop across the ranks (Alg. 1; SURVEY
    Sec.8(e) "Mixed").  Every rank holds full replicas (``full``, workspace
    ``ws`` of the whole loop):

      1. profile with per-chunk counts.  ``profile="replicated"`` (default):
         every rank profiles its full replica itself (jp_profile_plan_tasks:
         the address-bucket profile when the loop allows it, which also records
         per-chunk address ranges for the PDG) -- no exchange, and cheaper than
         exchanging len(A)-sized stamp tables once A is large; ``"partitioned"``:
         rank k stamps its chunk-aligned range, C1, classifies its chunks, then
         C3 (SUM) of the whole chunk-count array and of the totals;
      2. the plan on every rank (identical): tasks = maximal same-mode chunk
         runs, PDG from the per-address task masks (reading B2), batches;
      3. jp_plan_stealing: chunk owners by Alg. 1 (TLS tasks pinned to rank 0,
         tails stolen by idle ranks, reading A18);
      4. batch by batch: each rank runs its chunks -- DOALL / PRIVATIZED chunks
         through the privatized stream (packed last-writer keys; their exposed
         reads see the replica, which holds every earlier batch), rank 0 the
         batch's TLS tasks in place (then jp_export_keys) -- then C4 over the
         keys (dense or owner form) and every rank applies them: every replica
         holds the sequential result after the last batch.  ``dynamic``:
         the batch's DOALL / privatized chunks are claimed on the device
         (jp_run_priv_claim over a counter table shared through CUDA IPC):
         every rank starts on the chunks the plan gave it and, once idle --
         rank 0 after the pinned TLS task -- steals the tail of the most
         loaded rank's block, so the plan's balance is corrected at run time
         (Alg. 1's "steal when empty" on the device).  Outputs written
         through identity indices (no key table, e.g. config 4's Y) stay with
         the rank that executed the chunk, as under task sharing (``chunks``
         of the result gives the owners).

    A one-rank group has nothing to exchange: it runs the single-GPU
    scheduler, jp_schedule(STEALING) -- the same Alg. 1 plan without the
    partitioned profile, the key exchange and the privatized replicas
    (``force_ranks=True`` keeps the multi-rank path, e.g. to measure it).
    """
    jp = _engine(engine)
    world, rank = world_rank(group)
    n = full.n
    if world == 1 and not dynamic and not force_ranks and hasattr(jp, "jp_schedule"):
        ev = [torch.cuda.Event(enable_timing=True) for _ in range(2)] if timings else None
        if ev:
            ev[0].record()
        res = jp.jp_schedule(full, ws, scheme=_abi.JP_SCHED_STEALING, chunk_iters=chunk_iters, tau_high=tau_high)
        phases = None
        if ev:
            ev[1].record()
            torch.cuda.synchronize()
            phases = {"profile_ms": 0.0, "plan_ms": 0.0, "busy_ms": ev[0].elapsed_time(ev[1]), "merge_ms": 0.0,
                      "what": "one rank: jp_schedule(STEALING), phases not separated"}
        return {"scheme": "stealing", "phases": phases, "prof": res["prof"], "n_tasks": res["n_tasks"],
                "n_batches": res["n_batches"], "tasks": None, "chunks": [(0, n, res["mode"], 0)], "stolen": 0,
                "tls": res["tls"], "rank_work": {"chunks": -(-n // chunk_iters), "iters": n},
                "delegated": "jp_schedule(STEALING)"}
    nck = -(-n // chunk_iters)
    marks = []   # (phase, event) on the current stream when timings=True

    def mark(name):
        if timings:
            ev = torch.cuda.Event(enable_timing=True)
            ev.record()
            marks.append((name, ev))
    mark("start")
    if profile == "replicated" and hasattr(jp, "jp_profile_plan_tasks"):
        # every rank profiles its full replica itself (the address-bucket profile
        # with per-chunk counts and address ranges): no C1 / C3 exchange, the same
        # counts, tasks and PDG on every rank
        prof, ccl, tasks, conf = jp.jp_profile_plan_tasks(full, chunk_iters, ws, tau_high)
        mark("profile")
    else:
        c0, c1 = rank * nck // world, (rank + 1) * nck // world
        b, e = min(c0 * chunk_iters, n), min(c1 * chunk_iters, n)
        loop = full.range(b, e)
        dev = ws.device
        cc_loc = torch.zeros(max(3 * (c1 - c0), 3), dtype=torch.int64, device=dev)
        prof = profile_partitioned(loop, ws, group, jp, exchange, chunk_iters, cc_loc)
        cc = torch.zeros(3 * nck, dtype=torch.int64, device=dev)
        cc[3 * c0:3 * c1] = cc_loc[:3 * (c1 - c0)]
        if world > 1:
            dist.all_reduce(cc, group=group)
        mark("profile")
        tasks, conf = jp.jp_plan_tasks(full, cc.cpu(), chunk_iters, ws, tau_high)
        ccl = cc.cpu().tolist()
    lv = _levels(conf, len(tasks))
    chunks, stolen = jp.jp_plan_stealing(tasks, world, chunk_iters, speed, speed_tls)
    task_of = {}
    for t, (s, e2, _) in enumerate(tasks):
        task_of[(s, e2)] = t
    tls_stats = {"committed": 0, "executed": 0, "windows": 0, "violations": 0}
    mine = {"chunks": 0, "iters": 0}
    mark("plan")
    busy = merge = 0.0
    claim = ClaimCounters(ws.device, group) if dynamic else None
    claimed = [0, 0, 0]
    for level in range(max(lv) + 1 if lv else 0):
        mark("level")
        for name in ("keys_A", "keys_T"):
            t = _region(ws, full, name, torch.int64, jp)
            if t is not None:
                t.zero_()
        for t, (s, e2, mode) in enumerate(tasks):
            if lv[t] != level:
                continue
            if mode in (_abi.JP_MODE_TLS, _abi.JP_MODE_SEQ_RECOMMENDED):
                if rank == 0:   # pinned (Alg. 1: TLS tasks are never stolen)
                    sub = full.range(s, e2)
                    k0, k1 = s // chunk_iters, -(-e2 // chunk_iters)
                    raw = sum(ccl[3 * k] for k in range(k0, k1))
                    waw = sum(ccl[3 * k + 2] for k in range(k0, k1))
                    tp = {"n": e2 - s, "raw_iters": raw, "war_iters": 0, "waw_iters": waw, "first_raw_iter": -1,
                          "d_raw": raw / max(e2 - s, 1), "d_war": 0.0, "d_waw": waw / max(e2 - s, 1)}
                    if mode == _abi.JP_MODE_SEQ_RECOMMENDED:   # mode C: one warp, program order
                        st = jp.jp_run_tls(sub, prof=tp, ws=ws, path=7)
                    else:
                        st = jp.jp_run_tls(sub, prof=tp, ws=ws, recovery=int(waw == 0))
                    for k in tls_stats:
                        tls_stats[k] += st[k]
                    jp.jp_export_keys(sub, ws)
                    mine["chunks"] += k1 - k0
                    mine["iters"] += e2 - s
                continue
            if dynamic:
                continue
            # this rank's chunks of the task, adjacent ones run as one range (one launch)
            runs = []
            for (cs, ce, cm, owner) in sorted(c for c in chunks if c[3] == rank and s <= c[0] and c[1] <= e2):
                if runs and runs[-1][1] == cs:
                    runs[-1][1] = ce
                else:
                    runs.append([cs, ce])
                mine["chunks"] += 1
                mine["iters"] += ce - cs
            for cs, ce in runs:
                jp.jp_priv_stream(full.range(cs, ce), _NO_RAW, ws, clear_keys=False)
        if dynamic:   # the batch's partitioned chunks, dealt by the plan, claimed on the device
            part = [t for t, (_, _, m) in enumerate(tasks) if lv[t] == level and
                    m not in (_abi.JP_MODE_TLS, _abi.JP_MODE_SEQ_RECOMMENDED)]
            blocks = [[] for _ in range(world)]
            for (cs, ce, cm, owner) in sorted(chunks):
                if any(tasks[t][0] <= cs and ce <= tasks[t][1] for t in part):
                    blocks[owner].append((cs, ce))
            first = [0]
            for b_ in blocks:
                first.append(first[-1] + len(b_))
            flat = [x for b_ in blocks for c_ in b_ for x in c_]
            dch = torch.tensor(flat if flat else [0, 0], dtype=torch.int64, device=ws.device).view(-1, 2)
            st_ = claim.run(jp, full, dch, first, ws)
            claimed = [a + b for a, b in zip(claimed, st_)]
        mark("exec")
        if world > 1:
            for name in ("keys_A", "keys_T"):
                for t in _reduce_tables([_region(ws, full, name, torch.int64, jp)], 0, group, exchange, jp):
                    owner_reduce_replicate(t, 0, group, jp)
        jp.jp_priv_finalize(full, ws)
        mark("merge")
    phases = None
    if timings:
        torch.cuda.synchronize()
        phases = {"profile_ms": marks[0][1].elapsed_time(marks[1][1]), "plan_ms": marks[1][1].elapsed_time(marks[2][1])}
        for k in range(3, len(marks), 3):   # (level, exec, merge) per batch
            busy += marks[k][1].elapsed_time(marks[k + 1][1])
            merge += marks[k + 1][1].elapsed_time(marks[k + 2][1])
        phases.update(busy_ms=busy, merge_ms=merge)
    if claim is not None:
        mine = {"chunks": mine["chunks"], "iters": mine["iters"] + claimed[0] + claimed[1],
                "own_iters": claimed[0], "stolen_iters": claimed[1], "stolen_chunks": claimed[2]}
        claim.close()
    return {"scheme": "stealing", "phases": phases, "prof": prof, "n_tasks": len(tasks), "n_batches": max(lv) + 1 if lv else 0,
            "tasks": tasks, "chunks": chunks, "stolen": stolen, "tls": tls_stats, "rank_work": mine}


_NO_RAW = {"n": 0, "raw_iters": 0, "war_iters": 0, "waw_iters": 0, "first_raw_iter": -1, "d_raw": 0.0, "d_war": 0.0,
           "d_waw": 0.0}


class ClaimCounters:
    """The per-rank chunk counters of device-side stealing (jp_run_priv_claim),
    in rank 0's memory and mapped by every rank through CUDA IPC."""

    def __init__(self, dev, group=None):
        import paper_conf_icpp_hanzlw13_b200 as jp
        self.jp, self.group = jp, group
        self.world, self.rank = world_rank(group)
        self.ctr = torch.zeros(self.world, dtype=torch.int64, device=dev)
        self.stats = torch.zeros(3, dtype=torch.int64, device=dev)
        self.ref, self._opened = self.ctr, None
        if self.world > 1:
            info = [None] * self.world
            dist.all_gather_object(info, jp.jp_ipc_export(self.ctr) if self.rank == 0 else None, group=group)
            if self.rank != 0:
                p = jp.jp_ipc_import(*info[0])
                self._opened = (p, info[0][1])
                self.ref = _RawPtr(p)

    def run(self, jp, loop, chunks, first, ws):
        """One batch: zero the counters (rank 0), barrier, claim kernel, barrier."""
        if self.rank == 0:
            self.ctr.zero_()
        self.stats.zero_()
        if self.world > 1:
            torch.cuda.synchronize()
            dist.barrier(group=self.group)
        jp.jp_run_priv_claim(loop, chunks if first[-1] else chunks[:0], first, self.rank, self.ref, ws, self.stats)
        if self.world > 1:
            torch.cuda.synchronize()
            dist.barrier(group=self.group)
        return [int(x) for x in self.stats.tolist()]

    def close(self):
        if self._opened:
            self.jp.jp_ipc_close(*self._opened)
            self._opened = None


class SpillGroup:
    """Task sharing with cross-boundary spill across the ranks (M1, P:L350-353;
    C8): every rank maps every other rank's affine shard and rank 0's chunk
    counter table through CUDA IPC once; ``run`` then executes the whole loop
    with jp_run_doall_spill on every rank -- each rank consumes its own chunks
    ascending and, when done, takes the most-loaded rank's chunks descending,
    reading and writing them in the peer's memory over NVLink.  No collective
    moves data; two barriers bracket the run (counters zero before any rank
    starts; every chunk written before any rank reads its shard)."""

    def __init__(self, shard, group=None):
        import paper_conf_icpp_hanzlw13_b200 as jp
        self.jp, self.group = jp, group
        self.world, self.rank = world_rank(group)
        if self.world > 8:
            raise ValueError("spill supports up to 8 ranks (one node)")
        self.shard = shard
        dev = shard.tensors["A"].device
        self.ctr = torch.zeros(self.world, dtype=torch.int64, device=dev)
        self.stats = torch.zeros(3, dtype=torch.int64, device=dev)
        self._opened = []
        views = [shard.c]
        if self.world > 1:
            mine = {k: (None if shard.tensors[k] is None else jp.jp_ipc_export(shard.tensors[k])) for k in "AXT"}
            mine["ctr"] = jp.jp_ipc_export(self.ctr) if self.rank == 0 else None
            allinfo = [None] * self.world
            dist.all_gather_object(allinfo, mine, group=group)
            views = []
            for k, info in enumerate(allinfo):
                if k == self.rank:
                    views.append(shard.c)
                    continue
                v = _abi.jp_loop.from_buffer_copy(shard.c)
                for name in "AXT":
                    if info[name] is not None:
                        ptr = jp.jp_ipc_import(*info[name])
                        self._opened.append((ptr, info[name][1]))
                        setattr(v, name, ptr)
                views.append(v)
            if self.rank != 0:
                ptr = jp.jp_ipc_import(*allinfo[0]["ctr"])
                self._opened.append((ptr, allinfo[0]["ctr"][1]))
                self._ctr_ptr = ptr
            # every rank's shard has the same length semantics; n per rank from the peers
            ns = [None] * self.world
            dist.all_gather_object(ns, (shard.n, shard.c.len_A, shard.c.len_X, shard.c.len_T), group=group)
            for k, v in enumerate(views):
                v.n, v.len_A, v.len_X, v.len_T = ns[k]
        self.views = views

    def _ctr(self):
        if self.rank == 0 or self.world == 1:
            return self.ctr
        return _RawPtr(self._ctr_ptr)

    def run(self, chunk: int = 1 << 16, max_ctas: int = 0, stream=None) -> dict:
        if self.rank == 0:
            self.ctr.zero_()
        self.stats.zero_()
        if self.world > 1:
            torch.cuda.synchronize()
            dist.barrier(group=self.group)
        self.jp.jp_run_doall_spill(self.views, self.rank, chunk, self._ctr(), self.stats, max_ctas, stream)
        if self.world > 1:
            torch.cuda.synchronize()
            dist.barrier(group=self.group)
        own, stolen, nst = (int(x) for x in self.stats.tolist())
        return {"own_iters": own, "stolen_iters": stolen, "stolen_chunks": nst}

    def close(self):
        for ptr, off in self._opened:
            self.jp.jp_ipc_close(ptr, off)
        self._opened = []


class _RawPtr:
    """A device pointer posing as a tensor for the binding (data_ptr only)."""

    def __init__(self, ptr):
        self.ptr = ptr

    def data_ptr(self):
        return self.ptr


def stealing_plan(tasks, world: int, chunk_iters: int, speed=None, speed_tls: float = 0.05, engine=None):
    """Alg. 1 as a deterministic plan: [(start, end, mode, owner)] and #stolen."""
    return _engine(engine).jp_plan_stealing(tasks, world, chunk_iters, speed, speed_tls)
