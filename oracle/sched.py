"""TEST INFRASTRUCTURE ONLY -- plain-Python restatements of the scheduler
decisions of Japonica Sec. V, used to pin the host logic
of libjp.so (jp_select_mode, jp_plan_sharing, jp_plan_stealing).
"""
from __future__ import annotations

import math

DOALL, PRIVATIZED, TLS, SEQ_RECOMMENDED = 0, 1, 2, 3


def select_mode(all_null: bool, n: int, raw: int, war: int, waw: int, tau_high: float = 0.999) -> int:
    """Fig. 2(b) workflow, readings A4 and A5:
    determined DOALL? -> A;  TD density high -> C;  low -> B;  FD -> D;  else D'."""
    if all_null:
        return DOALL
    d_raw = raw / n if n else 0.0
    if d_raw > tau_high:
        return SEQ_RECOMMENDED
    if raw > 0:
        return TLS
    if war > 0 or waw > 0:
        return PRIVATIZED
    return DOALL


def boundary(cg: float, fg: float, cc: float, fc: float) -> float:
    """Task-sharing boundary Cg*Fg / (Cg*Fg + Cc*Fc) (reading A15)."""
    return cg * fg / (cg * fg + cc * fc)


def sharing_ranges(n: int, weights):
    """Rank k gets [floor(n*S_k), floor(n*S_{k+1})), S = prefix of normalised weights."""
    total = 0.0
    for w in weights:
        total += w
    out, pre = [], 0.0
    for k, w in enumerate(weights):
        b0 = math.floor(n * (pre / total))
        pre += w
        b1 = n if k == len(weights) - 1 else math.floor(n * (pre / total))
        out.append((b0, b1))
    return out


def stealing_plan(tasks, world, chunk, speed=None, speed_tls=1.0):
    """Alg. 1 with readings A16/A18 as a discrete-event plan:
      * TLS tasks stay whole and are pinned to rank 0 (their commit is ordered);
      * other tasks are cut into chunks and dealt to per-rank deques by task
        sharing with weights = speeds;
      * the rank with the smallest clock (ties: lowest rank) runs its pinned
        task, else the head of its own deque, else steals the TAIL chunk of the
        deque with the most remaining iterations (ties: lowest rank).
    Returns ([(start, end, mode, owner)], stolen)."""
    speed = speed or [1.0] * world
    chunks = []
    for (s, e, m) in tasks:
        if m in (TLS, SEQ_RECOMMENDED):
            chunks.append([s, e, m, 0, -1, True])
        else:
            c = s
            while c < e:
                chunks.append([c, min(e, c + chunk), m, -1, -1, False])
                c += chunk
    part = [i for i, c in enumerate(chunks) if not c[5]]
    deques = [[] for _ in range(world)]
    for k, (b0, b1) in enumerate(sharing_ranges(len(part), speed)):
        for q in range(b0, b1):
            chunks[part[q]][3] = k
            deques[k].append(part[q])
    pinned = [i for i, c in enumerate(chunks) if c[5]]
    clock = [0.0] * world
    done = [False] * world
    stolen = 0
    while True:
        live = [k for k in range(world) if not done[k]]
        if not live:
            break
        k = min(live, key=lambda q: (clock[q], q))
        rate = speed[k]
        if k == 0 and pinned:
            c = pinned.pop(0)
            rate = speed_tls
        elif deques[k]:
            c = deques[k].pop(0)
        else:
            best, v = 0, -1
            for q in range(world):
                if q == k:
                    continue
                rem = sum(chunks[x][1] - chunks[x][0] for x in deques[q])
                if rem > best:
                    best, v = rem, q
            if v < 0:
                done[k] = True
                continue
            c = deques[v].pop()
            stolen += 1
        chunks[c][4] = k
        clock[k] += (chunks[c][1] - chunks[c][0]) / rate
    return [(c[0], c[1], c[2], c[4]) for c in chunks], stolen


# ---------------------------------------------------------------------------
# workflows (P:L197-200 PDG, Alg. 1 over loops, P:L461-469 scheme
# selection; readings B9, B10)
# ---------------------------------------------------------------------------
SHARING, STEALING, AUTO = 0, 1, 2


def workflow_plan(footprints, iters, scheme=AUTO):
    """footprints[u]: list of (lo, hi, writes) byte ranges loop u touches; iters[u]
    its trip count.  Loop u depends on t < u iff a range of one that writes
    overlaps a range of the other; batch[u] = 1 + max batch of its dependencies.
    AUTO -> STEALING iff some batch holds >= 2 loops and no loop has more than
    half of all iterations, else SHARING."""
    n = len(footprints)
    batch = [0] * n
    deps = [0] * n
    for u in range(n):
        for t in range(u):
            hit = any((wa or wb) and la < hb and lb < ha
                      for (la, ha, wa) in footprints[t] for (lb, hb, wb) in footprints[u])
            if hit:
                deps[u] |= 1 << t
                batch[u] = max(batch[u], batch[t] + 1)
    n_batches = max(batch) + 1 if n else 0
    if scheme == AUTO:
        wide = any(batch.count(b) >= 2 for b in range(n_batches))
        scheme = STEALING if wide and 2 * max(iters, default=0) <= sum(iters) else SHARING
    return {"scheme": scheme, "n_batches": n_batches, "batch": batch, "deps": deps}
