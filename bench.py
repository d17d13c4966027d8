#!/usr/bin/env python
"""bench.py -- the Japonica loop-mode hot path on B200 (driver contract).

Headline workload (BASELINE.json configs[1], the configuration the metric is
quoted on): DOALL streaming SAXPY fp32, N = 2^28, task sharing across
--gpus ranks (strong scaling: the 2^28 iterations are split by
jp_plan_sharing, each rank's shard resident in its HBM before timing).  One
step = one jp_schedule() call on the rank's shard = the whole hot path for
that loop (static DOALL decision -> doall kernel).  The JSON line adds the
roofline of the dominant kernel, the CPU oracle baseline, and (N=1 only) a
"modes" object: TLS committed iter/s over the config-3 density sweep,
privatized config 4, tiny config 1 and the mixed config 5.

  python bench.py [--gpus N] [--steps K] [--warmup W] [--impl jp|reference]
"""
from __future__ import annotations

import argparse
import json
import os
import statistics
import subprocess
import sys
import threading
import time

ROOT = os.path.dirname(os.path.abspath(__file__))
sys.path.insert(0, ROOT)

import torch  # noqa: E402

METRIC = json.load(open(os.path.join(ROOT, "BASELINE.json")))["metric"]
N2 = 1 << 28
BYTES_PER_ITER_SAXPY = 12        # X 4 + Y 4 read, Y 4 written
BYTES_PER_ITER_PRIV = 12         # X 4 + s 4 read, Y 4 written


def peaks():
    p = os.path.join(ROOT, "MEASURED_PEAKS.json")
    if os.path.exists(p):
        d = json.load(open(p))
        return float(d["hbm_gbs"]), "measured (MEASURED_PEAKS.json hbm_gbs)"
    return 6650.0, "fallback (B200_PROFILING.md 6.65 TB/s)"


class Clocks:
    """nvidia-smi sampling around the timed region (B200_PROFILING.md clocks line).
    The sampler is started and primed before the timed region; samples taken
    between the last one before the region and the first one after it count."""
    Q = ("clocks.sm,clocks.max.sm,clocks_event_reasons.active,clocks_event_reasons.hw_slowdown,"
         "clocks_event_reasons.hw_thermal_slowdown,clocks_event_reasons.sw_thermal_slowdown,"
         "clocks_event_reasons.sw_power_cap")

    def __init__(self, index: int):
        self.index, self.rows, self.proc = index, [], None
        self.t0 = self.t1 = None

    def start(self):
        try:
            self.proc = subprocess.Popen(["nvidia-smi", "-i", str(self.index), f"--query-gpu={self.Q}",
                                          "--format=csv,noheader,nounits", "-lms", "50"],
                                         stdout=subprocess.PIPE, stderr=subprocess.DEVNULL, text=True)
            self.t = threading.Thread(target=self._read, daemon=True)
            self.t.start()
            deadline = time.time() + 5.0
            while not self.rows and time.time() < deadline:
                time.sleep(0.01)
        except OSError:
            self.proc = None
        return self

    def _read(self):
        for line in self.proc.stdout:
            self.rows.append((time.time(), [x.strip() for x in line.split(",")]))

    def mark_start(self):
        self.t0 = time.time()

    def mark_end(self):
        self.t1 = time.time()
        deadline = self.t1 + 1.0     # wait for the first sample after the region
        while time.time() < deadline and not any(t > self.t1 for t, _ in self.rows):
            time.sleep(0.01)

    def stop(self):
        if self.proc:
            self.proc.terminate()
            try:
                self.proc.wait(timeout=5)
            except subprocess.TimeoutExpired:
                self.proc.kill()

    def summary(self):
        rows = [(t, r) for t, r in self.rows if len(r) >= 7 and r[0].isdigit()]
        if self.t0 is not None and rows:
            before = [t for t, _ in rows if t <= self.t0]
            after = [t for t, _ in rows if t >= self.t1]
            lo = before[-1] if before else self.t0
            hi = after[0] if after else self.t1
            rows = [(t, r) for t, r in rows if lo <= t <= hi]
        if not rows:
            return {"sm_mhz": None, "sm_max_mhz": None, "reasons": ["unsampled"], "samples": 0}
        names = ["hw_slowdown", "hw_thermal_slowdown", "sw_thermal_slowdown", "sw_power_cap"]
        reasons = sorted({names[k] for _, r in rows for k in range(4) if r[3 + k].lower() == "active"})
        return {"sm_mhz": statistics.median(int(r[0]) for _, r in rows), "sm_max_mhz": int(rows[0][1][1]),
                "reasons": reasons, "samples": len(rows)}


def dist_env():
    world = int(os.environ.get("WORLD_SIZE", "1"))
    rank = int(os.environ.get("RANK", "0"))
    local = int(os.environ.get("LOCAL_RANK", "0"))
    return world, rank, local


def barrier(world):
    if world > 1:
        torch.distributed.barrier()
    torch.cuda.synchronize()


def _coll_dev(dev):
    # NCCL reduces device tensors; the gloo test mode (JP_DIST_BACKEND=gloo) host ones
    return dev if torch.distributed.get_backend() == "nccl" else "cpu"


def max_over_ranks(x: float, world: int, dev) -> float:
    if world == 1:
        return x
    t = torch.tensor([x], dtype=torch.float64, device=_coll_dev(dev))
    torch.distributed.all_reduce(t, op=torch.distributed.ReduceOp.MAX)
    return float(t.item())


def sum_over_ranks(x: float, world: int, dev) -> float:
    if world == 1:
        return x
    t = torch.tensor([x], dtype=torch.float64, device=_coll_dev(dev))
    torch.distributed.all_reduce(t)
    return float(t.item())


# ---------------------------------------------------------------------------
def oracle_loop(sample_iters: int):
    """The config-2 workload's first `sample_iters` iterations for the CPU oracle
    (generated by synth: identical bits to the GPU inputs)."""
    import oracle as O
    import synth
    dev = "cuda" if torch.cuda.is_available() else "cpu"
    wl = synth.config2(n=N2, count=sample_iters, device=dev)
    return O, O.Loop(1, 1, sample_iters, wl.A.cpu().numpy(), X=wl.X.cpu().numpy(), c0=wl.c0)


def oracle_baseline(sample_iters: int, max_runs: int = 5, budget_s: float = 10.0):
    """The CPU oracle (oracle/jpo.c jpo_run_seq, single thread) timed on the
    box's host on a bounded sample of the same workload."""
    O, L = oracle_loop(sample_iters)
    O.run_seq_inplace(L)  # warm (and build) the .so
    old = os.sched_getaffinity(0)
    cpu = min(old)
    os.sched_setaffinity(0, {cpu})   # one core, as `taskset -c 0`
    try:
        times, t_end = [], time.perf_counter() + budget_s
        while not times or (len(times) < max_runs and time.perf_counter() < t_end):
            t0 = time.perf_counter()
            O.run_seq_inplace(L)
            times.append(time.perf_counter() - t0)
    finally:
        os.sched_setaffinity(0, old)
    t = statistics.median(times)
    return {"value": sample_iters / t, "unit": "iter/s", "cores": 1, "kind": "oracle", "cpu_model": _cpu_model(),
            "pinned_cpu": cpu,
            "sample": f"config2 SAXPY fp32, first {sample_iters} of the 2^28 iterations, jpo_run_seq on 1 host "
                      f"thread (pinned to cpu {cpu}) of {os.cpu_count()}, median of {len(times)} runs "
                      f"({t:.3f} s each)"}


# The paper's own numbers are context, not the target: another
# machine, another workload mix, a different program (Java + JNI + Fermi).
PAPER_CONTEXT = {
    "source": "Han, Zhang, Lam, Wang, ICPP'13 (PAPER.md L41-43 abstract; L471-491 Sec. VI setup)",
    "platform": "NVIDIA Tesla M2050 (Fermi, CUDA 3.2) + 2x Intel Xeon X5650 (12 cores), Java 1.6",
    "speedups_vs_serial_cpu": {"doall_loops": "10x (average)", "false_dependence_privatized": "2.5x",
                               "true_dependence_density_low": "2.14x"},
    "note": "speedups of whole Java applications over a 1-thread CPU run, on Fermi; the bench here reports "
            "committed iterations/s and HBM fraction of the loop hot path on one B200, with the CPU oracle "
            "(1 core) beside it"}


def _cpu_model() -> str:
    try:
        for line in open("/proc/cpuinfo"):
            if line.startswith("model name"):
                return line.split(":", 1)[1].strip()
    except OSError:
        pass
    return "unknown"


def arm_config(world: int, n_per_rank: int) -> dict:
    """The workload both arms report (the reference arm times the oracle on a
    bounded sample of it; its cpu_baseline.sample says which)."""
    return {"workload": "config2: DOALL streaming SAXPY fp32 Y=c0*X+Y, N=2^28, r=w=NULL",
            "n_total": N2, "n_per_rank": n_per_rank, "partition": "task sharing, equal weights",
            "l2": "inputs (3.2 GB) larger than L2 (126 MB); no flush needed",
            "parallelism": f"iteration-range sharding x{world}"}


def run_reference(args):
    """--impl reference: the oracle (the deliberately slow CPU program) on the
    host cores, each step a bounded 2^25-iteration sample of config 2."""
    world, rank, _ = dist_env()
    if rank != 0:
        return
    sample = 1 << 25
    O, L = oracle_loop(sample)
    times = []
    old = os.sched_getaffinity(0)
    os.sched_setaffinity(0, {min(old)})   # one host core (taskset -c 0)
    for k in range(args.warmup + args.steps):
        t0 = time.perf_counter()
        O.run_seq_inplace(L)
        if k >= args.warmup:
            times.append(time.perf_counter() - t0)
    os.sched_setaffinity(0, old)
    t = statistics.mean(times)
    v = sample / t
    print(json.dumps({"impl": "reference", "metric": METRIC, "value": v, "unit": "iter/s", "n_gpus": args.gpus,
                      "steps": args.steps, "warmup": args.warmup, "ms_per_step": t * 1e3,
                      "higher_is_better": True, "scaling": "strong", "vs_baseline": None, "dtype": "f32",
                      "data": "synthetic (synth.config2, seed 1002)",
                      "config": arm_config(args.gpus, N2 // args.gpus),
                      "cpu_baseline": {"value": v, "unit": "iter/s", "cores": 1, "kind": "oracle",
                                       "sample": f"first {sample} iterations of config2 per step, jpo_run_seq, "
                                                 f"1 host thread of {os.cpu_count()}"},
                      "e2e": {"value": v, "unit": "iter/s", "h2d_bytes_per_step": 0, "d2h_bytes_per_step": 0}}),
          flush=True)


# ---------------------------------------------------------------------------
def time_steps(fn, steps, st):
    """CUDA events on the launching stream around each step; returns per-step ms."""
    ev = [(torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)) for _ in range(steps)]
    for a, b in ev:
        a.record(st)
        fn()
        b.record(st)
    torch.cuda.synchronize()
    return [a.elapsed_time(b) for a, b in ev]


def median_timed(fn, A, A0, st, reps=None, budget_ms=2500.0):
    out, ts = None, []
    for k in range(3):   # warm-up
        if A is not None:
            A.copy_(A0)
        torch.cuda.synchronize()
        a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        a.record(st)
        out = fn()
        b.record(st)
        torch.cuda.synchronize()
        if k == 0 and a.elapsed_time(b) > 300:   # slow call: one warm-up is enough
            break
    first = a.elapsed_time(b)
    k = reps if reps is not None else int(min(20, max(3, budget_ms / max(first, 1e-3))))
    for _ in range(k):
        if A is not None:
            A.copy_(A0)
        torch.cuda.synchronize()
        a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        a.record(st)
        out = fn()
        b.record(st)
        torch.cuda.synchronize()
        ts.append(a.elapsed_time(b))
    return out, statistics.median(ts)


def pinned_oracle_rate(loop, budget_s: float = 1.0) -> float:
    """The CPU oracle (jpo_run_seq) on one host core (the calling thread pinned
    to the first allowed CPU, as `taskset -c 0` would), iterations per second:
    median of up to 5 runs within the budget."""
    import oracle as O
    old = os.sched_getaffinity(0)
    os.sched_setaffinity(0, {min(old)})
    try:
        ts, t_end = [], time.perf_counter() + budget_s
        while not ts or (len(ts) < 5 and time.perf_counter() < t_end):
            L = loop.copy()
            t0 = time.perf_counter()
            O.run_seq_inplace(L)
            ts.append(time.perf_counter() - t0)
    finally:
        os.sched_setaffinity(0, old)
    return loop.n / statistics.median(ts)


def crossover_sweep(jp, dev, st, n=1 << 20):
    """Reading A4's tau_high, measured (Fig. 2(b) "(Density > N)", P:L399-410;
    mode C P:L375-378): committed iter/s of the whole jp_schedule call with
    on-chip TLS (B7), restart TLS (A6) and the one-warp program-order path 7,
    against the 1-thread CPU oracle, over true-RAW densities 10-100%, for the
    config-3 recipe (delta <= 1024) and for chains (delta = 1: r[i] = w[i-1])."""
    import oracle as O
    import synth
    rows = []
    for delta in (1024, 1):
        for d in (0.10, 0.25, 0.50, 0.75, 0.90, 0.99, 0.999, 1.0):
            wl = synth.config3(d, n=n, delta=delta, device=dev)
            ref = O.Loop(wl.op, wl.dtype, wl.n, wl.A.cpu().numpy(), r=wl.r.cpu().numpy(), w=wl.w.cpu().numpy(),
                         c0=wl.c0)
            A0 = wl.A.clone()
            L = jp.Loop.from_workload(wl)
            ws = jp.workspace(L)
            row = {"delta": delta, "density": d}
            for name, kw in (("onchip", dict(tau_high=1.0, tls_recovery=2)),
                             ("restart", dict(tau_high=1.0, tls_recovery=1)),
                             ("serial_path7", dict(tau_high=1e-9))):
                res, ms = median_timed(lambda: jp.jp_schedule(L, ws, stream=st, **kw), wl.A, A0, st, budget_ms=1500)
                row[name] = n / (ms * 1e-3)
                row["raw_iters"] = res["prof"]["raw_iters"]
            row["oracle_1core"] = pinned_oracle_rate(ref)
            rows.append(row)
            del wl, ws, L, A0, ref
    out = {"rows": rows, "n": n, "unit": "committed iter/s, whole jp_schedule call, median"}
    for delta in (1024, 1):
        rs = [r for r in rows if r["delta"] == delta]
        tls_best = lambda r: max(r["onchip"], r["restart"])  # noqa: E731
        a = [r["density"] for r in rs if r["serial_path7"] >= tls_best(r)]
        b = [r["density"] for r in rs if r["oracle_1core"] > max(tls_best(r), r["serial_path7"])]
        out[f"delta{delta}"] = {"serial_beats_tls_from_density": min(a) if a else None,
                                "cpu_beats_gpu_from_density": min(b) if b else None}
    return out


def modes_sweep(jp, dev, st):
    """N=1 extras: TLS vs density (config 3), privatized (config 4), tiny (config 1), mixed (config 5)."""
    import synth
    out = {}
    hbm, _ = peaks()
    # config 3: TLS committed iterations/s vs true-RAW density.
    #  schedule:  the whole jp_schedule() call (profile -> Fig. 2(b) mode -> guide -> TLS), what a user runs;
    #             on this write-once loop it takes on-chip recovery (reading B7) on every SM
    #  tls:       that TLS run alone (jp_run_tls with jp_schedule's choices), kernel time
    #  profile / guide: jp_profile_density and jp_tls_guide alone
    #  restart_*: the same with restart recovery (reading A6: prefix commit, restart at the first violator)
    tls = []
    names = {1: "cta", 2: "grid", 3: "cluster16", 4: "tiny", 5: "onchip-cluster", 6: "onchip-grid",
             7: "serial-warp", 8: "onchip-one-window", 9: "onchip-one-window-waw"}

    def timed(fn, A, A0, reps=None):
        """warm up, then the median of `reps` timed runs (20, or
        fewer for calls slower than ~100 ms, so the sweep ends in minutes); the
        in-place array is restored from a pristine copy outside the timed region."""
        return median_timed(fn, A, A0, st, reps)

    for d in (0.001, 0.01, 0.05, 0.10):
        wl = synth.config3(d, device=dev)
        A0 = wl.A.clone()
        L = jp.Loop.from_workload(wl)
        ws = jp.workspace(L)
        row = {"density": d}
        for tag, rec in (("", 0), ("restart_", 1)):
            res, ms = timed(lambda: jp.jp_schedule(L, ws, stream=st, tls_recovery=rec), wl.A, A0)
            row["raw_iters"] = res["prof"]["raw_iters"]
            row[tag + "schedule"] = {"mode": res["mode_name"], "ms": ms, "committed_per_s": wl.n / (ms * 1e-3),
                                     "windows": res["tls"]["windows"], "violations": res["tls"]["violations"],
                                     "recovery": ["restart", "onchip"][res["tls_recovery"]],
                                     "window" if res["tls_recovery"] else "tls_w_max": res["tls_w_max"],
                                     "tls_path": names.get(res["tls_path"], "?"), "ctas": res["tls_cluster"],
                                     "guided": bool(res["tls_guided"])}
            prof = jp.jp_profile_density(L, ws)
            if res["tls_guided"]:
                jp.jp_tls_guide(L, ws)
            kw = dict(window=res["tls_w_max"], path=res["tls_path"], guided=bool(res["tls_guided"]), recovery=1) \
                if res["tls_recovery"] else \
                dict(window=0, w_max=res["tls_w_max"], path=res["tls_path"], guided=bool(res["tls_guided"]))
            s, ms = timed(lambda: jp.jp_run_tls(L, prof=prof, ws=ws, stream=st, **kw), wl.A, A0)
            row[tag + "tls"] = {"committed_per_s": s["committed"] / (ms * 1e-3), "ms": ms, "windows": s["windows"],
                                "violations": s["violations"], "executed_over_committed": s["executed"] / s["committed"],
                                "us_per_window": ms * 1e3 / s["windows"]}
        _, ms = timed(lambda: jp.jp_profile_density(L, ws, stream=st), wl.A, A0)
        row["profile_ms"] = ms
        _, ms = timed(lambda: jp.jp_tls_guide(L, ws, stream=st), wl.A, A0)
        row["guide_ms"] = ms
        tls.append(row)
        del wl, ws, L, A0
    out["config3_tls"] = tls
    # sensitivity run: dependence distances up to 2^20
    sens = []
    for d in (0.01, 0.10):
        wl = synth.config3(d, delta=1 << 20, device=dev)
        A0 = wl.A.clone()
        L = jp.Loop.from_workload(wl)
        ws = jp.workspace(L)
        row = {"density": d, "delta": 1 << 20}
        for tag, rec in (("", 0), ("restart_", 1)):
            res, ms = timed(lambda: jp.jp_schedule(L, ws, stream=st, tls_recovery=rec), wl.A, A0)
            row[tag + "schedule"] = {"mode": res["mode_name"], "ms": ms, "committed_per_s": wl.n / (ms * 1e-3),
                                     "windows": res["tls"]["windows"], "violations": res["tls"]["violations"],
                                     "recovery": ["restart", "onchip"][res["tls_recovery"]],
                                     "tls_w_max": res["tls_w_max"], "tls_path": names.get(res["tls_path"], "?")}
        sens.append(row)
        del wl, ws, L, A0
    out["config3_tls_delta_2e20"] = sens
    # config 3's shape WITH write-after-write (synth.config3_waw: w 2-to-1 onto half
    # the addresses): jp_schedule runs the one-window on-chip TLS fed by the last
    # earlier writer of every raw read (path 9, reading B14); the restart form
    # (reading A6, tls_recovery = 1, cap / path from the distance-hazard plan)
    # beside it
    waw = []
    for delta in (1024, 1 << 20):
        for d in (0.001, 0.01, 0.05, 0.10):
            wl = synth.config3_waw(d, delta=delta, device=dev)
            A0 = wl.A.clone()
            L = jp.Loop.from_workload(wl)
            ws = jp.workspace(L)
            row = {"density": d, "delta": delta}
            for tag, rec in (("", 0), ("restart_", 1)):
                res, ms = timed(lambda: jp.jp_schedule(L, ws, stream=st, tls_recovery=rec), wl.A, A0)
                row["raw_iters"] = res["prof"]["raw_iters"]
                row["waw_iters"] = res["prof"]["waw_iters"]
                row[tag + "schedule"] = {
                    "mode": res["mode_name"], "ms": ms, "committed_per_s": wl.n / (ms * 1e-3),
                    "windows": res["tls"]["windows"], "violations": res["tls"]["violations"],
                    "recovery": ["restart", "onchip"][res["tls_recovery"]], "tls_w_max": res["tls_w_max"],
                    "tls_path": names.get(res["tls_path"], "?"),
                    "us_per_window": ms * 1e3 / max(res["tls"]["windows"], 1)}
            waw.append(row)
            del wl, ws, L, A0
    out["config3_waw"] = waw
    # SAXPY with duplicate indirect writes (a scatter-add, raw = waw: the writers
    # of one address chain), N = 2^24 fp32: path 9 through jp_schedule
    sax = []
    for dup in (0.3, 0.7):
        g = torch.Generator(device="cpu").manual_seed(1017)
        n = 1 << 24
        m = int(n * (1 - dup)) + 1
        w = torch.randint(0, m, (n,), generator=g, dtype=torch.int32).to(dev)
        r = torch.randint(0, n, (n,), generator=g, dtype=torch.int32).to(dev)
        Y = (torch.randint(0, 1 << 23, (n,), generator=g).to(torch.float32) * 2.0 ** -22 - 1).to(dev)
        X = (torch.randint(0, 1 << 23, (n,), generator=g).to(torch.float32) * 2.0 ** -22 - 1).to(dev)
        Y0 = Y.clone()
        L = jp.Loop(jp.JP_OP_SAXPY, jp.JP_F32, n, Y, r=r, w=w, X=X, c0=1.1)
        ws = jp.workspace(L)
        res, ms = timed(lambda: jp.jp_schedule(L, ws, stream=st), Y, Y0)
        sax.append({"dup_frac": dup, "n": n, "mode": res["mode_name"], "ms": ms, "committed_per_s": n / (ms * 1e-3),
                    "raw_iters": res["prof"]["raw_iters"], "tls_path": names.get(res["tls_path"], "?"),
                    "windows": res["tls"]["windows"]})
        del L, ws, Y, Y0, X, r, w
    out["saxpy_scatter_add"] = sax
    out["crossover"] = crossover_sweep(jp, dev, st)
    # config 4: privatized.  The whole jp_schedule call (what a user runs: reading
    # B11 decides privatized without a profile, the s indices are checked on the
    # device, then stream + merge + apply), the privatized run alone, and the
    # profile alone (jp_profile_density: what Fig. 2(b) would have cost)
    wl = synth.config4(device=dev)
    L = jp.Loop.from_workload(wl)
    ws = jp.workspace(L)
    res, ms_call = timed(lambda: jp.jp_schedule(L, ws, stream=st), None, None)
    prof = jp.jp_profile_density(L, ws)
    _, ms_run = timed(lambda: jp.jp_run_privatized(L, prof, ws, stream=st), None, None)
    _, ms_prof = timed(lambda: jp.jp_profile_density(L, ws, stream=st), None, None)
    byt = BYTES_PER_ITER_PRIV * wl.n
    # back to back (a user's stream of calls): the call returns after the index
    # check, so the next call's host work overlaps this one's X -> Y phase
    kp = 20
    torch.cuda.synchronize()
    a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    a.record(st)
    for _ in range(kp):
        jp.jp_schedule(L, ws, stream=st)
    b.record(st)
    torch.cuda.synchronize()
    ms_pipe = a.elapsed_time(b) / kp
    out["config4_priv"] = {"n": wl.n, "mode": res["mode_name"], "profiled": res["profiled"],
                           "schedule_pipelined_ms": ms_pipe,
                           "schedule_pipelined_frac": byt / (ms_pipe * 1e-3) / 1e9 / hbm,
                           "schedule_ms": ms_call, "iters_per_s": wl.n / (ms_call * 1e-3),
                           "schedule_hbm_gbs": byt / (ms_call * 1e-3) / 1e9,
                           "schedule_frac": byt / (ms_call * 1e-3) / 1e9 / hbm,
                           "run_ms": ms_run, "run_frac": byt / (ms_run * 1e-3) / 1e9 / hbm,
                           "profile_ms": ms_prof,
                           "algorithmic_bytes": "12 B/iter (X, s read; Y written); the whole call's two-phase "
                                                "kernel checks the indices in its s phase (no extra bytes)",
                           "timing": "median of up to 20 single calls (CUDA events on the stream, idle GPU before each); pipelined: 20 back-to-back calls between two events"}
    del wl, ws, L
    # config 1: tiny loop, latency-bound (us per jp_schedule call, incl. profile + mode + run)
    c1 = {}
    for d in (0.0, 0.05):
        wl = synth.config1(d, device=dev)
        L = jp.Loop.from_workload(wl)
        ws = jp.workspace(L)
        for _ in range(20):
            res = jp.jp_schedule(L, ws, stream=st)
        ts = []
        for _ in range(200):   # jp_schedule syncs its stream: the call's wall time is the latency
            t0 = time.perf_counter()
            jp.jp_schedule(L, ws, stream=st)
            ts.append(time.perf_counter() - t0)
        # the CPU oracle on the same loop (sequential run, one host thread) for context
        import oracle as O
        ref = O.Loop(wl.op, wl.dtype, wl.n, wl.A.cpu().numpy(), r=wl.r.cpu().numpy(), w=wl.w.cpu().numpy(), c0=wl.c0)
        to = []
        for _ in range(200):
            t0 = time.perf_counter()
            O.run_seq_inplace(ref)
            to.append(time.perf_counter() - t0)
        c1[f"d{d}"] = {"mode": res["mode_name"], "us_per_call": statistics.median(ts) * 1e6,
                       "path": "tiny (one CTA: profile + mode + run, one launch)" if res.get("profiled") else "",
                       "oracle_us_per_call": statistics.median(to) * 1e6}
    out["config1"] = c1
    # config 5: mixed, stealing scheme on one GPU (per-chunk profile, tasks, concurrent batch)
    wl = synth.config5(device=dev)
    A0 = wl.A.clone()
    L = jp.Loop.from_workload(wl)
    ws = jp.workspace(L)
    res, ms = timed(lambda: jp.jp_schedule(L, ws, stream=st, scheme=jp.JP_SCHED_STEALING, chunk_iters=65536),
                    wl.A, A0)
    out["config5_mixed"] = {"n": wl.n, "iters_per_s": wl.n / (ms * 1e-3), "ms": ms, "n_tasks": res["n_tasks"],
                            "n_batches": res["n_batches"], "task_mode_iters": res["task_mode_iters"],
                            "tls": res["tls"], "timing": "median of up to 20, CUDA events on the stream"}
    del wl, ws, L, A0
    # workflows: the paper's task-stealing shapes, N = 2^24
    # iterations per original loop, every scheme; whole jp_schedule_workflow call
    wf = {}
    for name, fn in (("bicg", synth.workflow_bicg), ("2mm", synth.workflow_2mm), ("crypt", synth.workflow_crypt)):
        loops, arrays = fn(device=dev)
        init = [b.clone() for b in arrays]
        Ls = [jp.Loop.from_workload(x) for x in loops]
        wss = [jp.workspace(x) for x in Ls]
        row = {"loops": len(loops), "iters": sum(x.n for x in loops)}
        for sname, sch in (("sharing", jp.JP_SCHED_SHARING), ("stealing", jp.JP_SCHED_STEALING),
                           ("auto", jp.JP_SCHED_AUTO)):
            ts = []
            for rep in range(3):
                for b, b0 in zip(arrays, init):
                    b.copy_(b0)
                torch.cuda.synchronize()
                t0 = time.perf_counter()
                _, plan = jp.jp_schedule_workflow(Ls, wss, scheme=sch, stream=st)
                torch.cuda.synchronize()
                ts.append(time.perf_counter() - t0)
            t = min(ts[1:])
            row[sname] = {"ms": t * 1e3, "iters_per_s": row["iters"] / t, "n_batches": plan["n_batches"],
                          "scheme": ["sharing", "stealing"][plan["scheme"]]}
        wf[name] = row
        del loops, arrays, init, Ls, wss
    out["workflows"] = wf
    return out


def partitioned_config4(jp, dev, st, world, rank, steps):
    """Config 4 (PRIV_TMP fp32, N = 2^26, S = 1024) under task sharing across the
    ranks.  Profile (local stamp -> C1 MAX over 2 x 4 KiB -> local classify ->
    C3) timed separately from execution; one step = the
    privatized execution: local stream -> C4 (MAX over the 8 KiB packed keys)
    -> finalize.  Barrier, events on the launching stream, max over ranks."""
    import synth
    from paper_conf_icpp_hanzlw13_b200 import dist as jd
    wl = synth.config4(device=dev)
    full = jp.Loop.from_workload(wl)
    b, e = jd.sharing_ranges(wl.n, world)[rank]
    loop = full.range(b, e)
    ws = jp.workspace(loop)

    def timed(fn, k):
        for _ in range(3):
            fn()
        barrier(world)
        t0 = torch.cuda.Event(enable_timing=True)
        t1 = torch.cuda.Event(enable_timing=True)
        t0.record(st)
        for _ in range(k):
            fn()
        t1.record(st)
        barrier(world)
        return max_over_ranks(t0.elapsed_time(t1) / k, world, dev)

    prof = {}
    prof_ms = timed(lambda: prof.update(jd.profile_partitioned(loop, ws)), steps)
    mode = jp.jp_select_mode(loop, prof)
    ms = timed(lambda: jd.privatized_partitioned(loop, ws, prof), steps)
    hbm, _ = peaks()
    out = {"workload": "config4: PRIV_TMP fp32 N=2^26 S=1024, task sharing; step = privatized stream + C4 + finalize",
           "n": wl.n, "n_per_rank": e - b, "mode": jp.MODE_NAMES[mode], "ms": ms, "iters_per_s": wl.n / (ms * 1e-3),
           "per_rank_frac_of_hbm": BYTES_PER_ITER_PRIV * (e - b) / (ms * 1e-3) / 1e9 / hbm,
           "profile_ms": prof_ms, "collective": "torch.distributed all_reduce MAX (C4, 8 KiB int64) + finalize"}
    # C4 over peer memory as a separate single-CTA kernel (jp_keys_merge_p2p)
    if world > 1 and IPC_ROWS:
        try:
            handles = jd.p2p_handles(loop, ws)   # collective, once: the IPC mappings outlive the steps
            out["ms_p2p_merge"] = timed(lambda: jd.privatized_partitioned(loop, ws, prof, exchange="p2p", p2p=handles),
                                        steps)
            barrier(world)
            for h in handles.values():
                h.close()
        except Exception as ex:   # recorded, never fatal to the bench line
            out["ms_p2p_merge"] = f"error: {ex!r}"[:200]
    # C4 fused into the stream kernel (jp_priv_stream_merge): one launch per rank and
    # step, keys pushed into every rank's inbox over NVLink, replayed from a CUDA graph
    if IPC_ROWS:
        try:
            m = jd.PrivMerge(loop, ws)
            g = m.graph()
            fn = g.replay if g is not None else m.step
            fused_ms = timed(fn, steps)
            m.check()
            out["fused"] = {"ms": fused_ms, "iters_per_s": wl.n / (fused_ms * 1e-3),
                            "per_rank_frac_of_hbm": BYTES_PER_ITER_PRIV * (e - b) / (fused_ms * 1e-3) / 1e9 / hbm,
                            "cuda_graph": g is not None,
                            "what": "jp_priv_stream_merge: stream + C4 (peer stores + flags) + R2 in one cooperative "
                                    "kernel per rank; no NCCL call"}
            if world == 1:   # the merge's fixed cost on one rank: the same stream with its local finalize
                solo = timed(lambda: jp.jp_run_privatized(loop, prof, ws, stream=st), steps)
                out["fused"]["stream_alone_ms"] = solo
                out["fused"]["merge_fixed_cost_us"] = (fused_ms - solo) * 1e3
            barrier(world)
            m.close()
        except Exception as ex:
            out["fused"] = f"error: {ex!r}"[:200]
    return out


def partitioned_spill(jp, dev, st, world, rank, steps):
    """Config 2 under task sharing with cross-boundary spill (M1, C8): every rank
    runs jp_run_doall_spill over its shard and steals chunks (2^16 iterations,
    reading A17) descending from the most-loaded peer's shard over CUDA IPC.
    Step = counter reset + barrier + kernel + barrier; max over ranks.  At N = 1
    also a two-virtual-rank imbalance on one GPU: the second "rank" capped to 8
    CTAs (a slow device), static sharing vs spill, wall clock around both
    streams."""
    import synth
    from paper_conf_icpp_hanzlw13_b200 import dist as jd
    s0, s1 = jp.jp_plan_sharing(N2, world)[rank]
    wl = synth.config2(n=N2, device=dev, start=s0, count=s1 - s0)
    L = jp.Loop.from_workload(wl, iter_base=s0)
    sg = jd.SpillGroup(L)
    for _ in range(3):
        sg.run()
    kernel_ms = None
    if world == 1:   # the spill kernel alone (CUDA events on the launching stream)
        ctr = torch.zeros(1, dtype=torch.int64, device=dev)
        evs = []
        for _ in range(steps):
            ctr.zero_()
            a, z = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            a.record(st)
            jp.jp_run_doall_spill([L], 0, 1 << 16, ctr, None, 0, st)
            z.record(st)
            evs.append((a, z))
        torch.cuda.synchronize()
        kernel_ms = statistics.median([a.elapsed_time(z) for a, z in evs])
    ts, res = [], None
    for _ in range(steps):
        torch.cuda.synchronize()
        t0 = time.perf_counter()
        res = sg.run()
        ts.append(time.perf_counter() - t0)
    ms = max_over_ranks(statistics.median(ts) * 1e3, world, dev)
    sg.close()
    out = {"workload": "config2 SAXPY fp32 N=2^28, task sharing + spill (chunk 2^16)", "ms": ms,
           "iters_per_s": N2 / (ms * 1e-3), "rank0": res, "timing": "wall clock incl. 2 barriers, max over ranks"}
    if kernel_ms:
        out["kernel_ms"] = kernel_ms
        out["kernel_GBps"] = BYTES_PER_ITER_SAXPY * N2 / (kernel_ms * 1e-3) / 1e9
    del wl, L, sg
    if world == 1:
        hbm, _ = peaks()
        half = N2 // 2
        shards = [synth.config2(n=N2, device=dev, start=k * half, count=half) for k in range(2)]
        Ls = [jp.Loop.from_workload(x, iter_base=k * half) for k, x in enumerate(shards)]
        sts = [torch.cuda.Stream(), torch.cuda.Stream()]
        ctr = torch.zeros(2, dtype=torch.int64, device=dev)
        stats = torch.zeros(3, dtype=torch.int64, device=dev)

        def once(spill):
            ctr.zero_()
            stats.zero_()
            torch.cuda.synchronize()
            t0 = time.perf_counter()
            for k in range(2):
                views = Ls if spill else [Ls[k]]
                jp.jp_run_doall_spill(views, k if spill else 0, 1 << 16, ctr if spill else ctr[k:k + 1],
                                      stats if k == 0 else None, 0 if k == 0 else 8, sts[k])
            torch.cuda.synchronize()
            return time.perf_counter() - t0

        row = {}
        for name, spill in (("static", False), ("spill", True)):
            for _ in range(2):
                once(spill)
            t = statistics.median([once(spill) for _ in range(5)])
            row[name] = {"ms": t * 1e3, "iters_per_s": N2 / t, "GBps": BYTES_PER_ITER_SAXPY * N2 / t / 1e9}
            if spill:
                own, stolen, nst = (int(x) for x in stats.tolist())
                row[name].update({"fast_rank_own_iters": own, "fast_rank_stolen_iters": stolen})
        row["note"] = "2 virtual ranks on one GPU (separate shards, streams); rank 1 capped to 8 CTAs"
        out["imbalanced_2x1gpu"] = row
        del shards, Ls
    return out


def partitioned_config5(jp, dev, st, world, rank, steps):
    """Config 5 (mixed, N = 2^24) under the multi-rank task-stealing scheme
    (dist.schedule_stealing: partitioned profile with chunk counts -> tasks +
    PDG -> Alg. 1 plan -> batches with C4 merges; TLS pinned to rank 0).  One
    step = the whole call from pristine replicas; wall clock between barriers,
    max over ranks."""
    import synth
    from paper_conf_icpp_hanzlw13_b200 import dist as jd
    wl = synth.config5(device=dev)
    A0 = wl.A.clone()
    full = jp.Loop.from_workload(wl)
    ws = jp.workspace(full)
    ts, res = [], None
    for k in range(steps + 2):
        wl.A.copy_(A0)
        torch.cuda.synchronize()
        barrier(world)
        t0 = time.perf_counter()
        res = jd.schedule_stealing(full, ws, chunk_iters=65536)
        torch.cuda.synchronize()
        barrier(world)
        if k >= 2:
            ts.append(time.perf_counter() - t0)
    # one more call with per-phase CUDA events (not in the timing above); at one
    # rank the driver runs jp_schedule(STEALING): the multi-rank path itself is
    # timed too (force_ranks), with its phases
    wl.A.copy_(A0)
    barrier(world)
    ph = jd.schedule_stealing(full, ws, chunk_iters=65536, timings=True, force_ranks=True)["phases"]
    forced_ms = {}
    if world == 1:
        for prof_kind in ("replicated", "partitioned"):
            fts = []
            for k in range(6):
                wl.A.copy_(A0)
                torch.cuda.synchronize()
                t0 = time.perf_counter()
                jd.schedule_stealing(full, ws, chunk_iters=65536, force_ranks=True, profile=prof_kind)
                torch.cuda.synchronize()
                if k >= 1:
                    fts.append(time.perf_counter() - t0)
            forced_ms[prof_kind] = statistics.median(fts) * 1e3
    # device-side stealing (jp_run_priv_claim): chunks claimed at run time
    dts, dres = [], {"rank_work": "skipped: CUDA-IPC rows turned off (JP_BENCH_IPC=0)"}
    try:
        for k in range(4 if world == 1 or IPC_ROWS else 0):
            wl.A.copy_(A0)
            torch.cuda.synchronize()
            barrier(world)
            t0 = time.perf_counter()
            dres = jd.schedule_stealing(full, ws, chunk_iters=65536, dynamic=True)
            torch.cuda.synchronize()
            barrier(world)
            if k >= 1:
                dts.append(time.perf_counter() - t0)
    except Exception as ex:   # recorded, never fatal to the bench line
        dts, dres = [], {"rank_work": f"error: {ex!r}"[:200]}
    dyn_ms = max_over_ranks(statistics.median(dts) * 1e3, world, dev) if dts else None
    phases = {k: max_over_ranks(v, world, dev) for k, v in ph.items()}
    busy = [0.0] * world
    if world > 1:
        bt = torch.zeros(world, dtype=torch.float64, device=dev)
        bt[rank] = ph["busy_ms"]
        torch.distributed.all_reduce(bt)
        busy = bt.tolist()
    else:
        busy = [ph["busy_ms"]]
    n_stolen = res["stolen"]
    ms = max_over_ranks(statistics.median(ts) * 1e3, world, dev)
    out = {"workload": "config5 mixed ADD_C int32 N=2^24, multi-rank task stealing (chunk 2^16)", "ms": ms,
           "iters_per_s": wl.n / (ms * 1e-3), "n_tasks": res["n_tasks"], "n_batches": res["n_batches"],
           "rank0_iters": res["rank_work"]["iters"], "tls": res["tls"], "phases_max_over_ranks": phases,
           "busy_ms_per_rank": busy, "stolen_chunks": n_stolen, "multi_rank_path_ms_at_one_rank": forced_ms,
           "delegated": res.get("delegated"),
           "dynamic": {"ms": dyn_ms, "iters_per_s": wl.n / (dyn_ms * 1e-3) if dyn_ms else None,
                       "rank0": dres["rank_work"],
                       "what": "the batch's partitioned chunks claimed on the device (jp_run_priv_claim)"},
           "merge": "C4 all_reduce MAX over 2^24 int64 keys (128 MiB) + apply, per batch",
           "timing": "wall clock between barriers, max over ranks"}
    del wl, A0, full, ws
    return out


def exchange_cost(jp, dev, st):
    """NEXT-2 on one GPU: rank 0 of 8 of config 3 (d = 1%) and config 5's
    privatized tail: what the owner form sends vs the dense all_reduce, and the
    time of its local kernels (pack, reduce, gather, scatter).  The all_to_all
    itself needs several GPUs (unmeasured here)."""
    import synth
    from paper_conf_icpp_hanzlw13_b200 import dist as jd
    out = {}
    world = 8
    wl = synth.config3(0.01, device=dev)
    full = jp.Loop.from_workload(wl)
    b, e = jd.sharing_ranges(wl.n, world)[0]
    loop = full.range(b, e)
    ws = jp.workspace(loop)
    jp.jp_profile_stamp(loop, ws)
    W = jd._region(ws, loop, "minW_A", torch.int32, jp)
    R = jd._region(ws, loop, "minR_A", torch.int32, jp)

    def ev(fn, k=5):
        fn()
        a, z = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        torch.cuda.synchronize()
        a.record(st)
        for _ in range(k):
            fn()
        z.record(st)
        torch.cuda.synchronize()
        return a.elapsed_time(z) / k

    rows, counts = jp.jp_sparse_pack(W, R, -1, world)
    pack_ms = ev(lambda: jp.jp_sparse_pack(W, R, -1, world))
    R2 = rows.clone()
    red_ms = ev(lambda: jp.jp_sparse_reduce_max(W, R, R2))
    gat_ms = ev(lambda: jp.jp_sparse_gather(W, R, R2))
    sca_ms = ev(lambda: jp.jp_sparse_scatter(W, R, R2))
    dense = 2 * W.numel() * 4
    out["config3_profile_C1"] = {
        "rank_range": e - b, "rows": int(rows.shape[0]), "rows_per_owner": counts,
        "owner_bytes_sent_per_rank": 2 * rows.numel() * 4, "dense_table_bytes": dense,
        "dense_allreduce_bytes_sent_per_rank_ring": 2 * (world - 1) / world * dense,
        "pack_ms": pack_ms, "reduce_ms": red_ms, "gather_ms": gat_ms, "scatter_ms": sca_ms}
    del wl, full, loop, ws, W, R, rows, R2
    torch.cuda.empty_cache()
    return out


# Rows that map peer memory through CUDA IPC (spill, p2p and fused C4, device-side
# stealing) run at every N (JP_BENCH_IPC=0 turns them off); each is wrapped so an
# error is recorded in its row instead of ending the run, and every device-side
# wait has a timeout.
IPC_ROWS = os.environ.get("JP_BENCH_IPC", "1") == "1"


def run_jp(args):
    import paper_conf_icpp_hanzlw13_b200 as jp
    import synth
    world, rank, local = dist_env()
    if world != args.gpus:
        raise SystemExit(f"--gpus {args.gpus} but WORLD_SIZE={world}: launch N>1 with torchrun")
    # one process per GPU over NCCL; JP_DIST_BACKEND=gloo lets several ranks share
    # the GPUs of a smaller box to exercise the multi-rank code path (test mode)
    backend = os.environ.get("JP_DIST_BACKEND", "nccl")
    dev = torch.device("cuda", local % torch.cuda.device_count())
    torch.cuda.set_device(dev)
    if world > 1:
        if backend == "nccl":
            torch.distributed.init_process_group("nccl", device_id=dev)
        else:
            torch.distributed.init_process_group(backend)
    st = torch.cuda.current_stream()
    # task sharing: equal weights on identical B200s (reading A15)
    s0, s1 = jp.jp_plan_sharing(N2, world)[rank]
    wl = synth.config2(n=N2, device=dev, start=s0, count=s1 - s0)
    L = jp.Loop.from_workload(wl, iter_base=s0)
    step = lambda: jp.jp_schedule(L, None, stream=st)  # noqa: E731  (static DOALL: no workspace needed)
    for _ in range(args.warmup):
        step()
    clk = Clocks(local).start()
    barrier(world)
    n_launch0 = jp.jp_launch_count()
    clk.mark_start()
    t0 = torch.cuda.Event(enable_timing=True)
    t1 = torch.cuda.Event(enable_timing=True)
    t0.record(st)
    per_step = time_steps(step, args.steps, st)
    t1.record(st)
    barrier(world)
    clk.mark_end()
    clk.stop()
    launches = jp.jp_launch_count() - n_launch0
    total_ms = max_over_ranks(t0.elapsed_time(t1), world, dev)
    kernel_ms = max_over_ranks(statistics.mean(per_step), world, dev)
    value = N2 * args.steps / (total_ms * 1e-3)
    hbm, peak_src = peaks()
    achieved = BYTES_PER_ITER_SAXPY * (s1 - s0) / (kernel_ms * 1e-3) / 1e9
    # ncu DRAM bytes per launch of the whole 2^28 step (profiles/ncu_doall_traffic.json,
    # one `ncu --set full` capture of this command at N = 1), scaled to this rank's
    # share of the iterations (the kernel streams its range exactly once)
    traffic = None
    tp = os.path.join(ROOT, "profiles", "ncu_doall_traffic.json")
    if os.path.exists(tp):
        full = json.load(open(tp)).get("dram_bytes_per_launch")
        traffic = None if full is None else full * (s1 - s0) / N2

    # e2e: the same step through jp_schedule_host with pinned host buffers
    e2e_steps = min(args.steps, 3)
    hA, hX = wl.A.cpu().pin_memory(), wl.X.cpu().pin_memory()
    Lh = jp.Loop(1, 1, s1 - s0, hA, X=hX, c0=wl.c0, iter_base=s0)
    stage = torch.empty(jp.jp_stage_bytes(Lh), dtype=torch.uint8, device=dev)
    jp.jp_schedule_host(Lh, stage, None, stream=st)
    barrier(world)
    te = time.perf_counter()
    for _ in range(e2e_steps):
        jp.jp_schedule_host(Lh, stage, None, stream=st)
    barrier(world)
    e2e_s = max_over_ranks(time.perf_counter() - te, world, dev)
    e2e = {"value": N2 * e2e_steps / e2e_s, "unit": "iter/s",
           "h2d_bytes_per_step": int(sum_over_ranks(8 * (s1 - s0), world, dev)),
           "d2h_bytes_per_step": int(sum_over_ranks(4 * (s1 - s0), world, dev)),
           "api": "jp_schedule_host (pinned host X,Y -> H2D -> DOALL -> D2H Y)"}
    # the copy-only bound of the same step: X, Y up and Y down on two streams, no kernel
    dX = stage[:4 * (s1 - s0)].view(torch.float32)
    dY = stage[4 * (s1 - s0):8 * (s1 - s0)].view(torch.float32)
    su, sd = torch.cuda.Stream(), torch.cuda.Stream()

    def copies():
        with torch.cuda.stream(su):
            dX.copy_(hX, non_blocking=True)
            dY.copy_(hA, non_blocking=True)
        with torch.cuda.stream(sd):
            hA.copy_(dY, non_blocking=True)
    copies()
    torch.cuda.synchronize()
    tc = time.perf_counter()
    copies()
    torch.cuda.synchronize()
    tc = max_over_ranks(time.perf_counter() - tc, world, dev)
    e2e["pcie_copy_only_bound"] = N2 / tc
    e2e["frac_of_copy_bound"] = e2e["value"] / (N2 / tc)
    del stage, hA, hX
    launches_all = int(sum_over_ranks(launches, world, dev))
    # C7: gathering the sharded output on rank 0 is reported
    # separately and is not in T(k)
    gather = None
    if world > 1:
        try:
            outs = [torch.empty_like(wl.A) for _ in range(world)] if rank == 0 else None
            barrier(world)
            g0, g1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            g0.record(st)
            torch.distributed.gather(wl.A, outs, dst=0)
            g1.record(st)
            barrier(world)
            gms = max_over_ranks(g0.elapsed_time(g1), world, dev)
            gather = {"ms": gms, "bytes_to_rank0": 4 * (N2 - (s1 - s0)), "GBps": 4 * (N2 - (s1 - s0)) / (gms * 1e-3) / 1e9,
                      "what": "torch.distributed.gather of every rank's Y shard to rank 0 (C7), after the timed steps"}
            del outs
        except Exception as ex:   # e.g. the gloo test mode with device tensors
            gather = {"error": repr(ex)[:200]}

    out = None
    if rank == 0:
        out = {"metric": METRIC, "value": value, "unit": "iter/s", "n_gpus": world, "steps": args.steps,
               "warmup": args.warmup, "ms_per_step": total_ms / args.steps, "higher_is_better": True,
               "scaling": "strong", "vs_baseline": None, "dtype": "f32",
               "data": "synthetic (synth.config2 counter-based generator, seed 1002), resident in HBM",
               "config": arm_config(world, s1 - s0),
               "roofline": {"bound": "hbm", "kernel": ["k_doall_affine_vec<SAXPY,F32>",
                                                        "k_doall_affine_tma<SAXPY,F32>"][jp.jp_doall_kernel(-1)],
                            "achieved": achieved,
                            "peak": hbm, "unit": "GB/s", "frac": achieved / hbm, "traffic": traffic,
                            "traffic_source": "ncu dram__bytes_read.sum + dram__bytes_write.sum per launch "
                                              "(profiles/ncu_doall_traffic.json, N=1), x this rank's share",
                            "algorithmic_bytes_per_iter": BYTES_PER_ITER_SAXPY, "peak_source": peak_src,
                            "kernel_ms": kernel_ms},
               "clocks": clk.summary(), "e2e": e2e, "gpu_launches": launches_all, "paper_context": PAPER_CONTEXT,
               "gather_to_one": gather}
    if not args.no_modes:
        del wl, L
        torch.cuda.empty_cache()
        part = partitioned_config4(jp, dev, st, world, rank, 5)
        torch.cuda.empty_cache()
        try:
            spill = partitioned_spill(jp, dev, st, world, rank, 5) if world == 1 or IPC_ROWS else \
                {"skipped": "CUDA-IPC rows turned off (JP_BENCH_IPC=0)"}
        except Exception as ex:   # recorded, never fatal to the bench line
            spill = {"error": repr(ex)[:200]}
        torch.cuda.empty_cache()
        steal = partitioned_config5(jp, dev, st, world, rank, 10)
        torch.cuda.empty_cache()
        if rank == 0:
            out["partitioned"] = {"config4": part, "config2_spill": spill, "config5_stealing": steal}
        if world == 1:
            out["modes"] = modes_sweep(jp, dev, st)
            out["modes"]["exchange_owner"] = exchange_cost(jp, dev, st)
    if rank == 0:
        out["cpu_baseline"] = oracle_baseline(1 << 25)
        print(json.dumps(out), flush=True)
    if world > 1:
        torch.distributed.destroy_process_group()


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--gpus", type=int, default=1)
    ap.add_argument("--steps", type=int, default=20)
    ap.add_argument("--warmup", type=int, default=5)
    ap.add_argument("--impl", default="jp", choices=["jp", "reference"])
    ap.add_argument("--no-modes", action="store_true", help="skip the N=1 modes sweep")
    args = ap.parse_args()
    if args.warmup < 3:
        raise SystemExit("--warmup must be >= 3")
    if args.impl == "reference":
        run_reference(args)
    else:
        run_jp(args)


if __name__ == "__main__":
    main()
