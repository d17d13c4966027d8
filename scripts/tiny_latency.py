#!/usr/bin/env python
"""Config 1 latency breakdown: wall time of jp_schedule (Python call -> C ->
one launch -> D2H -> sync) vs the tiny kernel alone (CUDA events)."""
import json
import os
import statistics
import sys
import time

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import paper_conf_icpp_hanzlw13_b200 as jp  # noqa: E402
import synth  # noqa: E402

dev = torch.device("cuda:0")
st = torch.cuda.current_stream()
for d in (0.0, 0.05):
    wl = synth.config1(d, device=dev)
    L = jp.Loop.from_workload(wl)
    ws = jp.workspace(L)
    cfg = jp.sched_cfg()
    for _ in range(5):
        jp.jp_schedule(L, ws, cfg=cfg, stream=st)
    wall, gpu = [], []
    for _ in range(50):
        a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        torch.cuda.synchronize()
        t0 = time.perf_counter()
        a.record(st)
        res = jp.jp_schedule(L, ws, cfg=cfg, stream=st)
        b.record(st)
        torch.cuda.synchronize()
        wall.append((time.perf_counter() - t0) * 1e6)
        gpu.append(a.elapsed_time(b) * 1e3)
    print(json.dumps({"d": d, "mode": res["mode_name"], "wall_us_median": statistics.median(wall),
                      "wall_us_min": min(wall), "gpu_us_median": statistics.median(gpu),
                      "windows": res["tls"]["windows"]}), flush=True)
