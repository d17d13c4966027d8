#!/usr/bin/env python
"""Config 5 jp_schedule(STEALING), median of 20 (CUDA events)."""
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import torch  # noqa: E402

import bench  # noqa: E402
import paper_conf_icpp_hanzlw13_b200 as jp  # noqa: E402
import synth  # noqa: E402

st = torch.cuda.current_stream()
wl = synth.config5(device="cuda")
A0 = wl.A.clone()
L = jp.Loop.from_workload(wl)
ws = jp.workspace(L)
res, ms = bench.median_timed(lambda: jp.jp_schedule(L, ws, stream=st, scheme=jp.JP_SCHED_STEALING, chunk_iters=65536),
                             wl.A, A0, st, 20)
print(f"config5 {ms:.4f} ms = {wl.n / ms / 1e6:.2f} G iter/s, tls path {res['tls_path']}, tls {res['tls']}")
