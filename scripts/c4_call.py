#!/usr/bin/env python
"""Config 4 whole jp_schedule call vs the privatized run alone (median of 20, CUDA events)."""
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import torch  # noqa: E402

import bench  # noqa: E402
import paper_conf_icpp_hanzlw13_b200 as jp  # noqa: E402
import synth  # noqa: E402

st = torch.cuda.current_stream()
wl = synth.config4(device="cuda")
L = jp.Loop.from_workload(wl)
ws = jp.workspace(L)
res, ms = bench.median_timed(lambda: jp.jp_schedule(L, ws, stream=st), None, None, st, 20)
prof = jp.jp_profile_density(L, ws)
_, ms_run = bench.median_timed(lambda: jp.jp_run_privatized(L, prof, ws, stream=st), None, None, st, 20)
hbm, _ = bench.peaks()
print(f"config4 jp_schedule {ms:.4f} ms ({12 * wl.n / ms / 1e6 / hbm:.3f} of HBM), run alone {ms_run:.4f} ms, "
      f"mode {res['mode_name']} profiled {res['profiled']}")
torch.cuda.synchronize()
a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
a.record(st)
for _ in range(20):
    jp.jp_schedule(L, ws, stream=st)
b.record(st)
torch.cuda.synchronize()
mp = a.elapsed_time(b) / 20
print(f"config4 jp_schedule back to back: {mp:.4f} ms per call ({12 * wl.n / mp / 1e6 / hbm:.3f} of HBM)")
