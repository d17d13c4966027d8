#!/usr/bin/env python
"""TLS design sweep on one B200 (config 3, N = 2^24): single-CTA hash path vs
the cluster path at several cluster sizes, fixed W = 4096 and adaptive windows.
Prints one JSON object per line (ms, committed iter/s, us/window).

  python scripts/tls_sweep.py [--n LOG2N] [--dens 0.001,0.01,0.05,0.1]
"""
import argparse
import json
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import torch  # noqa: E402

import paper_conf_icpp_hanzlw13_b200 as jp  # noqa: E402
import synth  # noqa: E402


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--n", type=int, default=24)
    ap.add_argument("--dens", default="0.001,0.01,0.05,0.1")
    ap.add_argument("--variants", default="all")
    args = ap.parse_args()
    dev = torch.device("cuda:0")
    st = torch.cuda.current_stream()
    # (name, path, cluster, window, w_max, guided)
    variants = []
    for g in (False, True):
        variants += [("cta", 1, 0, 4096, 4096, g)]
        variants += [("cta", 1, 0, 0, wm, g) for wm in (512, 1024, 2048, 4096)]
        for c in (4, 8, 16):
            variants += [(f"cl{c}", 3, c, 4096, 4096, g)]
            variants += [(f"cl{c}", 3, c, 0, wm, g) for wm in (1024, 2048, 4096)]
        variants += [("cl16", 3, 16, 0, 65024, g)]
    if args.variants == "small":
        variants = [("cta", 1, 0, 0, wm, g) for g in (False, True) for wm in (256, 512, 1024)]
    elif args.variants == "wmax":
        variants = [("cta", 1, 0, 0, wm, g) for g in (False, True) for wm in (128, 256, 384, 512, 768, 1024, 1536)]
    elif args.variants != "all":
        keep = set(args.variants.split(","))
        variants = [v for v in variants if v[0] in keep]
    for d in [float(x) for x in args.dens.split(",")]:
        wl = synth.config3(d, n=1 << args.n, device=dev)
        A0 = wl.A.clone()
        L = jp.Loop.from_workload(wl)
        ws = jp.workspace(L)
        prof = jp.jp_profile_density(L, ws)
        ref = None
        jp.jp_tls_guide(L, ws)
        for name, path, cl, window, wmax, guided in variants:
            kw = dict(window=window, w_max=wmax, path=path, cluster=cl, prof=prof, ws=ws, stream=st, guided=guided)
            wl.A.copy_(A0)
            jp.jp_run_tls(L, **kw)
            torch.cuda.synchronize()
            out = wl.A.clone()
            wl.A.copy_(A0)
            torch.cuda.synchronize()
            a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            a.record(st)
            s = jp.jp_run_tls(L, **kw)
            b.record(st)
            torch.cuda.synchronize()
            ms = a.elapsed_time(b)
            if ref is None:
                ref = out
            same = bool(torch.equal(out, ref)) and bool(torch.equal(wl.A, ref))
            print(json.dumps({"d": d, "variant": name, "guided": guided, "window": window, "w_max": wmax, "ms": round(ms, 3),
                              "committed_per_s": s["committed"] / (ms * 1e-3), "windows": s["windows"],
                              "us_per_window": round(ms * 1e3 / s["windows"], 3),
                              "exec_over_commit": round(s["executed"] / s["committed"], 3),
                              "same_result": same}), flush=True)
        del wl, A0, L, ws
        torch.cuda.empty_cache()


if __name__ == "__main__":
    main()
