#!/usr/bin/env python
"""Summaries of ncu launch lists (CSV from --metrics ... --csv) and full
captures (.ncu-rep, read with `ncu -i --page raw --csv`) for profiles/.

  python scripts/ncu_summary.py launches FILE.csv [--skip N]
  python scripts/ncu_summary.py full FILE.ncu-rep
"""
import csv
import subprocess
import sys


def launches(path, skip=0):
    rows = list(csv.reader(open(path)))
    hdr, out = None, {}
    for r in rows:
        if "Kernel Name" in r:
            hdr = r
            continue
        if hdr and len(r) == len(hdr):
            d = dict(zip(hdr, r))
            out.setdefault((int(d["ID"]), d["Kernel Name"].split("(")[0][:60]), {})[d["Metric Name"]] = \
                float(d["Metric Value"].replace(",", ""))
    print("| launch | kernel | us | DRAM read MB | DRAM write MB |")
    print("|---|---|---|---|---|")
    for (i, k), v in sorted(out.items()):
        if i < skip:
            continue
        print(f"| {i} | `{k}` | {v.get('gpu__time_duration.sum', 0) / 1e3:.1f} | "
              f"{v.get('dram__bytes_read.sum', 0) / 1e6:.1f} | {v.get('dram__bytes_write.sum', 0) / 1e6:.1f} |")


KEYS = ["gpu__time_duration.sum", "dram__bytes_read.sum", "dram__bytes_write.sum",
        "gpu__dram_throughput.avg.pct_of_peak_sustained_elapsed", "sm__throughput.avg.pct_of_peak_sustained_elapsed",
        "lts__t_sectors_op_atom.sum", "lts__t_sectors_op_red.sum", "sm__warps_active.avg.pct_of_peak_sustained_active",
        "smsp__issue_active.avg.pct_of_peak_sustained_active", "launch__registers_per_thread", "launch__grid_size",
        "launch__block_size", "l1tex__data_bank_conflicts_pipe_lsu_mem_shared.sum"]


def full(path):
    txt = subprocess.run(["ncu", "-i", path, "--page", "raw", "--csv"], capture_output=True, text=True).stdout
    rows = list(csv.reader(txt.splitlines()))
    hdr, units = rows[0], rows[1]
    for r in rows[2:]:
        print(f"### `{r[hdr.index('Kernel Name')][:90]}`")
        for k in KEYS:
            if k in hdr:
                print(f"- {k}: {r[hdr.index(k)]} {units[hdr.index(k)]}")
        st = []
        for i, h in enumerate(hdr):
            if "issue_stalled" in h and h.endswith("per_issue_active.ratio"):
                try:
                    st.append((float(r[i]), h.replace("smsp__average_warps_issue_stalled_", "").replace(
                        "_per_issue_active.ratio", "")))
                except ValueError:
                    pass
        st.sort(reverse=True)
        print("- top stalls (warps per issue): " + ", ".join(f"{h} {v:.2f}" for v, h in st[:4]))
        print()


if __name__ == "__main__":
    if sys.argv[1] == "launches":
        launches(sys.argv[2], int(sys.argv[4]) if len(sys.argv) > 4 else 0)
    else:
        full(sys.argv[2])
