"""Summarise an ncu --set full report and a launch list into profiles/<tag>/.

    python tools/summarize_ncu.py <tag> [gpurun_out/prof_<tag>.ncu-rep] [gpurun_out/launches_<tag>.csv]

Writes profiles/<tag>/summary.md (per-kernel duration, DRAM bytes, throughput,
pipe utilisation, occupancy, instruction counts; launch-list shares) and
profiles/spmv_traffic.json (DRAM bytes per protected-SpMV launch, read by
bench.py's roofline.traffic).
"""
import collections
import csv
import io
import json
import os
import subprocess
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
METRICS = [
    ("gpu__time_duration.sum", "dur"),
    ("dram__bytes_read.sum", "dram_rd"),
    ("dram__bytes_write.sum", "dram_wr"),
    ("gpu__dram_throughput.avg.pct_of_peak_sustained_elapsed", "dram%"),
    ("sm__throughput.avg.pct_of_peak_sustained_elapsed", "sm%"),
    ("smsp__issue_active.avg.pct_of_peak_sustained_active", "issue%"),
    ("sm__inst_executed_pipe_alu.avg.pct_of_peak_sustained_active", "alu%"),
    ("sm__inst_executed_pipe_fma.avg.pct_of_peak_sustained_active", "fma%"),
    ("sm__inst_executed_pipe_lsu.avg.pct_of_peak_sustained_active", "lsu%"),
    ("sm__pipe_fp64_cycles_active.avg.pct_of_peak_sustained_active", "fp64%"),
    ("sm__warps_active.avg.pct_of_peak_sustained_active", "occ%"),
    ("launch__registers_per_thread", "regs"),
    ("smsp__inst_executed.sum", "warp_inst"),
]
SCALE = {"byte": 1, "Kbyte": 1e3, "Mbyte": 1e6, "Gbyte": 1e9, "Tbyte": 1e12,
         "ns": 1e-3, "us": 1, "usecond": 1, "ms": 1e3, "msecond": 1e3, "nsecond": 1e-3}


def load_raw(rep):
    out = subprocess.run(["ncu", "-i", rep, "--page", "raw", "--csv"], capture_output=True, text=True).stdout
    rows = list(csv.reader(io.StringIO(out)))
    return rows[0], rows[1], rows[2:]


def main():
    tag = sys.argv[1]
    rep = sys.argv[2] if len(sys.argv) > 2 else os.path.join(ROOT, "gpurun_out", f"prof_{tag}.ncu-rep")
    lau = sys.argv[3] if len(sys.argv) > 3 else os.path.join(ROOT, "gpurun_out", f"launches_{tag}.csv")
    outdir = os.path.join(ROOT, "profiles", tag)
    os.makedirs(outdir, exist_ok=True)
    lines = [f"# ncu summary {tag}", ""]
    per = collections.OrderedDict()
    if os.path.exists(rep):
        hdr, units, rows = load_raw(rep)
        with open(os.path.join(outdir, "ncu_full_raw.csv"), "w") as f:
            w = csv.writer(f)
            w.writerow(hdr)
            w.writerow(units)
            w.writerows(rows)
        ki = hdr.index("Kernel Name")
        for r in rows:
            k = r[ki].split("(")[0]
            d = {}
            for m, short in METRICS:
                if m in hdr:
                    i = hdr.index(m)
                    try:
                        v = float(r[i].replace(",", ""))
                    except ValueError:
                        continue
                    v *= SCALE.get(units[i], 1)
                    d[short] = v
            per.setdefault(k, []).append(d)
        lines += ["## ncu --set full (cold-cache, serialised replays; compare shares, not absolutes)", "",
                  "| kernel | launches | dur us | DRAM read MB | DRAM write MB | DRAM % | SM % | issue % | ALU % |"
                  " FMA % | LSU % | FP64 % | occupancy % | regs | warp-inst (M) |",
                  "|---|---|---|---|---|---|---|---|---|---|---|---|---|---|---|"]
        for k, ds in per.items():
            avg = {m: sum(d.get(m, 0) for d in ds) / len(ds) for _, m in METRICS}
            lines.append(f"| `{k}` | {len(ds)} | {avg['dur']:.1f} | {avg['dram_rd'] / 1e6:.1f} | {avg['dram_wr'] / 1e6:.1f} |"
                         f" {avg['dram%']:.1f} | {avg['sm%']:.1f} | {avg['issue%']:.1f} | {avg['alu%']:.1f} |"
                         f" {avg['fma%']:.1f} | {avg['lsu%']:.1f} | {avg['fp64%']:.1f} | {avg['occ%']:.1f} |"
                         f" {avg['regs']:.0f} | {avg['warp_inst'] / 1e6:.1f} |")
            # the protected CG SpMV of the bench (tiled path; the generic kernel in old reports)
            if "k_spmv_tile<2, 2, 2, 1" in k or "k_spmv<2, 2, 2, 1>" in k:
                json.dump({"kernel": k, "bytes_per_launch": avg["dram_rd"] + avg["dram_wr"],
                           "read": avg["dram_rd"], "write": avg["dram_wr"], "source": f"profiles/{tag}/ncu_full_raw.csv",
                           "dur_us_under_ncu": avg["dur"]},
                          open(os.path.join(ROOT, "profiles", "spmv_traffic.json"), "w"), indent=1)
        lines.append("")
    if os.path.exists(lau):
        rows = list(csv.reader(open(lau)))
        start = next(i for i, r in enumerate(rows) if "Kernel Name" in r)
        hdr = rows[start]
        ki, vi = hdr.index("Kernel Name"), hdr.index("Metric Value")
        agg = collections.defaultdict(lambda: [0, 0.0])
        for r in rows[start + 1:]:
            try:
                v = float(r[vi].replace(",", ""))
            except (ValueError, IndexError):
                continue
            k = r[ki].split("(")[0]
            if "abft::" not in k:
                continue
            agg[k][0] += 1
            agg[k][1] += v
        tot = sum(t for _, t in agg.values())
        lines += ["## launch list (ncu gpu__time_duration, our kernels only)", "",
                  "| kernel | launches | avg us | share of our kernel time |", "|---|---|---|---|"]
        for k, (n, t) in sorted(agg.items(), key=lambda x: -x[1][1]):
            lines.append(f"| `{k}` | {n} | {t / n / 1e3:.2f} | {100 * t / tot:.1f}% |")
        lines.append("")
    open(os.path.join(outdir, "summary.md"), "w").write("\n".join(lines))
    print("\n".join(lines))


if __name__ == "__main__":
    main()
