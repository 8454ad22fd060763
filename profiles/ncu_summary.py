"""Summarise an ncu --set full report (per launch: duration, DRAM bytes, throughput, occupancy,
issue activity, smem wavefronts and bank conflicts, top stall reasons) -> text."""
import csv
import io
import subprocess
import sys

KEYS = [
    ("gpu__time_duration.sum", "duration"),
    ("dram__bytes_read.sum", "dram read"),
    ("dram__bytes_write.sum", "dram write"),
    ("dram__throughput.avg.pct_of_peak_sustained_elapsed", "dram % of peak"),
    ("sm__throughput.avg.pct_of_peak_sustained_elapsed", "SM % of peak"),
    ("smsp__issue_active.avg.pct_of_peak_sustained_active", "issue active %"),
    ("sm__warps_active.avg.pct_of_peak_sustained_active", "warps active %"),
    ("smsp__inst_executed.sum", "warp instructions"),
    ("l1tex__data_pipe_lsu_wavefronts_mem_shared.sum", "smem wavefronts"),
    ("l1tex__data_bank_conflicts_pipe_lsu_mem_shared.sum", "smem bank conflicts"),
    ("launch__registers_per_thread", "registers/thread"),
    ("launch__grid_size", "grid"),
    ("launch__block_size", "block"),
]


def main(rep):
    out = subprocess.run(["ncu", "-i", rep, "--page", "raw", "--csv"], capture_output=True, text=True).stdout
    rows = list(csv.reader(io.StringIO(out)))
    h, units, data = rows[0], rows[1], rows[2:]
    col = {n: i for i, n in enumerate(h)}
    for r in data:
        print(f"== {r[col['Kernel Name']][:100]}")
        for k, label in KEYS:
            if k in col:
                print(f"   {label:22s} {r[col[k]]:>18s} {units[col[k]]}")
        st = sorted(((h[i], r[i]) for i in range(len(h)) if h[i].startswith("smsp__average_warps_issue_stalled")
                     and h[i].endswith("_per_issue_active.ratio")), key=lambda x: -float(x[1] or 0))[:5]
        print("   top stalls (cycles per issued instruction): " + ", ".join(
            f"{n.split('stalled_')[1].split('_per')[0]}={float(v):.2f}" for n, v in st))


if __name__ == "__main__":
    main(sys.argv[1])
