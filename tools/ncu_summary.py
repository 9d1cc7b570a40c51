"""Summarise an `ncu --page raw --csv` export of one kernel launch (profiles/r01_ncu_*.txt)
and record its DRAM traffic per launch in profiles/ncu_traffic.json (bench.py roofline.traffic).

    python tools/ncu_summary.py gpurun_out/ncu_full_C4_raw.csv C4_k4w2d1 "C4 NW dim=32768 ..." > profiles/r01_ncu_C4.txt
"""
import csv
import json
import os
import sys

KEYS = ["gpu__time_duration.sum", "dram__bytes_read.sum", "dram__bytes_write.sum",
        "gpu__dram_throughput.avg.pct_of_peak_sustained_elapsed", "dram__bytes.sum.per_second",
        "sm__throughput.avg.pct_of_peak_sustained_elapsed", "smsp__issue_active.avg.pct_of_peak_sustained_active",
        "sm__warps_active.avg.pct_of_peak_sustained_active", "smsp__inst_executed.sum",
        "sm__inst_executed_pipe_alu.avg.pct_of_peak_sustained_active",
        "sm__inst_executed_pipe_fma.avg.pct_of_peak_sustained_active",
        "l1tex__data_pipe_lsu_wavefronts_mem_shared.sum", "launch__registers_per_thread", "launch__grid_size",
        "launch__block_size", "launch__shared_mem_per_block_dynamic", "sm__cycles_elapsed.avg.per_second",
        "smsp__average_warp_latency_issue_stalled_wait", "smsp__warp_issue_stalled_wait_per_warp_active.pct",
        "smsp__warp_issue_stalled_short_scoreboard_per_warp_active.pct",
        "smsp__warp_issue_stalled_long_scoreboard_per_warp_active.pct",
        "smsp__warp_issue_stalled_branch_resolving_per_warp_active.pct",
        "smsp__warp_issue_stalled_sleeping_per_warp_active.pct"]
SCALE = {"byte": 1, "Kbyte": 1e3, "Mbyte": 1e6, "Gbyte": 1e9, "Tbyte": 1e12}


def main():
    path, key = sys.argv[1], sys.argv[2]
    title = sys.argv[3] if len(sys.argv) > 3 else key
    rows = list(csv.reader(open(path)))
    hdr, units, vals = rows[0], rows[1], rows[2]
    get = {h: (v, u) for h, u, v in zip(hdr, units, vals)}
    print(f"# ncu --set full --clock-control none, {title}")
    print(f"# kernel: {get.get('Kernel Name', ('?', ''))[0][:110]}")
    nbytes = 0.0
    for k in KEYS:
        if k in get:
            v, u = get[k]
            print(f"{k} = {v} {u}")
            if k in ("dram__bytes_read.sum", "dram__bytes_write.sum"):
                nbytes += float(v.replace(",", "")) * SCALE.get(u.strip(), 1)
    print(f"traffic_bytes_per_launch = {int(nbytes)}  (dram__bytes_read.sum + dram__bytes_write.sum)")
    tp = os.path.join(os.path.dirname(os.path.dirname(os.path.abspath(__file__))), "profiles", "ncu_traffic.json")
    try:
        d = json.load(open(tp))
    except Exception:
        d = {}
    d[key] = int(nbytes)
    json.dump(d, open(tp, "w"), indent=1, sort_keys=True)


if __name__ == "__main__":
    main()
