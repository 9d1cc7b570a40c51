"""Per-instruction view of the hottest SASS of one kernel from `ncu --page source --csv
--print-source sass`: address, instructions executed, warp-stall samples (total / wait /
short scoreboard / long scoreboard / selected / sleeping), instruction text.

    python tools/ncu_hot_sass.py export.csv [min_executed] [max_lines]
"""
import csv
import sys

rows = list(csv.reader(open(sys.argv[1])))
lo = float(sys.argv[2]) if len(sys.argv) > 2 else 1e5
cap = int(sys.argv[3]) if len(sys.argv) > 3 else 400
hdr = rows[1]
ix = {h: i for i, h in enumerate(hdr)}
cols = ["# Samples", "stall_wait", "stall_short_sb", "stall_long_sb", "stall_selected", "stall_sleep",
        "stall_branch_resolving"]
tot = {c: 0 for c in cols}
n = 0
print("addr    exec     " + " ".join(f"{c[6:12] if c.startswith('stall') else 'samp':>6}" for c in cols) + "  sass")
for r in rows[2:]:
    try:
        ex = float(r[ix["Instructions Executed"]])
    except (ValueError, IndexError):
        continue
    for c in cols:
        tot[c] += float(r[ix[c]] or 0)
    if ex >= lo and n < cap:
        n += 1
        print(f"{r[0][-5:]} {ex:9.0f} " + " ".join(f"{float(r[ix[c]] or 0):6.0f}" for c in cols) + "  " + r[1].strip())
print("totals:", {c: int(v) for c, v in tot.items()})
