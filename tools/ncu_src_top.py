"""Summarise an ncu --page source --csv (SASS) export: top stall reasons and hottest instructions.
    python tools/ncu_src_top.py gpurun_out/ncu_X_src.csv [N]"""
import csv, sys, collections
rows = list(csv.reader(open(sys.argv[1])))
hdr = rows[1]
ix = {h: i for i, h in enumerate(hdr)}
data = rows[2:]
stall_cols = [h for h in hdr if h.startswith("stall_") and "Not Issued" not in h]
tot = collections.Counter()
for r in data:
    for h in stall_cols:
        try: tot[h] += int(r[ix[h]])
        except ValueError: pass
S = sum(tot.values())
print("samples", S)
for h, v in tot.most_common(10): print(f"  {h:26s} {v / S * 100:5.1f}%")
n = int(sys.argv[2]) if len(sys.argv) > 2 else 25
hot = sorted(data, key=lambda r: -int(r[ix["Warp Stall Sampling (All Samples)"]] or 0))[:n]
for r in hot:
    st = sorted(((int(r[ix[h]] or 0), h[6:]) for h in stall_cols), reverse=True)[:3]
    print(f"{r[ix['Address']][-5:]} {int(r[ix['Warp Stall Sampling (All Samples)']]):7d} {r[ix['Source']].strip()[:60]:60s} {st}")
