"""Warp-stall samples by source region of one kernel launch, from an
`ncu --page source --csv --print-source cuda,sass` export: every SASS instruction is listed under
the source line it came from; instructions of inlined helpers (intrinsics, headers) inherit the
region of the nearest preceding instruction (address order) whose line lies in FILE.

    python tools/ncu_region.py export.csv wf_nw8.cu lo:hi:name [lo:hi:name ...]
"""
import collections
import csv
import sys


def main():
    path, fsuffix = sys.argv[1], sys.argv[2]
    specs = []
    for s in sys.argv[3:]:
        lo, hi, nm = s.split(":", 2)
        specs.append((int(lo), int(hi), nm))
    fpath, line, hdr = "", None, None
    insts = []   # (addr, file, line, {stall: n})
    for r in csv.reader(open(path)):
        if not r:
            continue
        if r[0] == "File Path":
            fpath = r[1]
            continue
        if r[0] == "Line No":
            hdr = {h: i for i, h in enumerate(r)}
            stall_cols = [(i, h[6:]) for i, h in enumerate(r) if h.startswith("stall_") and "Not Issued" not in h]
            continue
        if hdr is None or r[0] == "Function Name":
            continue
        if r[0]:
            line = int(r[0]) if r[0].isdigit() else None
            continue
        a = r[2]
        if not a.startswith("0x"):
            continue
        st = {}
        for i, h in stall_cols:
            try:
                v = int(r[i])
            except ValueError:
                v = 0
            if v:
                st[h] = v
        insts.append((int(a, 16), fpath, line, st))
    insts.sort()
    agg = collections.defaultdict(collections.Counter)
    cur = "other"
    for a, f, ln, st in insts:
        if f.endswith(fsuffix) and ln is not None:
            cur = next((nm for lo, hi, nm in specs if lo <= ln <= hi), "other")
        for k, v in st.items():
            agg[cur][k] += v
    tot = sum(sum(c.values()) for c in agg.values())
    for nm, c in sorted(agg.items(), key=lambda kv: -sum(kv[1].values())):
        s = sum(c.values())
        top = ", ".join(f"{k} {v / s * 100:.0f}%" for k, v in c.most_common(6))
        print(f"{nm:34s} {s:7d} ({s / max(tot, 1) * 100:4.1f}%)  {top}")


if __name__ == "__main__":
    main()
