"""Stall-on-flag fraction of one kernel launch from an `ncu --page source --csv --print-source cuda,sass`
export (tools/gpu_stall.sh): every SASS instruction's warp-stall samples are attributed to a code
region (the compute warps' dependency waits, their cell / publish work, the I/O-feeder warp, the
x-staging warp), and the share of samples in flag / counter polling is reported.

    python tools/ncu_flag_stall.py gpurun_out/st_C4_cs.csv nw  > profiles/r01_stall_C4.txt

Inlined helpers (ld.volatile wrappers, __nanosleep, the watchdog) carry their own file:line, so an
instruction is assigned the region of the nearest preceding instruction (in address order) whose
line lies inside a region of the kernel's own source file; the spin loops' helper instructions
therefore inherit the loop's region.
"""
import collections
import csv
import sys

# (file suffix, first line, last line, region) -- line ranges of the sources as committed
REGIONS = {
    "nw": [
        ("wf_nw.cuh", 311, 339, "compute: dependency wait (wait_ctr: west feed / x ring / ring slot)"),
        ("wf_nw.cuh", 143, 310, "compute: cells, staging, write-back"),
        ("wf_nw.cuh", 340, 607, "compute: row blocks, TMA store, publish"),
        ("wf_nw.cuh", 614, 751, "I/O warp: west feed + east forward (polls LL ring / counters)"),
        ("wf_nw.cuh", 756, 784, "x warp: row-code staging (polls consumer counters)"),
        ("wf_nw.cuh", 786, 834, "kernel entry / exit"),
    ],
    "nw8": [
        ("wf_nw8.cu", 271, 325, "compute: cell step (DPX chain, staging STS, east hand-off)"),
        ("wf_nw8.cu", 326, 372, "compute: block (x codes, west ring LDS, east quads)"),
        ("wf_nw8.cu", 373, 387, "compute: TMA store publish (tail only)"),
        ("wf_nw8.cu", 388, 398, "compute: block barrier (lockstep wait)"),
        ("wf_nw8.cu", 399, 442, "compute: lag / drain barriers, run loop"),
        ("wf_nw8.cu", 193, 270, "compute: setup"),
        ("wf_nw8.cu", 446, 463, "helper: spin on a stale global quad (stall on flag)"),
        ("wf_nw8.cu", 557, 585, "storer warp: TMA output stores + its barriers"),
        ("wf_nw8.cu", 476, 556, "helper warp: inbound ring + its barriers"),
        ("wf_nw8.cu", 586, 655, "helper warp: inbound ring + its barriers"),
        ("wf_nw8.cu", 657, 708, "kernel entry / dispatch / exit"),
    ],
    "syn": [
        ("wf_syn.cu", 236, 248, "compute: dependency wait (wait_ctr: west hand-off / ring slot)"),
        ("wf_syn.cu", 118, 235, "compute: cells, staging, next-row word loads"),
        ("wf_syn.cu", 249, 301, "compute: step loop (lane hand-off shuffles, east LL stores)"),
        ("wf_syn.cu", 303, 387, "compute: block loop, TMA store, publish"),
        ("wf_syn.cu", 397, 467, "feeder warp: west words from the LL ring (polls)"),
        ("wf_syn.cu", 470, 535, "kernel entry / exit"),
    ],
}
POLL = ("dependency wait", "I/O warp", "x warp", "feeder warp")


def main():
    path, kind = sys.argv[1], sys.argv[2]
    regs = REGIONS[kind]
    rows = list(csv.reader(open(path)))
    hdr = None
    fname, line = "", 0
    insts = []   # (addr, file, line, samples, stall dict)
    for r in rows:
        if not r:
            continue
        if r[0] == "File Path":
            fname = r[1]
            continue
        if r[0] == "Line No":
            hdr = r
            ix = {h: i for i, h in enumerate(hdr)}
            stall_cols = [h for h in hdr if h.startswith("stall_") and "Not Issued" not in h]
            continue
        if hdr is None:
            continue
        if r[0].isdigit():
            line = int(r[0])
            continue
        if len(r) > 4 and r[0] == "" and r[2].startswith("0x"):
            try:
                s = int(r[ix["Warp Stall Sampling (All Samples)"]] or 0)
            except (ValueError, IndexError):
                continue
            st = {}
            for h in stall_cols:
                try:
                    st[h[6:]] = int(r[ix[h]] or 0)
                except (ValueError, IndexError):
                    pass
            insts.append((int(r[2], 16), fname, line, s, st, r[3].strip()))

    def own(f, ln):
        for suf, a, b, name in regs:
            if f.endswith(suf) and a <= ln <= b:
                return name
        return None

    # an instruction listed under several source lines (inline stack) counts once, preferably
    # under a line of the kernel's own file
    by_addr = {}
    for ins in insts:
        prev = by_addr.get(ins[0])
        if prev is None or (own(prev[1], prev[2]) is None and own(ins[1], ins[2]) is not None):
            by_addr[ins[0]] = ins
    insts = sorted(by_addr.values())

    tot = collections.Counter()
    why = collections.defaultdict(collections.Counter)
    cur = "kernel entry / exit"
    for addr, f, ln, s, st, sass in insts:
        reg = own(f, ln)
        if reg is not None:
            cur = reg
        tot[cur] += s
        for k, v in st.items():
            why[cur][k] += v
    S = sum(tot.values())
    print(f"# warp-stall samples by code region, {path.split('/')[-1]} ({kind}); {len(insts)} SASS instructions, {S} samples")
    for reg, v in tot.most_common():
        top = ", ".join(f"{k} {c / max(v, 1) * 100:.0f}%" for k, c in why[reg].most_common(3))
        print(f"{v / S * 100:6.1f}%  {reg:70s} [{top}]")
    poll = sum(v for reg, v in tot.items() if any(p in reg for p in POLL))
    comp = sum(v for reg, v in tot.items() if reg.startswith("compute"))
    cwait = sum(v for reg, v in tot.items() if reg.startswith("compute") and "dependency wait" in reg)
    print(f"stall_on_flag_fraction (all warps: samples in flag / counter polling) = {poll / S:.3f}")
    print(f"compute_warps_wait_fraction (compute-warp samples in dependency waits) = {cwait / max(comp, 1):.3f}")


if __name__ == "__main__":
    main()
