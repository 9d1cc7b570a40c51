"""List the loops (backward branches) of a cleaned SASS listing that contain N shuffles,
with their instruction mix -- a quick per-step instruction count of the sweep's inner loop.

    python tools/sass_loops.py listing.sass [N]
"""
import re
import sys
from collections import Counter

path = sys.argv[1]
want = int(sys.argv[2]) if len(sys.argv) > 2 else 8
ins = []
for line in open(path):
    m = re.match(r'\s*/\*([0-9a-f]+)\*/\s+(.*)', line)
    if m:
        ins.append((int(m.group(1), 16), m.group(2).strip()))
for a, x in ins:
    mm = re.search(r'BRA[^0-9]*(0x[0-9a-f]+)', x)
    if mm and int(mm.group(1), 16) < a:
        lo = int(mm.group(1), 16)
        body = [y for b, y in ins if lo <= b <= a]
        if sum('SHFL' in y for y in body) == want:
            c = Counter((y.split()[1] if y.startswith('@') else y.split()[0]) for y in body)
            print(hex(lo), hex(a), 'instrs', len(body), dict(c.most_common(14)))
