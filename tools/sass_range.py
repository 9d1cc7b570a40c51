"""Print the SASS instructions of a cleaned cuobjdump listing between two addresses.

    python tools/sass_range.py listing.sass 0x3c10 0x48d0
"""
import re
import sys

path, lo, hi = sys.argv[1], int(sys.argv[2], 16), int(sys.argv[3], 16)
for line in open(path):
    m = re.match(r'\s*/\*([0-9a-f]+)\*/\s+(.*)', line)
    if m and lo <= int(m.group(1), 16) <= hi:
        print(m.group(1), m.group(2).rstrip())
