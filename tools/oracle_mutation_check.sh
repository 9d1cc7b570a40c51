#!/usr/bin/env bash
# Mutation check of the oracle pins: each plausible mistake below
# (dropped term, wrong constant, off-by-one trip count, wrong shift, transposed operand,
# wrong mask, wrong operand, missing floor) must make `pytest -m "not gpu"` fail.
set -u
cd "$(dirname "$0")/.."
cp oracle/oracle.c /tmp/oracle.c.bak
trap 'cp /tmp/oracle.c.bak oracle/oracle.c; touch oracle/oracle.c' EXIT
fail=0
for mut in \
  's/NW + s, N + gap), W + gap/NW + s, N + gap), W + s/' \
  's/0x3F7FF000u/0x3F7FE000u/' \
  's/0x3EAAAAABu/0x3EAAAAAAu/' \
  's/t < tsize; ++t/t <= tsize; ++t/' \
  's/x ^= x >> 15;/x ^= x >> 14;/' \
  's/A\[a2 \* nstrat + b\] > A\[a \* nstrat + b\]/A[a * nstrat + a2] > A[a * nstrat + b]/' \
  's/& 255u);/\& 127u);/' \
  's/int32_t i1 = ((N.i1 - NW.i1) + 1) + W.i1;/int32_t i1 = ((N.i1 - NW.i1) + 1) + W.i0;/' \
  's/if (local) h = max2(h, 0);/;/' \
  's/(int32_t)i \* gap;   \/\* H\[i\]\[0\]/(int32_t)(i - 1) * gap;   \/* H[i][0]/' ; do
  cp /tmp/oracle.c.bak oracle/oracle.c; sed -i "$mut" oracle/oracle.c
  if cmp -s oracle/oracle.c /tmp/oracle.c.bak; then echo "MUTATION NOT APPLIED: $mut"; fail=1; continue; fi
  if timeout 600 python -m pytest tests -q -x -m "not gpu" -p no:cacheprovider >/dev/null 2>&1; then
    echo "SURVIVED: $mut"; fail=1
  else
    echo "killed:   $mut"
  fi
done
exit $fail
