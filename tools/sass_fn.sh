#!/usr/bin/env bash
# tools/sass_fn.sh LIB.so NAME_SUBSTRING  -> SASS of the first kernel whose mangled name contains it
cuobjdump -sass "$1" | awk -v pat="$2" '/Function :/{p = index($0, pat) > 0 && !done; if (p) done = 1} p'
