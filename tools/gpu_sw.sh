timeout 900 python -m pytest tests -m gpu -x -q -k "smith or seqcmp" > gpurun_out/pytest_sw.log 2>&1; echo "pytest rc=$?"; tail -25 gpurun_out/pytest_sw.log | cut -c1-300
python - <<'PY'
import torch, numpy as np, sys
sys.path.insert(0, '.')
import workloads
from paper_conf_ppopp_mohantyc14_b200.wf import Wavefront
x, y = workloads.seqcmp_inputs(32768, 32768)
dev = torch.device('cuda', 0)
for local in (0, 1):
    w = Wavefront('seqcmp', 32768, local=local, alphabet=4, match=1, mismatch=-1, gap=-1)
    xi, yi = torch.from_numpy(x).to(dev), torch.from_numpy(y).to(dev)
    out = w.alloc_out()
    for _ in range(3): w.run(xi, yi, None, None, out=out)
    w.sync()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    e0.record()
    for _ in range(10): w.run(xi, yi, None, None, out=out)
    e1.record(); torch.cuda.synchronize(); w.sync()
    ms = e0.elapsed_time(e1) / 10
    print('local', local, 'ms', round(ms, 4), 'GCUPS', round(32768**2 / ms / 1e6, 1), w.local_best() if local else '')
    w.close()
PY
