import sys; sys.path.insert(0, '.')
import numpy as np, torch, workloads
from paper_conf_ppopp_mohantyc14_b200.wf import Wavefront
dim = int(sys.argv[1]); k, w, d = (int(s) for s in sys.argv[2].split(','))
x, y = workloads.seqcmp_inputs(dim)
dev = torch.device('cuda')
wf = Wavefront('seqcmp', dim, lane_cols=k, warps=w, skew=d, alphabet=4)
out = wf.run(torch.from_numpy(x).to(dev), torch.from_numpy(y).to(dev))
wf.sync(); print('ok', out[0][-1, -1].item())
