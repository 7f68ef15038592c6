import numpy as np, torch, sys
sys.path.insert(0, '.')
import paper_journals_pvldb_heimelspmm13_b200 as ocl
from tests.test_distributed_cpu import route_of
DEV = torch.device("cuda", 0)
keys = np.array([885431098730, 946836666106, 505846784907, 1016073673741, 1, 2, 3, 4, 5, 6, 7, 8], np.int64)
rows = np.zeros((len(keys), 4), np.int64); rows[:, 0] = keys; rows[:, 1] = np.arange(len(keys))
part = torch.from_numpy(rows.view(np.uint8).reshape(len(keys), 32).copy()).to(DEV)
cnt = torch.tensor([len(keys)], dtype=torch.int64, device=DEV)
for P in (2, 3, 4):
    routed, counts = ocl.route_partials(part, cnt, P)
    torch.cuda.synchronize()
    r = routed.cpu().numpy().view(np.int64)
    print(P, "gpu counts", counts.tolist(), "numpy", np.bincount(route_of(keys.view(np.uint64), P).astype(np.int64), minlength=P).tolist())
    print("   routed order", r[:, 1].tolist(), "dest numpy", route_of(r[:, 0].view(np.uint64), P).tolist())
